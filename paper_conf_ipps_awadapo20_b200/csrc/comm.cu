// comm.cu — router transports (comm.h): NCCL (one process per GPU) and the
// in-process rank group (dg_group: P host threads of one process).
#include <dlfcn.h>

#include <chrono>
#include <condition_variable>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <new>
#include <vector>

#include <nccl.h>

#include "comm.h"

// ------------------------------------------------------- in-process group state --
// One per dg_group.  Collectives meet at a generation barrier; what a rank publishes
// before the barrier (a device pointer, a value, its send list) is read by the others
// after it, and the second barrier keeps it alive until everyone has read it.
struct dg_group_s {
  struct Msg {
    uint32_t peer;
    const void* p;
    size_t bytes;
  };
  uint32_t P = 0;
  std::mutex m;
  std::condition_variable cv;
  uint32_t arrived = 0;
  uint64_t gen = 0;
  bool broken = false;  // a barrier timed out: every later collective fails
  std::vector<const void*> ptr;
  std::vector<uint64_t> val;
  std::vector<int> dev;
  std::vector<const std::vector<Msg>*> sends;

  // false if the group is broken or the other ranks did not arrive in time (a rank
  // that died or skipped a collective must not hang the others forever)
  bool barrier() {
    static const long timeout_s = std::getenv("DG_GROUP_TIMEOUT_S")
                                      ? std::atol(std::getenv("DG_GROUP_TIMEOUT_S"))
                                      : 120;
    std::unique_lock<std::mutex> lk(m);
    if (broken) return false;
    const uint64_t my = gen;
    if (++arrived == P) {
      arrived = 0;
      ++gen;
      cv.notify_all();
      return true;
    }
    if (!cv.wait_for(lk, std::chrono::seconds(timeout_s), [&] { return gen != my || broken; }) ||
        broken) {
      broken = true;
      cv.notify_all();
      return false;
    }
    return true;
  }
};

namespace dg {
namespace {

// =================================================================== NCCL ========
struct Nccl {
  decltype(&ncclGetUniqueId) GetUniqueId = nullptr;
  decltype(&ncclCommInitRank) CommInitRank = nullptr;
  decltype(&ncclCommDestroy) CommDestroy = nullptr;
  decltype(&ncclSend) Send = nullptr;
  decltype(&ncclRecv) Recv = nullptr;
  decltype(&ncclGroupStart) GroupStart = nullptr;
  decltype(&ncclGroupEnd) GroupEnd = nullptr;
  decltype(&ncclAllGather) AllGather = nullptr;
  decltype(&ncclAllReduce) AllReduce = nullptr;
  bool ok = false;
};

template <typename F>
bool sym(void* h, const char* name, F& f) {
  f = reinterpret_cast<F>(dlsym(h, name));
  return f != nullptr;
}

// NCCL is loaded with dlopen (the copy torch already loaded when present), so
// libdg.so has no link-time NCCL dependency.
const Nccl& nccl() {
  static Nccl n;
  static std::once_flag once;
  std::call_once(once, [] {
    void* h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_NOLOAD);
    if (!h && std::getenv("DG_NCCL_LIB")) h = dlopen(std::getenv("DG_NCCL_LIB"), RTLD_NOW);
    if (!h) h = dlopen("libnccl.so.2", RTLD_NOW);
    if (!h) h = dlopen("libnccl.so", RTLD_NOW);
    if (!h) return;
    n.ok = sym(h, "ncclGetUniqueId", n.GetUniqueId) && sym(h, "ncclCommInitRank", n.CommInitRank) &&
           sym(h, "ncclCommDestroy", n.CommDestroy) && sym(h, "ncclSend", n.Send) &&
           sym(h, "ncclRecv", n.Recv) && sym(h, "ncclGroupStart", n.GroupStart) &&
           sym(h, "ncclGroupEnd", n.GroupEnd) && sym(h, "ncclAllGather", n.AllGather) &&
           sym(h, "ncclAllReduce", n.AllReduce);
  });
  return n;
}

#define CM_CK(expr)                              \
  do {                                           \
    if ((expr) != cudaSuccess) return DG_ERR_CUDA; \
  } while (0)
#define CM_NC(expr)                              \
  do {                                           \
    if ((expr) != ncclSuccess) return DG_ERR_NCCL; \
  } while (0)

class NcclComm final : public Comm {
 public:
  NcclComm(ncclComm_t c, uint32_t P, uint32_t r) : comm_(c), P_(P), rank_(r) {}
  ~NcclComm() override {
    if (scratch_) cudaFree(scratch_);
    if (h_) cudaFreeHost(h_);
    if (comm_ && nccl().ok) nccl().CommDestroy(comm_);
  }
  uint32_t size() const override { return P_; }
  uint32_t rank() const override { return rank_; }

  dg_status allgather(const void* send, void* recv, size_t bytes, cudaStream_t s) override {
    CM_NC(nccl().AllGather(send, recv, bytes, ncclUint8, comm_, s));
    return DG_OK;
  }
  dg_status group_start() override {
    CM_NC(nccl().GroupStart());
    return DG_OK;
  }
  dg_status send(const void* buf, size_t bytes, uint32_t peer, cudaStream_t s) override {
    CM_NC(nccl().Send(buf, bytes, ncclUint8, (int)peer, comm_, s));
    return DG_OK;
  }
  dg_status recv(void* buf, size_t bytes, uint32_t peer, cudaStream_t s) override {
    CM_NC(nccl().Recv(buf, bytes, ncclUint8, (int)peer, comm_, s));
    return DG_OK;
  }
  dg_status group_end(cudaStream_t) override {
    CM_NC(nccl().GroupEnd());
    return DG_OK;
  }
  dg_status allreduce_u64(uint64_t* dev, bool max, cudaStream_t s) override {
    CM_NC(nccl().AllReduce(dev, dev, 1, ncclUint64, max ? ncclMax : ncclSum, comm_, s));
    return DG_OK;
  }
  // CUDA IPC handles of every rank's window, all-gathered over NCCL
  dg_status map_windows(char* mine, char** peers, bool* fail, cudaStream_t s) override {
    static_assert(sizeof(cudaIpcMemHandle_t) == 64, "IPC handle size");
    *fail = false;
    peers[rank_] = mine;
    if (P_ == 1) return DG_OK;
    if (!scratch_) CM_CK(cudaMalloc(&scratch_, (size_t)(P_ + 1) * 64 + 64));
    if (!h_) CM_CK(cudaMallocHost(&h_, (size_t)(P_ + 1) * 64 + 64));
    char* hb = static_cast<char*>(h_);
    char* db = static_cast<char*>(scratch_);
    cudaIpcMemHandle_t me;
    bool bad = false;
    if (cudaIpcGetMemHandle(&me, mine) != cudaSuccess) {
      cudaGetLastError();
      bad = true;
      std::memset(&me, 0, sizeof(me));
    }
    std::memcpy(hb + (size_t)P_ * 64, &me, 64);
    CM_CK(cudaMemcpyAsync(db + (size_t)P_ * 64, hb + (size_t)P_ * 64, 64, cudaMemcpyHostToDevice, s));
    dg_status st = allgather(db + (size_t)P_ * 64, db, 64, s);
    if (st != DG_OK) return st;
    CM_CK(cudaMemcpyAsync(hb, db, (size_t)P_ * 64, cudaMemcpyDeviceToHost, s));
    CM_CK(cudaStreamSynchronize(s));
    for (uint32_t q = 0; q < P_ && !bad; ++q) {
      if (q == rank_) continue;
      cudaIpcMemHandle_t h;
      std::memcpy(&h, hb + (size_t)q * 64, 64);
      void* p = nullptr;
      if (cudaIpcOpenMemHandle(&p, h, cudaIpcMemLazyEnablePeerAccess) != cudaSuccess) {
        cudaGetLastError();
        bad = true;
      } else {
        peers[q] = static_cast<char*>(p);
      }
    }
    // agree: if any rank failed, every rank falls back
    uint64_t* v = reinterpret_cast<uint64_t*>(db + (size_t)(P_ + 1) * 64);
    const uint64_t one = bad ? 1 : 0;
    CM_CK(cudaMemcpyAsync(v, &one, 8, cudaMemcpyHostToDevice, s));
    if ((st = allreduce_u64(v, true, s)) != DG_OK) return st;
    uint64_t any = 0;
    CM_CK(cudaMemcpyAsync(&any, v, 8, cudaMemcpyDeviceToHost, s));
    CM_CK(cudaStreamSynchronize(s));
    *fail = any != 0;
    return DG_OK;
  }
  void unmap_windows(char** peers) override {
    for (uint32_t q = 0; q < P_; ++q) {
      if (q != rank_ && peers[q]) cudaIpcCloseMemHandle(peers[q]);
      peers[q] = nullptr;
    }
  }

 private:
  ncclComm_t comm_ = nullptr;
  uint32_t P_, rank_;
  void* scratch_ = nullptr;
  void* h_ = nullptr;
};

// ============================================================ in-process group ====
class GroupComm final : public Comm {
 public:
  GroupComm(dg_group g, uint32_t r, int dev) : G_(g), rank_(r), dev_(dev) {}
  uint32_t size() const override { return G_->P; }
  uint32_t rank() const override { return rank_; }

  dg_status allgather(const void* send, void* recv, size_t bytes, cudaStream_t s) override {
    CM_CK(cudaStreamSynchronize(s));  // `send` is complete
    G_->ptr[rank_] = send;
    if (!G_->barrier()) return DG_ERR_NCCL;
    for (uint32_t q = 0; q < G_->P; ++q)
      if (bytes)
        CM_CK(cudaMemcpyAsync(static_cast<char*>(recv) + (size_t)q * bytes, G_->ptr[q], bytes,
                              cudaMemcpyDefault, s));
    CM_CK(cudaStreamSynchronize(s));
    if (!G_->barrier()) return DG_ERR_NCCL;  // peers' send buffers may be reused now
    return DG_OK;
  }
  dg_status group_start() override {
    sends_.clear();
    recvs_.clear();
    return DG_OK;
  }
  dg_status send(const void* buf, size_t bytes, uint32_t peer, cudaStream_t) override {
    sends_.push_back({peer, buf, bytes});
    return DG_OK;
  }
  dg_status recv(void* buf, size_t bytes, uint32_t peer, cudaStream_t) override {
    recvs_.push_back({peer, buf, bytes});
    return DG_OK;
  }
  // receivers pull: the k-th recv from q copies the k-th send of q addressed to me
  dg_status group_end(cudaStream_t s) override {
    CM_CK(cudaStreamSynchronize(s));
    G_->sends[rank_] = &sends_;
    if (!G_->barrier()) return DG_ERR_NCCL;
    std::vector<size_t> next(G_->P, 0);
    dg_status st = DG_OK;
    for (const auto& r : recvs_) {
      const std::vector<dg_group_s::Msg>& from = *G_->sends[r.peer];
      size_t& k = next[r.peer];
      while (k < from.size() && from[k].peer != rank_) ++k;
      if (k == from.size() || from[k].bytes != r.bytes) {
        st = DG_ERR_NCCL;  // unmatched point-to-point
        break;
      }
      if (r.bytes &&
          cudaMemcpyAsync(const_cast<void*>(r.p), from[k].p, r.bytes, cudaMemcpyDefault, s) !=
              cudaSuccess)
        st = DG_ERR_CUDA;
      ++k;
    }
    if (cudaStreamSynchronize(s) != cudaSuccess && st == DG_OK) st = DG_ERR_CUDA;
    if (!G_->barrier()) return DG_ERR_NCCL;
    sends_.clear();
    recvs_.clear();
    return st;
  }
  dg_status allreduce_u64(uint64_t* dev, bool max, cudaStream_t s) override {
    uint64_t v = 0;
    CM_CK(cudaMemcpyAsync(&v, dev, 8, cudaMemcpyDeviceToHost, s));
    CM_CK(cudaStreamSynchronize(s));
    G_->val[rank_] = v;
    if (!G_->barrier()) return DG_ERR_NCCL;
    uint64_t r = 0;
    for (uint32_t q = 0; q < G_->P; ++q) r = max ? (G_->val[q] > r ? G_->val[q] : r) : r + G_->val[q];
    if (!G_->barrier()) return DG_ERR_NCCL;
    CM_CK(cudaMemcpyAsync(dev, &r, 8, cudaMemcpyHostToDevice, s));
    CM_CK(cudaStreamSynchronize(s));
    return DG_OK;
  }
  // windows are plain device pointers of one process: ranks on other GPUs need peer
  // access (NVLink); a rank that cannot get it makes every rank fall back
  dg_status map_windows(char* mine, char** peers, bool* fail, cudaStream_t) override {
    G_->ptr[rank_] = mine;
    G_->dev[rank_] = dev_;
    if (!G_->barrier()) return DG_ERR_NCCL;
    bool bad = false;
    for (uint32_t q = 0; q < G_->P; ++q) {
      peers[q] = static_cast<char*>(const_cast<void*>(G_->ptr[q]));
      const int d = G_->dev[q];
      if (d == dev_) continue;
      int can = 0;
      if (cudaDeviceCanAccessPeer(&can, dev_, d) != cudaSuccess || !can) {
        cudaGetLastError();
        bad = true;
        continue;
      }
      const cudaError_t e = cudaDeviceEnablePeerAccess(d, 0);
      if (e != cudaSuccess && e != cudaErrorPeerAccessAlreadyEnabled) bad = true;
      cudaGetLastError();
    }
    if (!G_->barrier()) return DG_ERR_NCCL;
    G_->val[rank_] = bad ? 1 : 0;
    if (!G_->barrier()) return DG_ERR_NCCL;
    bool any = false;
    for (uint32_t q = 0; q < G_->P; ++q) any = any || G_->val[q] != 0;
    if (!G_->barrier()) return DG_ERR_NCCL;
    *fail = any;
    return DG_OK;
  }
  void unmap_windows(char** peers) override {
    for (uint32_t q = 0; q < G_->P; ++q) peers[q] = nullptr;
  }
  dg_status quiesce() override { return G_->barrier() ? DG_OK : DG_ERR_NCCL; }
  bool host_ordered() const override { return true; }
  dg_status wait_peers(cudaEvent_t ev, cudaStream_t s) override {
    CM_CK(cudaEventRecord(ev, s));
    G_->ptr[rank_] = ev;
    if (!G_->barrier()) return DG_ERR_NCCL;
    for (uint32_t q = 0; q < G_->P; ++q)
      if (q != rank_)
        CM_CK(cudaStreamWaitEvent(s, static_cast<cudaEvent_t>(const_cast<void*>(G_->ptr[q])), 0));
    // (a peer re-records its event only after everyone has enqueued the wait)
    if (!G_->barrier()) return DG_ERR_NCCL;
    return DG_OK;
  }

 private:
  dg_group G_;
  uint32_t rank_;
  int dev_;
  std::vector<dg_group_s::Msg> sends_, recvs_;
};

}  // namespace

bool nccl_available() { return nccl().ok; }

dg_status nccl_unique_id(void* out128) {
  const Nccl& N = nccl();
  if (!N.ok) return DG_ERR_UNSUPPORTED;
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId size");
  ncclUniqueId id;
  if (N.GetUniqueId(&id) != ncclSuccess) return DG_ERR_NCCL;
  std::memcpy(out128, &id, sizeof(id));
  return DG_OK;
}

dg_status nccl_comm_create(const void* unique_id, uint32_t P, uint32_t rank, Comm** out) {
  const Nccl& N = nccl();
  if (!N.ok) return DG_ERR_UNSUPPORTED;
  ncclUniqueId id;
  std::memcpy(&id, unique_id, sizeof(id));
  ncclComm_t c = nullptr;
  if (N.CommInitRank(&c, (int)P, id, (int)rank) != ncclSuccess) return DG_ERR_NCCL;
  *out = new NcclComm(c, P, rank);
  return DG_OK;
}

dg_status group_comm_create(dg_group grp, uint32_t P, uint32_t rank, int device, Comm** out) {
  if (!grp || grp->P != P || rank >= P) return DG_ERR_INVALID_ARGUMENT;
  *out = new GroupComm(grp, rank, device);
  return DG_OK;
}

}  // namespace dg

extern "C" {

dg_status dg_group_create(int32_t nranks, dg_group* out) {
  if (!out || nranks < 1 || nranks > 64) return DG_ERR_INVALID_ARGUMENT;
  dg_group g = new (std::nothrow) dg_group_s();
  if (!g) return DG_ERR_OUT_OF_MEMORY;
  g->P = (uint32_t)nranks;
  g->ptr.assign(g->P, nullptr);
  g->val.assign(g->P, 0);
  g->dev.assign(g->P, -1);
  g->sends.assign(g->P, nullptr);
  *out = g;
  return DG_OK;
}

dg_status dg_group_destroy(dg_group g) {
  if (!g) return DG_ERR_INVALID_ARGUMENT;
  delete g;
  return DG_OK;
}

}  // extern "C"
