// router.cu — multi-GPU batch router (a2, a11 of DESIGN.md §2): shards every edge
// op by source vertex, owner(u) = u mod P, local row = u / P, over NCCL.
//
// Per routed batch (each rank holds its own slice of the batch):
//   1. k_route_count: one pass over the slice — range validation (Q7) and a
//      per-block histogram of owners (block-contiguous op ranges);
//   2. k_route_scan: per-block send offsets, grouped by destination rank;
//   3. k_route_scatter: ops written to the send buffers (SoA) at their offsets;
//      queries keep pos[i] = send position to put answers back in order;
//   4. ncclAllGather of each rank's P send counts + its validation flag: every
//      rank learns its receive counts and the batch-wide verdict (all-or-nothing
//      before any mutation);
//   5. grouped ncclSend/ncclRecv of (src, dst[, w]) to the owners;
//   6. the local probe kernel on the received ops;
//   7. queries: (found, weight) travel back through the reversed exchange and are
//      scattered to the caller's order through pos.
// Fused exchange (default when every peer's memory can be mapped; DG_ROUTER=nccl
// selects the path above): steps 3 and 5 become ONE kernel.  Each rank owns a
// receive window (plain device memory exported with CUDA IPC and mapped by every
// peer over NVLink / NVSwitch); after the counts all-gather every rank knows where
// its ops land in every owner's window, and k_route_scatter stores each op straight
// into its owner's window (peer stores) instead of a local send buffer.  The last
// block of the kernel fences (system scope) and bumps an arrival counter in every
// peer's window header; a one-thread kernel on the owner waits for P arrivals
// before the probe kernel reads the window.  Query answers return the same way:
// the owner's k_route_return stores (found, weight) into each asker's answer window
// and signals it.  The next batch's counts all-gather orders window reuse (a rank
// reaches it only after its kernels of the previous batch completed).
// The paper has a single GPU; this layer is the B200-node extension
// named by BASELINE.json's north_star.  NCCL is loaded with dlopen (the copy torch
// already loaded when present), so libdg.so has no link-time NCCL dependency.
#include <dlfcn.h>

#include <algorithm>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <vector>

#include <nccl.h>

#include "graph.h"
#include "kernels.h"
#include "router.h"

namespace dg {
namespace {

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

constexpr int kRouteBlocks = 1184;  // 148 SMs x 8
constexpr int kRouteThreads = 256;
constexpr int kMaxRanks = 64;

// ------------------------------------------------------------------ kernels ----
__device__ __forceinline__ void op_at(const u32* src, const u32* dst, u64 n, u64 j, u32& u,
                                      u32& v, u64& i) {
  if (j < n) { i = j; u = src[j]; v = dst[j]; }
  else { i = j - n; u = dst[i]; v = src[i]; }  // undirected mirror op
}

__global__ void k_route_count(const u32* src, const u32* dst, u64 n, u64 n_ops, u64 nv, u32 P,
                              u32* blockcnt, u32* flag) {
  __shared__ u32 cnt[kMaxRanks];
  for (u32 p = threadIdx.x; p < P; p += blockDim.x) cnt[p] = 0;
  __syncthreads();
  const u64 per = (n_ops + gridDim.x - 1) / gridDim.x;
  const u64 lo = (u64)blockIdx.x * per, hi = min(n_ops, lo + per);
  bool bad = false;
  for (u64 j = lo + threadIdx.x; j < hi; j += blockDim.x) {
    u32 u, v;
    u64 i;
    op_at(src, dst, n, j, u, v, i);
    if ((u64)u >= nv || (u64)v >= nv) {
      bad = true;
      continue;
    }
    atomicAdd(&cnt[u % P], 1u);
  }
  if (__any_sync(0xFFFFFFFFu, bad) && (threadIdx.x & 31) == 0) atomicOr(flag, 1u);
  __syncthreads();
  for (u32 p = threadIdx.x; p < P; p += blockDim.x) blockcnt[blockIdx.x * P + p] = cnt[p];
}

// offs[b*P + p] = start of block b's ops for rank p; meta[p] = ops for rank p;
// meta[P] = validation flag (P+1 u64 per rank, all-gathered next).
__global__ void k_route_scan(const u32* blockcnt, u32 nblocks, u32 P, u64* offs, u64* meta,
                             const u32* flag) {
  __shared__ u64 tot[kMaxRanks];
  const u32 p = threadIdx.x;
  if (p < P) {
    u64 s = 0;
    for (u32 b = 0; b < nblocks; ++b) s += blockcnt[b * P + p];
    tot[p] = s;
  }
  __syncthreads();
  if (p < P) {
    u64 base = 0;
    for (u32 q = 0; q < p; ++q) base += tot[q];
    for (u32 b = 0; b < nblocks; ++b) {
      offs[b * P + p] = base;
      base += blockcnt[b * P + p];
    }
    meta[p] = tot[p];
  }
  if (p == 0) meta[P] = *flag;
}

__global__ void k_route_scatter(const u32* src, const u32* dst, const u32* w, u64 n, u64 n_ops,
                                u32 P, const u64* offs, u32* ssrc, u32* sdst, u32* sw, u64* pos) {
  __shared__ unsigned long long cur[kMaxRanks];
  for (u32 p = threadIdx.x; p < P; p += blockDim.x) cur[p] = offs[blockIdx.x * P + p];
  __syncthreads();
  const u64 per = (n_ops + gridDim.x - 1) / gridDim.x;
  const u64 lo = (u64)blockIdx.x * per, hi = min(n_ops, lo + per);
  for (u64 j = lo + threadIdx.x; j < hi; j += blockDim.x) {
    u32 u, v;
    u64 i;
    op_at(src, dst, n, j, u, v, i);
    const u64 slot = atomicAdd(&cur[u % P], 1ull);
    ssrc[slot] = u;
    sdst[slot] = v;
    if (sw) sw[slot] = w ? w[i] : 0u;
    if (pos) pos[j] = slot;
  }
}

__global__ void k_route_unpermute(const u64* pos, u64 n, const uint8_t* fs, const u32* ws,
                                  uint8_t* found, u32* wout) {
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 j = (u64)blockIdx.x * blockDim.x + threadIdx.x; j < n; j += stride) {
    const u64 s = pos[j];
    found[j] = fs[s];
    if (wout) wout[j] = ws[s];
  }
}

// ---------------------------------------------------------- fused exchange ----
constexpr u64 kWinHdr = 256;  // window header bytes

struct WinHdr {
  unsigned long long arrive;      // ops-window arrivals (monotonic, +1 per peer per batch)
  unsigned long long ans_arrive;  // answer-window arrivals
  unsigned int done;              // blocks of the local scatter / return kernel finished
  unsigned int done_ret;
};

// where this rank's ops go (device copy, rebuilt every batch)
struct RouteTable {
  u32* src[kMaxRanks];        // owner p's window arrays
  u32* dst[kMaxRanks];
  u32* w[kMaxRanks];
  unsigned long long* arrive[kMaxRanks];      // owner p's arrival counter
  unsigned long long base[kMaxRanks];         // my first slot in owner p's window
  unsigned long long soff[kMaxRanks];         // my first send slot for owner p
  // query answers: for asker q, the ops it sent me occupy my window
  // [roff[q], roff[q+1]) and return to its answer window at aoff[q]
  uint8_t* afound[kMaxRanks];
  u32* awt[kMaxRanks];
  unsigned long long* ans_arrive[kMaxRanks];
  unsigned long long roff[kMaxRanks + 1];
  unsigned long long aoff[kMaxRanks];
};

__device__ __forceinline__ unsigned long long ld_acquire_sys(const unsigned long long* p) {
  unsigned long long v;
  asm volatile("ld.acquire.sys.global.u64 %0, [%1];" : "=l"(v) : "l"(p) : "memory");
  return v;
}

// last block of a grid: fence (system scope) and bump every peer's counter
__device__ __forceinline__ void signal_peers(unsigned int* done, unsigned long long* const* ctr,
                                             u32 P) {
  __threadfence_system();
  __syncthreads();
  if (threadIdx.x == 0) {
    const unsigned int prev = atomicAdd(done, 1u);
    if (prev == gridDim.x - 1) {
      *done = 0;
      __threadfence_system();
      for (u32 p = 0; p < P; ++p) atomicAdd_system(ctr[p], 1ull);
    }
  }
}

// steps 3 + 5 in one kernel: ops are stored straight into their owners' windows
__global__ void k_route_scatter_fused(const u32* src, const u32* dst, const u32* w, u64 n,
                                      u64 n_ops, u32 P, const u64* offs, const RouteTable* tb,
                                      bool with_w, u64* pos, unsigned int* done) {
  __shared__ unsigned long long cur[kMaxRanks];
  for (u32 p = threadIdx.x; p < P; p += blockDim.x) cur[p] = offs[blockIdx.x * P + p];
  __syncthreads();
  const u64 per = (n_ops + gridDim.x - 1) / gridDim.x;
  const u64 lo = (u64)blockIdx.x * per, hi = min(n_ops, lo + per);
  for (u64 j = lo + threadIdx.x; j < hi; j += blockDim.x) {
    u32 u, v;
    u64 i;
    op_at(src, dst, n, j, u, v, i);
    const u32 p = u % P;
    const u64 slot = atomicAdd(&cur[p], 1ull);
    const u64 at = tb->base[p] + (slot - tb->soff[p]);
    tb->src[p][at] = u;
    tb->dst[p][at] = v;
    if (with_w) tb->w[p][at] = w ? w[i] : 0u;
    if (pos) pos[j] = slot;
  }
  signal_peers(done, tb->arrive, P);
}

// Spins until every rank has signalled.  A peer that never arrives (a rank that
// died or skipped the collective) must not hang the device: after kWaitTimeoutNs the
// kernel raises ctl->route_timeout and returns; the host turns it into DG_ERR_NCCL at
// the next batch and the handle goes bad.
constexpr unsigned long long kWaitTimeoutNs = 30ull * 1000 * 1000 * 1000;

__device__ __forceinline__ unsigned long long globaltimer_ns() {
  unsigned long long t;
  asm volatile("mov.u64 %0, %globaltimer;" : "=l"(t));
  return t;
}

__global__ void k_route_wait(const unsigned long long* ctr, unsigned long long expected,
                             DevCtl* ctl) {
  if (threadIdx.x != 0) return;
  const unsigned long long t0 = globaltimer_ns();
  while (ld_acquire_sys(ctr) < expected) {
    __nanosleep(64);
    if (globaltimer_ns() - t0 > kWaitTimeoutNs) {
      atomicExch(&ctl->route_timeout, 1u);
      return;
    }
  }
}

// query answers back to the askers' answer windows (a11), in send order
__global__ void k_route_return(const uint8_t* found, const u32* wt, u32 P, const RouteTable* tb,
                               unsigned int* done) {
  const u64 total = tb->roff[P];
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 k = (u64)blockIdx.x * blockDim.x + threadIdx.x; k < total; k += stride) {
    u32 q = 0;
    while (q + 1 < P && tb->roff[q + 1] <= k) ++q;
    const u64 at = tb->aoff[q] + (k - tb->roff[q]);
    tb->afound[q][at] = found[k];
    tb->awt[q][at] = wt[k];
  }
  signal_peers(done, tb->ans_arrive, P);
}

}  // namespace

struct Router {
  ncclComm_t comm = nullptr;
  u32 P = 1, rank = 0;
  struct Buf {
    void* p = nullptr;
    size_t bytes = 0;
  };
  Buf ssrc, sdst, sw, rsrc, rdst, rw, pos, blockcnt, offs, meta_all, flag, rfound, rwt, sfound,
      swt, ids, ids2, scalar;
  u64* h_meta = nullptr;  // pinned, P*(P+1)
  u64* h_scalar = nullptr;
  std::vector<u64> scnt, soff, rcnt, roff;
  // fused exchange: receive window [WinHdr | src | dst | w | found | wt], wcap ops
  bool fused = false;
  u64 wcap = 0;
  char* win = nullptr;
  char* peer[kMaxRanks] = {};      // mapped windows of every rank (self: win)
  std::vector<char*> retired;      // outgrown windows (peers may still map them)
  unsigned long long arrive_expected = 0, ans_expected = 0;
  Buf table;
  RouteTable* h_table = nullptr;   // pinned
};

dg_status allreduce_u64(dg_graph g, u64* v, ncclRedOp_t op, cudaStream_t s);

namespace {

cudaError_t grow(Router::Buf& b, size_t bytes) {
  if (bytes <= b.bytes) return cudaSuccess;
  if (b.p) cudaFree(b.p);
  b.p = nullptr;
  b.bytes = 0;
  const size_t want = std::max<size_t>(bytes + bytes / 8, 1 << 16);
  cudaError_t e = cudaMalloc(&b.p, want);
  if (e == cudaSuccess) b.bytes = want;
  return e;
}

#define RT_CK(expr)                       \
  do {                                    \
    if ((expr) != cudaSuccess) {          \
      g->bad = true;                      \
      return DG_ERR_CUDA;                 \
    }                                     \
  } while (0)
#define RT_NC(expr)                       \
  do {                                    \
    if ((expr) != ncclSuccess) {          \
      g->bad = true;                      \
      return DG_ERR_NCCL;                 \
    }                                     \
  } while (0)

template <typename T>
T* as(Router::Buf& b) {
  return reinterpret_cast<T*>(b.p);
}

// Steps 1-4: partition this rank's slice by owner and agree on counts/validity.
// Returns DG_ERR_VERTEX_OUT_OF_RANGE (on every rank) if any rank saw a bad ID.
dg_status route_partition(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n,
                          bool mirror, bool with_w, bool keep_pos, cudaStream_t s) {
  Router& r = *g->router;
  const Nccl& N = nccl();
  const u32 P = r.P;
  const u64 n_ops = mirror ? 2 * n : n;
  if (!r.fused) {  // the fused path scatters after the counts exchange, into the windows
    RT_CK(grow(r.ssrc, n_ops * 4 + 4));
    RT_CK(grow(r.sdst, n_ops * 4 + 4));
    if (with_w) RT_CK(grow(r.sw, n_ops * 4 + 4));
  }
  if (keep_pos) RT_CK(grow(r.pos, n_ops * 8 + 8));
  RT_CK(grow(r.blockcnt, (size_t)kRouteBlocks * P * 4));
  RT_CK(grow(r.offs, (size_t)kRouteBlocks * P * 8));
  RT_CK(grow(r.meta_all, (size_t)(P + 1) * (P + 1) * 8));
  RT_CK(grow(r.flag, 8));
  RT_CK(cudaMemsetAsync(r.flag.p, 0, 4, s));
  u64* meta_mine = as<u64>(r.meta_all) + (size_t)P * (P + 1);  // scratch row after the P rows
  k_route_count<<<kRouteBlocks, kRouteThreads, 0, s>>>(src, dst, n, n_ops, g->nv, P,
                                                       as<u32>(r.blockcnt), as<u32>(r.flag));
  note_kernel(1);
  k_route_scan<<<1, 64, 0, s>>>(as<u32>(r.blockcnt), kRouteBlocks, P, as<u64>(r.offs), meta_mine,
                                as<u32>(r.flag));
  note_kernel(1);
  if (!r.fused) {
    k_route_scatter<<<kRouteBlocks, kRouteThreads, 0, s>>>(
        src, dst, w, n, n_ops, P, as<u64>(r.offs), as<u32>(r.ssrc), as<u32>(r.sdst),
        with_w ? as<u32>(r.sw) : nullptr, keep_pos ? as<u64>(r.pos) : nullptr);
    note_kernel(1);
  }
  RT_CK(cudaGetLastError());
  RT_NC(N.AllGather(meta_mine, r.meta_all.p, P + 1, ncclUint64, r.comm, s));
  RT_CK(cudaMemcpyAsync(r.h_meta, r.meta_all.p, (size_t)P * (P + 1) * 8, cudaMemcpyDeviceToHost, s));
  RT_CK(cudaMemcpyAsync(r.h_scalar + 1, &g->ctl->route_timeout, 4, cudaMemcpyDeviceToHost, s));
  RT_CK(cudaStreamSynchronize(s));
  if (reinterpret_cast<const u32*>(r.h_scalar + 1)[0]) {  // a peer never arrived (k_route_wait)
    g->bad = true;
    return DG_ERR_NCCL;
  }
  bool bad = false;
  r.scnt.assign(P, 0);
  r.rcnt.assign(P, 0);
  r.soff.assign(P + 1, 0);
  r.roff.assign(P + 1, 0);
  for (u32 q = 0; q < P; ++q) {
    bad |= r.h_meta[(size_t)q * (P + 1) + P] != 0;
    r.scnt[q] = r.h_meta[(size_t)r.rank * (P + 1) + q];
    r.rcnt[q] = r.h_meta[(size_t)q * (P + 1) + r.rank];
  }
  for (u32 q = 0; q < P; ++q) {
    r.soff[q + 1] = r.soff[q] + r.scnt[q];
    r.roff[q + 1] = r.roff[q] + r.rcnt[q];
  }
  return bad ? DG_ERR_VERTEX_OUT_OF_RANGE : DG_OK;
}

// Step 5: ship the partitioned ops to their owners.
dg_status route_exchange(dg_graph g, bool with_w, cudaStream_t s) {
  Router& r = *g->router;
  const Nccl& N = nccl();
  const u64 total = r.roff[r.P];
  RT_CK(grow(r.rsrc, total * 4 + 4));
  RT_CK(grow(r.rdst, total * 4 + 4));
  if (with_w) RT_CK(grow(r.rw, total * 4 + 4));
  Router::Buf* sb[3] = {&r.ssrc, &r.sdst, &r.sw};
  Router::Buf* rb[3] = {&r.rsrc, &r.rdst, &r.rw};
  const int arrays = with_w ? 3 : 2;
  // self segment: device copy
  for (int k = 0; k < arrays; ++k)
    if (r.scnt[r.rank])
      RT_CK(cudaMemcpyAsync(as<u32>(*rb[k]) + r.roff[r.rank], as<u32>(*sb[k]) + r.soff[r.rank],
                            r.scnt[r.rank] * 4, cudaMemcpyDeviceToDevice, s));
  RT_NC(N.GroupStart());
  for (u32 q = 0; q < r.P; ++q) {
    if (q == r.rank) continue;
    for (int k = 0; k < arrays; ++k) {
      if (r.scnt[q]) RT_NC(N.Send(as<u32>(*sb[k]) + r.soff[q], r.scnt[q], ncclUint32, q, r.comm, s));
      if (r.rcnt[q]) RT_NC(N.Recv(as<u32>(*rb[k]) + r.roff[q], r.rcnt[q], ncclUint32, q, r.comm, s));
    }
  }
  RT_NC(N.GroupEnd());
  return DG_OK;
}

// ------------------------------------------------------ fused exchange (host) ----
struct WinPtrs {
  WinHdr* hdr;
  u32 *src, *dst, *w, *wt;
  uint8_t* found;
};

WinPtrs win_ptrs(char* base, u64 cap) {
  WinPtrs x;
  x.hdr = reinterpret_cast<WinHdr*>(base);
  char* p = base + kWinHdr;
  x.src = reinterpret_cast<u32*>(p); p += cap * 4;
  x.dst = reinterpret_cast<u32*>(p); p += cap * 4;
  x.w = reinterpret_cast<u32*>(p); p += cap * 4;
  x.wt = reinterpret_cast<u32*>(p); p += cap * 4;
  x.found = reinterpret_cast<uint8_t*>(p);
  return x;
}

void close_peers(Router& r) {
  for (u32 q = 0; q < r.P; ++q) {
    if (q != r.rank && r.peer[q]) cudaIpcCloseMemHandle(r.peer[q]);
    r.peer[q] = nullptr;
  }
}

// Collective: every rank allocates a window of `cap` ops and maps every peer's
// (CUDA IPC handles all-gathered over NCCL).  If any rank cannot map a peer, all
// ranks fall back to the NCCL exchange.
dg_status window_setup(dg_graph g, u64 cap, cudaStream_t s) {
  Router& r = *g->router;
  const Nccl& N = nccl();
  close_peers(r);
  if (r.win) r.retired.push_back(r.win);
  r.win = nullptr;
  r.fused = false;
  RT_CK(cudaMalloc(&r.win, kWinHdr + cap * 17 + 64));
  RT_CK(cudaMemsetAsync(r.win, 0, kWinHdr, s));
  r.wcap = cap;
  r.arrive_expected = r.ans_expected = 0;
  r.peer[r.rank] = r.win;
  int fail = 0;
  if (r.P > 1) {
    static_assert(sizeof(cudaIpcMemHandle_t) == 64, "IPC handle size");
    cudaIpcMemHandle_t mine;
    RT_CK(grow(r.scalar, (size_t)(r.P + 1) * 64 + 64));
    char* hbuf = as<char>(r.scalar);
    if (cudaIpcGetMemHandle(&mine, r.win) != cudaSuccess) {
      cudaGetLastError();
      fail = 1;
      std::memset(&mine, 0, sizeof(mine));
    }
    RT_CK(cudaMemcpyAsync(hbuf + (size_t)r.P * 64, &mine, 64, cudaMemcpyHostToDevice, s));
    RT_NC(N.AllGather(hbuf + (size_t)r.P * 64, hbuf, 64, ncclUint8, r.comm, s));
    std::vector<cudaIpcMemHandle_t> all(r.P);
    RT_CK(cudaMemcpyAsync(all.data(), hbuf, (size_t)r.P * 64, cudaMemcpyDeviceToHost, s));
    RT_CK(cudaStreamSynchronize(s));
    for (u32 q = 0; q < r.P && !fail; ++q) {
      if (q == r.rank) continue;
      void* p = nullptr;
      if (cudaIpcOpenMemHandle(&p, all[q], cudaIpcMemLazyEnablePeerAccess) != cudaSuccess) {
        cudaGetLastError();
        fail = 1;
      } else {
        r.peer[q] = reinterpret_cast<char*>(p);
      }
    }
    u64 v = fail;
    dg_status st = allreduce_u64(g, &v, ncclMax, s);
    if (st != DG_OK) return st;
    fail = v != 0;
  }
  if (fail) {
    close_peers(r);
    return DG_OK;  // NCCL exchange from now on
  }
  r.fused = true;
  return DG_OK;
}

// Fused steps 3 + 5 for the counts agreed by route_partition: ops land in their
// owners' windows; returns once the local window is complete (stream-ordered).
dg_status route_fused_scatter(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n,
                              bool mirror, bool with_w, bool keep_pos, cudaStream_t s) {
  Router& r = *g->router;
  const u32 P = r.P, me = r.rank;
  const u64 n_ops = mirror ? 2 * n : n;
  const u64* M = r.h_meta;  // row q: rank q's send counts per owner
  // the same capacity decision on every rank: largest inbound or outbound total
  u64 need = 0;
  for (u32 p = 0; p < P; ++p) {
    u64 in = 0, out = 0;
    for (u32 q = 0; q < P; ++q) {
      in += M[(size_t)q * (P + 1) + p];
      out += M[(size_t)p * (P + 1) + q];
    }
    need = std::max(need, std::max(in, out));
  }
  if (need > r.wcap) {
    dg_status st = window_setup(g, std::max<u64>(need + need / 4, 2 * r.wcap), s);
    if (st != DG_OK) return st;
    if (!r.fused) return DG_ERR_UNSUPPORTED;  // caller retries over NCCL
  }
  RouteTable& T = *r.h_table;
  for (u32 p = 0; p < P; ++p) {
    const WinPtrs x = win_ptrs(r.peer[p], r.wcap);
    T.src[p] = x.src;
    T.dst[p] = x.dst;
    T.w[p] = x.w;
    T.arrive[p] = &x.hdr->arrive;
    T.afound[p] = x.found;
    T.awt[p] = x.wt;
    T.ans_arrive[p] = &x.hdr->ans_arrive;
    u64 base = 0, aoff = 0;
    for (u32 q = 0; q < me; ++q) base += M[(size_t)q * (P + 1) + p];  // earlier senders to p
    for (u32 q = 0; q < me; ++q) aoff += M[(size_t)p * (P + 1) + q];  // p's ops to earlier owners
    T.base[p] = base;
    T.soff[p] = r.soff[p];
    T.aoff[p] = aoff;
    T.roff[p] = r.roff[p];
  }
  T.roff[P] = r.roff[P];
  RT_CK(grow(r.table, sizeof(RouteTable)));
  RT_CK(cudaMemcpyAsync(r.table.p, r.h_table, sizeof(RouteTable), cudaMemcpyHostToDevice, s));
  const WinPtrs mine = win_ptrs(r.win, r.wcap);
  k_route_scatter_fused<<<kRouteBlocks, kRouteThreads, 0, s>>>(
      src, dst, w, n, n_ops, P, as<u64>(r.offs), as<RouteTable>(r.table), with_w,
      keep_pos ? as<u64>(r.pos) : nullptr, &mine.hdr->done);
  r.arrive_expected += P;
  k_route_wait<<<1, 32, 0, s>>>(&mine.hdr->arrive, r.arrive_expected, g->ctl);
  note_kernel(2);
  RT_CK(cudaGetLastError());
  return DG_OK;
}

dg_status reset_counters(dg_graph g, cudaStream_t s) {
  RT_CK(cudaMemsetAsync(&g->ctl->count, 0, sizeof(u64), s));
  RT_CK(cudaMemsetAsync(&g->ctl->retry_count, 0, sizeof(u32), s));
  return DG_OK;
}

}  // namespace

dg_status router_unique_id(void* out128) {
  const Nccl& N = nccl();
  if (!N.ok) return DG_ERR_UNSUPPORTED;
  static_assert(sizeof(ncclUniqueId) == 128, "ncclUniqueId size");
  ncclUniqueId id;
  if (N.GetUniqueId(&id) != ncclSuccess) return DG_ERR_NCCL;
  std::memcpy(out128, &id, sizeof(id));
  return DG_OK;
}

dg_status router_create(dg_graph g, const void* unique_id, Router** out) {
  const Nccl& N = nccl();
  if (!N.ok) return DG_ERR_UNSUPPORTED;
  if (g->nranks > (u32)kMaxRanks) return DG_ERR_UNSUPPORTED;
  Router* r = new Router();
  r->P = g->nranks;
  r->rank = g->rank;
  ncclUniqueId id;
  std::memcpy(&id, unique_id, sizeof(id));
  if (N.CommInitRank(&r->comm, (int)r->P, id, (int)r->rank) != ncclSuccess) {
    delete r;
    return DG_ERR_NCCL;
  }
  if (cudaMallocHost(&r->h_meta, (size_t)(r->P + 1) * (r->P + 1) * 8) != cudaSuccess ||
      cudaMallocHost(&r->h_scalar, 64) != cudaSuccess ||
      cudaMallocHost(&r->h_table, sizeof(RouteTable)) != cudaSuccess) {
    router_destroy(r);
    return DG_ERR_CUDA;
  }
  *out = r;
  return DG_OK;
}

dg_status router_setup_fused(dg_graph g, cudaStream_t s) {
  const char* mode = std::getenv("DG_ROUTER");
  if (mode && std::strcmp(mode, "nccl") == 0) return DG_OK;
  return window_setup(g, 1ull << 20, s);
}

bool router_fused(const Router* r) { return r && r->fused; }

void router_destroy(Router* r) {
  if (!r) return;
  const Nccl& N = nccl();
  close_peers(*r);
  if (r->win) cudaFree(r->win);
  for (char* p : r->retired) cudaFree(p);
  if (r->h_table) cudaFreeHost(r->h_table);
  if (r->comm && N.ok) N.CommDestroy(r->comm);
  Router::Buf* all[] = {&r->ssrc, &r->sdst, &r->sw, &r->rsrc, &r->rdst, &r->rw, &r->pos,
                        &r->blockcnt, &r->offs, &r->meta_all, &r->flag, &r->rfound, &r->rwt,
                        &r->sfound, &r->swt, &r->ids, &r->ids2, &r->scalar, &r->table};
  for (auto* b : all)
    if (b->p) cudaFree(b->p);
  if (r->h_meta) cudaFreeHost(r->h_meta);
  if (r->h_scalar) cudaFreeHost(r->h_scalar);
  delete r;
}

dg_status router_insert(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n, u32 epoch,
                        cudaStream_t s) {
  dg_status st = route_partition(g, src, dst, w, n, !g->directed, true, false, s);
  if (st == DG_ERR_VERTEX_OUT_OF_RANGE) {
    // every rank agrees: no mutation; report it like the single-GPU path
    g->hctl->fail_epoch = epoch;
    RT_CK(cudaMemcpyAsync(&g->ctl->fail_epoch, &epoch, 4, cudaMemcpyHostToDevice, s));
    return reset_counters(g, s);
  }
  if (st != DG_OK) return st;
  Router& r = *g->router;
  if (r.fused) {
    if ((st = route_fused_scatter(g, src, dst, w, n, !g->directed, true, false, s)) != DG_OK)
      return st;
    if ((st = reset_counters(g, s)) != DG_OK) return st;
    const WinPtrs x = win_ptrs(r.win, r.wcap);
    return local_insert(g, x.src, x.dst, x.w, r.roff[r.P], false, epoch, s);
  }
  if ((st = route_exchange(g, true, s)) != DG_OK) return st;
  if ((st = reset_counters(g, s)) != DG_OK) return st;
  return local_insert(g, as<u32>(r.rsrc), as<u32>(r.rdst), as<u32>(r.rw), r.roff[r.P], false, epoch,
                      s);
}

dg_status router_delete(dg_graph g, const u32* src, const u32* dst, u64 n, u32 epoch,
                        cudaStream_t s) {
  dg_status st = route_partition(g, src, dst, nullptr, n, !g->directed, false, false, s);
  if (st == DG_ERR_VERTEX_OUT_OF_RANGE) {
    g->hctl->fail_epoch = epoch;
    RT_CK(cudaMemcpyAsync(&g->ctl->fail_epoch, &epoch, 4, cudaMemcpyHostToDevice, s));
    return reset_counters(g, s);
  }
  if (st != DG_OK) return st;
  Router& r = *g->router;
  if (r.fused) {
    if ((st = route_fused_scatter(g, src, dst, nullptr, n, !g->directed, false, false, s)) != DG_OK)
      return st;
    if ((st = reset_counters(g, s)) != DG_OK) return st;
    const WinPtrs x = win_ptrs(r.win, r.wcap);
    return local_delete(g, x.src, x.dst, r.roff[r.P], false, epoch, s);
  }
  if ((st = route_exchange(g, false, s)) != DG_OK) return st;
  if ((st = reset_counters(g, s)) != DG_OK) return st;
  return local_delete(g, as<u32>(r.rsrc), as<u32>(r.rdst), r.roff[r.P], false, epoch, s);
}

dg_status router_query(dg_graph g, const u32* src, const u32* dst, u64 n, uint8_t* found, u32* wout,
                       u32 epoch, cudaStream_t s) {
  Router& r = *g->router;
  const Nccl& N = nccl();
  dg_status st = route_partition(g, src, dst, nullptr, n, false, false, true, s);
  if (st == DG_ERR_VERTEX_OUT_OF_RANGE) {
    // answer 0 everywhere and report the batch as rejected (Q7/Q19)
    if (n) {
      RT_CK(cudaMemsetAsync(found, 0, n, s));
      if (wout) RT_CK(cudaMemsetAsync(wout, 0, n * 4, s));
    }
    RT_CK(cudaMemcpyAsync(&g->ctl->fail_epoch, &epoch, 4, cudaMemcpyHostToDevice, s));
    return DG_OK;
  }
  if (st != DG_OK) return st;
  const u64 total = r.roff[r.P];
  RT_CK(grow(r.rfound, total + 1));
  RT_CK(grow(r.rwt, total * 4 + 4));
  if (r.fused) {
    if ((st = route_fused_scatter(g, src, dst, nullptr, n, false, false, true, s)) != DG_OK)
      return st;
    const WinPtrs x = win_ptrs(r.win, r.wcap);
    if ((st = local_query(g, x.src, x.dst, total, as<uint8_t>(r.rfound), as<u32>(r.rwt), epoch,
                          s)) != DG_OK)
      return st;
    // answers straight into the askers' answer windows, then wait for ours (a11)
    k_route_return<<<(unsigned)g->sms * 4, 256, 0, s>>>(as<uint8_t>(r.rfound), as<u32>(r.rwt), r.P,
                                                        as<RouteTable>(r.table), &x.hdr->done_ret);
    r.ans_expected += r.P;
    k_route_wait<<<1, 32, 0, s>>>(&x.hdr->ans_arrive, r.ans_expected, g->ctl);
    note_kernel(2);
    if (n) {
      u64 blocks = std::min<u64>((n + 255) / 256, (u64)g->sms * 8);
      k_route_unpermute<<<(unsigned)blocks, 256, 0, s>>>(as<u64>(r.pos), n, x.found, x.wt, found,
                                                         wout);
      note_kernel(1);
    }
    RT_CK(cudaGetLastError());
    return DG_OK;
  }
  if ((st = route_exchange(g, false, s)) != DG_OK) return st;
  RT_CK(grow(r.sfound, n + 1));
  RT_CK(grow(r.swt, n * 4 + 4));
  if ((st = local_query(g, as<u32>(r.rsrc), as<u32>(r.rdst), total, as<uint8_t>(r.rfound),
                        as<u32>(r.rwt), epoch, s)) != DG_OK)
    return st;
  // answers travel back to the ranks that asked (a11)
  if (r.rcnt[r.rank]) {
    RT_CK(cudaMemcpyAsync(as<uint8_t>(r.sfound) + r.soff[r.rank], as<uint8_t>(r.rfound) + r.roff[r.rank],
                          r.rcnt[r.rank], cudaMemcpyDeviceToDevice, s));
    RT_CK(cudaMemcpyAsync(as<u32>(r.swt) + r.soff[r.rank], as<u32>(r.rwt) + r.roff[r.rank],
                          r.rcnt[r.rank] * 4, cudaMemcpyDeviceToDevice, s));
  }
  RT_NC(N.GroupStart());
  for (u32 q = 0; q < r.P; ++q) {
    if (q == r.rank) continue;
    if (r.rcnt[q]) {
      RT_NC(N.Send(as<uint8_t>(r.rfound) + r.roff[q], r.rcnt[q], ncclUint8, q, r.comm, s));
      RT_NC(N.Send(as<u32>(r.rwt) + r.roff[q], r.rcnt[q], ncclUint32, q, r.comm, s));
    }
    if (r.scnt[q]) {
      RT_NC(N.Recv(as<uint8_t>(r.sfound) + r.soff[q], r.scnt[q], ncclUint8, q, r.comm, s));
      RT_NC(N.Recv(as<u32>(r.swt) + r.soff[q], r.scnt[q], ncclUint32, q, r.comm, s));
    }
  }
  RT_NC(N.GroupEnd());
  if (n) {
    u64 blocks = std::min<u64>((n + 255) / 256, (u64)g->sms * 8);
    k_route_unpermute<<<(unsigned)blocks, 256, 0, s>>>(as<u64>(r.pos), n, as<uint8_t>(r.sfound),
                                                       as<u32>(r.swt), found, wout);
    note_kernel(1);
    RT_CK(cudaGetLastError());
  }
  return DG_OK;
}

dg_status router_allgather_u32(dg_graph g, const u32* ids, u64 n, int slot, const u32** all,
                               u64* all_n, cudaStream_t s) {
  Router& r = *g->router;
  Router::Buf& out = slot ? r.ids2 : r.ids;
  const Nccl& N = nccl();
  RT_CK(grow(r.scalar, (size_t)(r.P + 1) * 8));
  u64* cnts = as<u64>(r.scalar);
  RT_CK(cudaMemcpyAsync(cnts + r.P, &n, 8, cudaMemcpyHostToDevice, s));
  RT_NC(N.AllGather(cnts + r.P, cnts, 1, ncclUint64, r.comm, s));
  RT_CK(cudaMemcpyAsync(r.h_meta, cnts, (size_t)r.P * 8, cudaMemcpyDeviceToHost, s));
  RT_CK(cudaStreamSynchronize(s));
  std::vector<u64> off(r.P + 1, 0);
  for (u32 q = 0; q < r.P; ++q) off[q + 1] = off[q] + r.h_meta[q];
  const u64 total = off[r.P];
  RT_CK(grow(out, total * 4 + 4));
  if (n) RT_CK(cudaMemcpyAsync(as<u32>(out) + off[r.rank], ids, n * 4, cudaMemcpyDeviceToDevice, s));
  RT_NC(N.GroupStart());
  for (u32 q = 0; q < r.P; ++q) {
    if (q == r.rank) continue;
    if (n) RT_NC(N.Send(ids, n, ncclUint32, q, r.comm, s));
    if (r.h_meta[q]) RT_NC(N.Recv(as<u32>(out) + off[q], r.h_meta[q], ncclUint32, q, r.comm, s));
  }
  RT_NC(N.GroupEnd());
  *all = as<u32>(out);
  *all_n = total;
  return DG_OK;
}

dg_status allreduce_u64(dg_graph g, u64* v, ncclRedOp_t op, cudaStream_t s) {
  Router& r = *g->router;
  const Nccl& N = nccl();
  RT_CK(grow(r.scalar, (size_t)(r.P + 1) * 8));
  u64* d = as<u64>(r.scalar);
  r.h_scalar[0] = *v;
  RT_CK(cudaMemcpyAsync(d, r.h_scalar, 8, cudaMemcpyHostToDevice, s));
  RT_NC(N.AllReduce(d, d, 1, ncclUint64, op, r.comm, s));
  RT_CK(cudaMemcpyAsync(r.h_scalar, d, 8, cudaMemcpyDeviceToHost, s));
  RT_CK(cudaStreamSynchronize(s));
  *v = r.h_scalar[0];
  return DG_OK;
}

dg_status router_sum_u64(dg_graph g, u64* v, cudaStream_t s) { return allreduce_u64(g, v, ncclSum, s); }
dg_status router_max_u64(dg_graph g, u64* v, cudaStream_t s) { return allreduce_u64(g, v, ncclMax, s); }

}  // namespace dg
