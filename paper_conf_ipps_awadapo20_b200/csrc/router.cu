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
};

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
  RT_CK(grow(r.ssrc, n_ops * 4 + 4));
  RT_CK(grow(r.sdst, n_ops * 4 + 4));
  if (with_w) RT_CK(grow(r.sw, n_ops * 4 + 4));
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
  k_route_scatter<<<kRouteBlocks, kRouteThreads, 0, s>>>(
      src, dst, w, n, n_ops, P, as<u64>(r.offs), as<u32>(r.ssrc), as<u32>(r.sdst),
      with_w ? as<u32>(r.sw) : nullptr, keep_pos ? as<u64>(r.pos) : nullptr);
  note_kernel(1);
  RT_CK(cudaGetLastError());
  RT_NC(N.AllGather(meta_mine, r.meta_all.p, P + 1, ncclUint64, r.comm, s));
  RT_CK(cudaMemcpyAsync(r.h_meta, r.meta_all.p, (size_t)P * (P + 1) * 8, cudaMemcpyDeviceToHost, s));
  RT_CK(cudaStreamSynchronize(s));
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
      cudaMallocHost(&r->h_scalar, 64) != cudaSuccess) {
    router_destroy(r);
    return DG_ERR_CUDA;
  }
  *out = r;
  return DG_OK;
}

void router_destroy(Router* r) {
  if (!r) return;
  const Nccl& N = nccl();
  if (r->comm && N.ok) N.CommDestroy(r->comm);
  Router::Buf* all[] = {&r->ssrc, &r->sdst, &r->sw, &r->rsrc, &r->rdst, &r->rw, &r->pos,
                        &r->blockcnt, &r->offs, &r->meta_all, &r->flag, &r->rfound, &r->rwt,
                        &r->sfound, &r->swt, &r->ids, &r->ids2, &r->scalar};
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
  if ((st = route_exchange(g, true, s)) != DG_OK) return st;
  if ((st = reset_counters(g, s)) != DG_OK) return st;
  Router& r = *g->router;
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
  if ((st = route_exchange(g, false, s)) != DG_OK) return st;
  if ((st = reset_counters(g, s)) != DG_OK) return st;
  Router& r = *g->router;
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
  if ((st = route_exchange(g, false, s)) != DG_OK) return st;
  const u64 total = r.roff[r.P];
  RT_CK(grow(r.rfound, total + 1));
  RT_CK(grow(r.rwt, total * 4 + 4));
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

static dg_status allreduce_u64(dg_graph g, u64* v, ncclRedOp_t op, cudaStream_t s) {
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
