// router.cu — multi-GPU batch router (a2, a11 of DESIGN.md §1): shards every edge
// op by source vertex, owner(u) = u mod P, local row = u / P.
//
// Per routed batch (each rank holds its own slice of the batch):
//   1. k_route_count: one pass over the slice — range validation (Q7) and a
//      per-block histogram of owners over the VALID ops (block-contiguous ranges);
//   2. k_route_scan: per-block send offsets, grouped by destination rank;
//   3. k_route_scatter: valid ops written to the send buffers (SoA) at their
//      offsets; queries keep pos[i] = send position (or kNoPos for an out-of-range
//      query) to put answers back in the caller's order;
//   4. all-gather of each rank's P send counts + its validation flag: every rank
//      learns its receive counts and the batch-wide verdict (a mutating batch is
//      all-or-nothing before any mutation; a query batch answers its in-range ops
//      and reports the batch as rejected, exactly as at P = 1);
//   5. grouped send/recv of (src, dst[, w]) to the owners;
//   6. the local probe kernel on the received ops;
//   7. queries: (found, weight) travel back through the reversed exchange and are
//      scattered to the caller's order through pos.
// Fused exchange (default when every peer's memory can be mapped; DG_ROUTER=nccl or
// DG_FLAG_COPY_EXCHANGE selects the path above): steps 3 and 5 become ONE kernel.
// Each rank owns a receive window (plain device memory, mapped by every peer over
// NVLink / NVSwitch: CUDA IPC between processes, plain pointers inside one process);
// after the counts all-gather every rank knows where its ops land in every owner's
// window, and k_route_scatter_fused stores each op straight into its owner's window
// (peer stores) instead of a local send buffer.  The last block of the kernel fences
// (system scope) and bumps an arrival counter in every peer's window header; a
// one-thread kernel on the owner waits for P arrivals before the probe kernel reads
// the window (in-process rank groups order the ranks' streams with CUDA events
// instead, comm.h host_ordered()).  Query answers return the same way: the owner's k_route_return stores
// (found, weight) into each asker's answer window and signals it.  The next batch's
// counts all-gather orders window reuse (a rank reaches it only after its kernels of
// the previous batch completed).  A batch larger than the windows triggers a
// collective window re-setup; if that fails on any rank, every rank moves to the copy
// exchange for this batch and the rest of the handle's life.
// The transports (NCCL, or an in-process rank group on one or several GPUs) are in
// comm.cu.  The paper has a single GPU; this layer is the B200-node
// extension named by BASELINE.json's north_star.
#include <algorithm>
#include <cstdlib>
#include <cstring>
#include <vector>

#include "comm.h"
#include "graph.h"
#include "kernels.h"
#include "router.h"

namespace dg {
namespace {

constexpr int kRouteBlocks = 1184;  // 148 SMs x 8
constexpr int kRouteThreads = 256;
constexpr int kMaxRanks = 64;
constexpr u64 kNoPos = ~0ull;       // pos[] of a query that was not routed (out of range)

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
                                u64 nv, u32 P, const u64* offs, u32* ssrc, u32* sdst, u32* sw,
                                u64* pos) {
  __shared__ unsigned long long cur[kMaxRanks];
  for (u32 p = threadIdx.x; p < P; p += blockDim.x) cur[p] = offs[blockIdx.x * P + p];
  __syncthreads();
  const u64 per = (n_ops + gridDim.x - 1) / gridDim.x;
  const u64 lo = (u64)blockIdx.x * per, hi = min(n_ops, lo + per);
  for (u64 j = lo + threadIdx.x; j < hi; j += blockDim.x) {
    u32 u, v;
    u64 i;
    op_at(src, dst, n, j, u, v, i);
    if ((u64)u >= nv || (u64)v >= nv) {  // not routed (query batches only get here)
      if (pos) pos[j] = kNoPos;
      continue;
    }
    const u64 slot = atomicAdd(&cur[u % P], 1ull);
    ssrc[slot] = u;
    sdst[slot] = v;
    if (sw) sw[slot] = w ? w[i] : 0u;
    if (pos) pos[j] = slot;
  }
}

// answers back to the caller's order (Q19: an unrouted out-of-range query answers 0)
__global__ void k_route_unpermute(const u64* pos, u64 n, const uint8_t* fs, const u32* ws,
                                  uint8_t* found, u32* wout) {
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 j = (u64)blockIdx.x * blockDim.x + threadIdx.x; j < n; j += stride) {
    const u64 s = pos[j];
    const bool ok = s != kNoPos;
    found[j] = ok ? fs[s] : 0;
    if (wout) wout[j] = ok ? ws[s] : 0u;
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

// steps 3 + 5 in one kernel: valid ops are stored straight into their owners' windows
__global__ void k_route_scatter_fused(const u32* src, const u32* dst, const u32* w, u64 n,
                                      u64 n_ops, u64 nv, u32 P, const u64* offs,
                                      const RouteTable* tb, bool with_w, u64* pos,
                                      unsigned int* done) {
  __shared__ unsigned long long cur[kMaxRanks];
  for (u32 p = threadIdx.x; p < P; p += blockDim.x) cur[p] = offs[blockIdx.x * P + p];
  __syncthreads();
  const u64 per = (n_ops + gridDim.x - 1) / gridDim.x;
  const u64 lo = (u64)blockIdx.x * per, hi = min(n_ops, lo + per);
  for (u64 j = lo + threadIdx.x; j < hi; j += blockDim.x) {
    u32 u, v;
    u64 i;
    op_at(src, dst, n, j, u, v, i);
    if ((u64)u >= nv || (u64)v >= nv) {
      if (pos) pos[j] = kNoPos;
      continue;
    }
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
  Comm* comm = nullptr;
  u32 P = 1, rank = 0;
  struct Buf {
    void* p = nullptr;
    size_t bytes = 0;
  };
  Buf ssrc, sdst, sw, rsrc, rdst, rw, pos, blockcnt, offs, meta_all, flag, rfound, rwt, sfound,
      swt, ids, ids2, scalar, table;
  u64* h_meta = nullptr;  // pinned, P*(P+1)
  u64* h_scalar = nullptr;
  std::vector<u64> scnt, soff, rcnt, roff;
  // fused exchange: receive window [WinHdr | src | dst | w | wt | found], wcap ops
  bool fused = false;
  bool copy_only = false;          // DG_ROUTER=nccl / DG_FLAG_COPY_EXCHANGE, or a failed setup
  u32 setups = 0;                  // window setups so far
  u64 wcap = 0;
  char* win = nullptr;
  char* peer[kMaxRanks] = {};      // mapped windows of every rank (self: win)
  std::vector<char*> retired;      // outgrown windows (peers may still map them)
  unsigned long long arrive_expected = 0, ans_expected = 0;
  RouteTable* h_table = nullptr;   // pinned
  cudaEvent_t ev_done = nullptr;   // in-process groups: this rank's stores are issued
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
// a failed collective leaves the ranks out of step: the handle goes bad
#define RT_CM(expr)                       \
  do {                                    \
    const dg_status st_ = (expr);         \
    if (st_ != DG_OK) {                   \
      g->bad = true;                      \
      return st_;                         \
    }                                     \
  } while (0)

template <typename T>
T* as(Router::Buf& b) {
  return reinterpret_cast<T*>(b.p);
}

// Steps 1-4: partition this rank's slice by owner and agree on counts/validity.
// Returns DG_ERR_VERTEX_OUT_OF_RANGE (on every rank) if any rank saw a bad ID; the
// counts then cover the valid ops only (what a query batch still routes).
// Everything that may synchronise the device (allocation) happens BEFORE the counts
// exchange: after it, an in-process rank group has ranks spinning on the device for
// this rank's partition kernel (see the fused exchange).
dg_status route_partition(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n,
                          bool mirror, bool with_w, bool keep_pos, cudaStream_t s) {
  Router& r = *g->router;
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
  RT_CK(cudaGetLastError());
  RT_CM(r.comm->allgather(meta_mine, r.meta_all.p, (P + 1) * 8, s));
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

// Step 3 of the copy exchange: valid ops into the local send buffers.
dg_status route_scatter_copy(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n,
                             bool mirror, bool with_w, bool keep_pos, cudaStream_t s) {
  Router& r = *g->router;
  const u64 n_ops = mirror ? 2 * n : n;
  RT_CK(grow(r.ssrc, n_ops * 4 + 4));
  RT_CK(grow(r.sdst, n_ops * 4 + 4));
  if (with_w) RT_CK(grow(r.sw, n_ops * 4 + 4));
  k_route_scatter<<<kRouteBlocks, kRouteThreads, 0, s>>>(
      src, dst, w, n, n_ops, g->nv, r.P, as<u64>(r.offs), as<u32>(r.ssrc), as<u32>(r.sdst),
      with_w ? as<u32>(r.sw) : nullptr, keep_pos ? as<u64>(r.pos) : nullptr);
  note_kernel(1);
  RT_CK(cudaGetLastError());
  return DG_OK;
}

// Step 5: ship the partitioned ops to their owners.
dg_status route_exchange(dg_graph g, bool with_w, cudaStream_t s) {
  Router& r = *g->router;
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
  RT_CM(r.comm->group_start());
  for (u32 q = 0; q < r.P; ++q) {
    if (q == r.rank) continue;
    for (int k = 0; k < arrays; ++k) {
      if (r.scnt[q]) RT_CM(r.comm->send(as<u32>(*sb[k]) + r.soff[q], r.scnt[q] * 4, q, s));
      if (r.rcnt[q]) RT_CM(r.comm->recv(as<u32>(*rb[k]) + r.roff[q], r.rcnt[q] * 4, q, s));
    }
  }
  RT_CM(r.comm->group_end(s));
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

// Collective: every rank allocates a window of `cap` ops and maps every peer's.  If
// any rank cannot map a peer, every rank falls back to the copy exchange for good.
dg_status window_setup(dg_graph g, u64 cap, cudaStream_t s) {
  Router& r = *g->router;
  r.comm->unmap_windows(r.peer);
  if (r.win) r.retired.push_back(r.win);
  r.win = nullptr;
  r.fused = false;
  RT_CK(cudaMalloc(&r.win, kWinHdr + cap * 17 + 64));
  RT_CK(cudaMemsetAsync(r.win, 0, kWinHdr, s));
  // the owner's answer buffers hold up to a window of ops: sized here, so a fused
  // query batch allocates nothing after its counts exchange
  RT_CK(grow(r.rfound, cap + 1));
  RT_CK(grow(r.rwt, cap * 4 + 4));
  RT_CK(cudaStreamSynchronize(s));
  r.wcap = cap;
  r.arrive_expected = r.ans_expected = 0;
  bool fail = false;
  RT_CM(r.comm->map_windows(r.win, r.peer, &fail, s));
  // test hook: a failed re-setup (every rank reads the same environment)
  if (r.setups > 0 && std::getenv("DG_TEST_FUSED_REGROW_FAIL")) fail = true;
  ++r.setups;
  if (fail) {
    r.comm->unmap_windows(r.peer);
    r.copy_only = true;
    return DG_OK;  // copy exchange from now on
  }
  r.fused = true;
  return DG_OK;
}

// Fused steps 3 + 5 for the counts agreed by route_partition: ops land in their
// owners' windows; returns once the local window is complete (stream-ordered).
// *fell_back = the windows had to grow and the re-setup failed on some rank: the
// caller continues with the copy exchange (route_scatter_copy + route_exchange).
dg_status route_fused_scatter(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n,
                              bool mirror, bool with_w, bool keep_pos, bool* fell_back,
                              cudaStream_t s) {
  Router& r = *g->router;
  const u32 P = r.P, me = r.rank;
  const u64 n_ops = mirror ? 2 * n : n;
  const u64* M = r.h_meta;  // row q: rank q's send counts per owner
  *fell_back = false;
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
    if (!r.fused) {
      *fell_back = true;
      return DG_OK;
    }
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
  RT_CK(cudaMemcpyAsync(r.table.p, r.h_table, sizeof(RouteTable), cudaMemcpyHostToDevice, s));
  const WinPtrs mine = win_ptrs(r.win, r.wcap);
  k_route_scatter_fused<<<kRouteBlocks, kRouteThreads, 0, s>>>(
      src, dst, w, n, n_ops, g->nv, P, as<u64>(r.offs), as<RouteTable>(r.table), with_w,
      keep_pos ? as<u64>(r.pos) : nullptr, &mine.hdr->done);
  note_kernel(1);
  RT_CK(cudaGetLastError());
  r.arrive_expected += P;
  if (r.comm->host_ordered()) {
    RT_CM(r.comm->wait_peers(r.ev_done, s));
  } else {
    k_route_wait<<<1, 32, 0, s>>>(&mine.hdr->arrive, r.arrive_expected, g->ctl);
    note_kernel(1);
    RT_CK(cudaGetLastError());
  }
  return DG_OK;
}

// the ops this rank owns for the current batch, wherever the exchange left them
struct Received {
  const u32 *src, *dst, *w;
};

// Steps 3 + 5 by whichever exchange is active (fused, or copy; fused falls back to
// copy when its windows cannot grow).
dg_status route_ops(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n, bool mirror,
                    bool with_w, bool keep_pos, cudaStream_t s, Received* out, bool* via_window) {
  Router& r = *g->router;
  *via_window = false;
  if (r.fused) {
    bool fell_back = false;
    dg_status st = route_fused_scatter(g, src, dst, w, n, mirror, with_w, keep_pos, &fell_back, s);
    if (st != DG_OK) return st;
    if (!fell_back) {
      const WinPtrs x = win_ptrs(r.win, r.wcap);
      *out = Received{x.src, x.dst, x.w};
      *via_window = true;
      return DG_OK;
    }
  }
  dg_status st = route_scatter_copy(g, src, dst, w, n, mirror, with_w, keep_pos, s);
  if (st != DG_OK) return st;
  if ((st = route_exchange(g, with_w, s)) != DG_OK) return st;
  *out = Received{as<u32>(r.rsrc), as<u32>(r.rdst), with_w ? as<u32>(r.rw) : nullptr};
  return DG_OK;
}

dg_status reset_counters(dg_graph g, cudaStream_t s) {
  RT_CK(cudaMemsetAsync(&g->ctl->count, 0, sizeof(u64), s));
  RT_CK(cudaMemsetAsync(&g->ctl->retry_count, 0, sizeof(u32), s));
  return DG_OK;
}

// every rank agreed the batch holds an out-of-range ID: record the rejection on the
// host mirror and the device (read back by dg_batch_status / host-buffer calls)
dg_status mark_rejected(dg_graph g, u32 epoch, cudaStream_t s) {
  g->hctl->fail_epoch = std::max(g->hctl->fail_epoch, epoch);
  g->router->h_scalar[2] = epoch;
  RT_CK(cudaMemcpyAsync(&g->ctl->fail_epoch, g->router->h_scalar + 2, 4, cudaMemcpyHostToDevice, s));
  RT_CK(cudaStreamSynchronize(s));  // h_scalar is reused by the next collective
  return DG_OK;
}

}  // namespace

dg_status router_unique_id(void* out128) { return nccl_unique_id(out128); }

dg_status router_create(dg_graph g, const void* unique_id, Router** out) {
  if (g->nranks > (u32)kMaxRanks) return DG_ERR_UNSUPPORTED;
  Comm* c = nullptr;
  dg_status st = g->cfg.group ? group_comm_create(g->cfg.group, g->nranks, g->rank, g->device, &c)
                              : nccl_comm_create(unique_id, g->nranks, g->rank, &c);
  if (st != DG_OK) return st;
  Router* r = new Router();
  r->comm = c;
  r->P = g->nranks;
  r->rank = g->rank;
  if (cudaMallocHost(&r->h_meta, (size_t)(r->P + 1) * (r->P + 1) * 8) != cudaSuccess ||
      cudaMallocHost(&r->h_scalar, 64) != cudaSuccess ||
      cudaMallocHost(&r->h_table, sizeof(RouteTable)) != cudaSuccess ||
      grow(r->table, sizeof(RouteTable)) != cudaSuccess ||
      cudaEventCreateWithFlags(&r->ev_done, cudaEventDisableTiming) != cudaSuccess) {
    router_destroy(r);
    return DG_ERR_CUDA;
  }
  *out = r;
  return DG_OK;
}

dg_status router_setup_fused(dg_graph g, cudaStream_t s) {
  Router& r = *g->router;
  const char* mode = std::getenv("DG_ROUTER");
  if ((mode && std::strcmp(mode, "nccl") == 0) || (g->cfg.flags & DG_FLAG_COPY_EXCHANGE)) {
    r.copy_only = true;
    return DG_OK;
  }
  // initial window: 2^20 ops (17 MB); grows collectively with the batches
  u64 cap = 1ull << 20;
  if (const char* e = std::getenv("DG_ROUTER_WINDOW_OPS")) cap = std::max<u64>(64, std::strtoull(e, nullptr, 10));
  return window_setup(g, cap, s);
}

bool router_fused(const Router* r) { return r && r->fused; }

void router_destroy(Router* r) {
  if (!r) return;
  if (r->comm) r->comm->unmap_windows(r->peer);
  if (r->win) cudaFree(r->win);
  for (char* p : r->retired) cudaFree(p);
  if (r->h_table) cudaFreeHost(r->h_table);
  if (r->ev_done) cudaEventDestroy(r->ev_done);
  delete r->comm;
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
    if ((st = mark_rejected(g, epoch, s)) != DG_OK) return st;
    return reset_counters(g, s);
  }
  if (st != DG_OK) return st;
  Router& r = *g->router;
  // pool growth for the ops this rank receives happens now, before any rank scatters
  if ((st = prepare_insert(g, r.roff[r.P], s)) != DG_OK) return st;
  if (r.fused) RT_CM(r.comm->quiesce());
  Received rx;
  bool win = false;
  if ((st = route_ops(g, src, dst, w, n, !g->directed, true, false, s, &rx, &win)) != DG_OK)
    return st;
  if ((st = reset_counters(g, s)) != DG_OK) return st;
  return local_insert(g, rx.src, rx.dst, rx.w, r.roff[r.P], false, epoch, s);
}

dg_status router_delete(dg_graph g, const u32* src, const u32* dst, u64 n, u32 epoch,
                        cudaStream_t s) {
  dg_status st = route_partition(g, src, dst, nullptr, n, !g->directed, false, false, s);
  if (st == DG_ERR_VERTEX_OUT_OF_RANGE) {
    if ((st = mark_rejected(g, epoch, s)) != DG_OK) return st;
    return reset_counters(g, s);
  }
  if (st != DG_OK) return st;
  Router& r = *g->router;
  Received rx;
  bool win = false;
  if ((st = route_ops(g, src, dst, nullptr, n, !g->directed, false, false, s, &rx, &win)) != DG_OK)
    return st;
  if ((st = reset_counters(g, s)) != DG_OK) return st;
  return local_delete(g, rx.src, rx.dst, r.roff[r.P], false, epoch, s, false, false);
}

// Out-of-range queries (Q7/Q19) behave as at P = 1: they are not routed and answer 0,
// the in-range queries of the batch are answered, and the batch reports
// DG_ERR_VERTEX_OUT_OF_RANGE (on every rank).
dg_status router_query(dg_graph g, const u32* src, const u32* dst, u64 n, uint8_t* found, u32* wout,
                       u32 epoch, cudaStream_t s) {
  Router& r = *g->router;
  dg_status st = route_partition(g, src, dst, nullptr, n, false, false, true, s);
  if (st == DG_ERR_VERTEX_OUT_OF_RANGE) {
    if ((st = mark_rejected(g, epoch, s)) != DG_OK) return st;
  } else if (st != DG_OK) {
    return st;
  }
  const u64 total = r.roff[r.P];
  if (!r.fused) {  // (fused: sized with the windows, see window_setup)
    RT_CK(grow(r.rfound, total + 1));
    RT_CK(grow(r.rwt, total * 4 + 4));
  }
  Received rx;
  bool win = false;
  if ((st = route_ops(g, src, dst, nullptr, n, false, false, true, s, &rx, &win)) != DG_OK)
    return st;
  if ((st = local_query(g, rx.src, rx.dst, total, as<uint8_t>(r.rfound), as<u32>(r.rwt), epoch,
                        s)) != DG_OK)
    return st;
  const uint8_t* afound = nullptr;
  const u32* awt = nullptr;
  if (win) {
    // answers straight into the askers' answer windows, then wait for ours (a11)
    const WinPtrs x = win_ptrs(r.win, r.wcap);
    k_route_return<<<(unsigned)g->sms * 4, 256, 0, s>>>(as<uint8_t>(r.rfound), as<u32>(r.rwt), r.P,
                                                        as<RouteTable>(r.table), &x.hdr->done_ret);
    note_kernel(1);
    RT_CK(cudaGetLastError());
    r.ans_expected += r.P;
    if (r.comm->host_ordered()) {
      RT_CM(r.comm->wait_peers(r.ev_done, s));
    } else {
      k_route_wait<<<1, 32, 0, s>>>(&x.hdr->ans_arrive, r.ans_expected, g->ctl);
      note_kernel(1);
      RT_CK(cudaGetLastError());
    }
    afound = x.found;
    awt = x.wt;
  } else {
    // answers travel back through the reversed exchange (a11)
    RT_CK(grow(r.rfound, total + 1));  // (a fused batch that fell back)
    RT_CK(grow(r.rwt, total * 4 + 4));
    RT_CK(grow(r.sfound, n + 1));
    RT_CK(grow(r.swt, n * 4 + 4));
    if (r.rcnt[r.rank]) {
      RT_CK(cudaMemcpyAsync(as<uint8_t>(r.sfound) + r.soff[r.rank],
                            as<uint8_t>(r.rfound) + r.roff[r.rank], r.rcnt[r.rank],
                            cudaMemcpyDeviceToDevice, s));
      RT_CK(cudaMemcpyAsync(as<u32>(r.swt) + r.soff[r.rank], as<u32>(r.rwt) + r.roff[r.rank],
                            r.rcnt[r.rank] * 4, cudaMemcpyDeviceToDevice, s));
    }
    RT_CM(r.comm->group_start());
    for (u32 q = 0; q < r.P; ++q) {
      if (q == r.rank) continue;
      if (r.rcnt[q]) {
        RT_CM(r.comm->send(as<uint8_t>(r.rfound) + r.roff[q], r.rcnt[q], q, s));
        RT_CM(r.comm->send(as<u32>(r.rwt) + r.roff[q], r.rcnt[q] * 4, q, s));
      }
      if (r.scnt[q]) {
        RT_CM(r.comm->recv(as<uint8_t>(r.sfound) + r.soff[q], r.scnt[q], q, s));
        RT_CM(r.comm->recv(as<u32>(r.swt) + r.soff[q], r.scnt[q] * 4, q, s));
      }
    }
    RT_CM(r.comm->group_end(s));
    afound = as<uint8_t>(r.sfound);
    awt = as<u32>(r.swt);
  }
  if (n) {
    u64 blocks = std::min<u64>((n + 255) / 256, (u64)g->sms * 8);
    k_route_unpermute<<<(unsigned)blocks, 256, 0, s>>>(as<u64>(r.pos), n, afound, awt, found, wout);
    note_kernel(1);
    RT_CK(cudaGetLastError());
  }
  return DG_OK;
}

dg_status router_allgather_u32(dg_graph g, const u32* ids, u64 n, int slot, const u32** all,
                               u64* all_n, cudaStream_t s) {
  Router& r = *g->router;
  Router::Buf& out = slot ? r.ids2 : r.ids;
  RT_CK(grow(r.scalar, (size_t)(r.P + 1) * 8));
  u64* cnts = as<u64>(r.scalar);
  r.h_scalar[3] = n;
  RT_CK(cudaMemcpyAsync(cnts + r.P, r.h_scalar + 3, 8, cudaMemcpyHostToDevice, s));
  RT_CM(r.comm->allgather(cnts + r.P, cnts, 8, s));
  RT_CK(cudaMemcpyAsync(r.h_meta, cnts, (size_t)r.P * 8, cudaMemcpyDeviceToHost, s));
  RT_CK(cudaStreamSynchronize(s));
  std::vector<u64> off(r.P + 1, 0);
  for (u32 q = 0; q < r.P; ++q) off[q + 1] = off[q] + r.h_meta[q];
  const u64 total = off[r.P];
  RT_CK(grow(out, total * 4 + 4));
  if (n) RT_CK(cudaMemcpyAsync(as<u32>(out) + off[r.rank], ids, n * 4, cudaMemcpyDeviceToDevice, s));
  RT_CM(r.comm->group_start());
  for (u32 q = 0; q < r.P; ++q) {
    if (q == r.rank) continue;
    if (n) RT_CM(r.comm->send(ids, n * 4, q, s));
    if (r.h_meta[q]) RT_CM(r.comm->recv(as<u32>(out) + off[q], r.h_meta[q] * 4, q, s));
  }
  RT_CM(r.comm->group_end(s));
  *all = as<u32>(out);
  *all_n = total;
  return DG_OK;
}

namespace {
dg_status allreduce_u64(dg_graph g, u64* v, bool max, cudaStream_t s) {
  Router& r = *g->router;
  RT_CK(grow(r.scalar, (size_t)(r.P + 1) * 8));
  u64* d = as<u64>(r.scalar);
  r.h_scalar[0] = *v;
  RT_CK(cudaMemcpyAsync(d, r.h_scalar, 8, cudaMemcpyHostToDevice, s));
  RT_CM(r.comm->allreduce_u64(d, max, s));
  RT_CK(cudaMemcpyAsync(r.h_scalar, d, 8, cudaMemcpyDeviceToHost, s));
  RT_CK(cudaStreamSynchronize(s));
  *v = r.h_scalar[0];
  return DG_OK;
}
}  // namespace

dg_status router_sum_u64(dg_graph g, u64* v, cudaStream_t s) { return allreduce_u64(g, v, false, s); }
dg_status router_max_u64(dg_graph g, u64* v, cudaStream_t s) { return allreduce_u64(g, v, true, s); }

}  // namespace dg
