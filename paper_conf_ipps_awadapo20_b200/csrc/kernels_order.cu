// kernels_order.cu — locality order of a large batch before its probe kernel.
//
// The paper processes a batch in the order it is given (one warp per op)
// and groups same-source ops only inside a warp.  On a B200 the probe
// kernels are bound by random DRAM requests: a uniform batch touches
// each row's buckets ~3.5 times per 2^24 ops, spread over the whole launch, so the
// 126 MB L2 cannot keep a bucket between its touches (the tables are 5x larger).
// Partitioning the batch by row >> shift (a counting sort on the high row bits, not
// a sort: ops keep no particular order inside a partition) makes the ops in flight at
// any moment cover a window of rows whose buckets fit in L2, so repeated touches of a
// bucket hit L2 and consecutive DRAM requests fall into nearby pages.  Measured on
// cfg2 2^24 batches (tools/locality_probe.py, the reorder itself untimed): delete
// 0.80 -> 0.54 ms, query 0.62 -> 0.49 ms.  Deletes use it (order-independent: each
// key is removed once, the count is of keys that existed, Q5), and inserts with at
// most ~1 op per row (cfg3: 1.50 -> 0.95 ms; with more ops per row they gain nothing:
// ops of one row then race for the same free slot); the weights move with their ops.
// Queries lose more than they gain (answers written back to the caller's positions
// scatter 1- and 4-B stores: 7x the DRAM write bytes; measured 0.64 -> 0.78 ms for
// the probe alone).
//
// The batch is split into one contiguous range per block (B = 4 per SM):
//   k_order_count   : block b's shared histogram of its range -> h[b][p], totals[p]
//   k_order_scan    : one block per partition p: h[b][p] -> the first output slot of
//                     (b, p) = sum of totals[q < p] + sum of h[b' < b][p]
//   k_order_scatter : block b re-reads its range; a shared-memory cursor per partition
//                     places each op (the order inside a (b, p) run is arbitrary)
// No global atomics on the partition cursors (a per-tile reservation scheme measured
// 0.24 ms per 2^24 ops on 148 cursor addresses).  Measured on cfg2 2^24 deletes:
// count 31 us, scan 7 us, scatter 120 us (reads 183 MB: partial output sectors are
// re-read on eviction; L2 evict-first loads / evict-last stores did not change it),
// delete probe 0.80 -> 0.54 ms.
// Undirected batches (mirror = true) expand op j >= n to (dst[j-n], src[j-n]) here,
// so the probe sees explicit directed ops.
#include <functional>

#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

namespace {

constexpr int kOrdThreads = 256;
#ifndef DG_ORDER_ITEMS
#define DG_ORDER_ITEMS 8
#endif
constexpr int kOrdItems = DG_ORDER_ITEMS;  // ops per thread per step (all loads issued first)
constexpr u32 kOrdStep = kOrdThreads * kOrdItems;
// (measured, cfg2 2^24 delete: 4 / 6 / 8 blocks -> scatter 71 / 75 / 90 us: more
// block ranges leave more partial runs)
#ifndef DG_ORDER_BLOCKS
#define DG_ORDER_BLOCKS 4
#endif
constexpr int kOrdBlocksPerSm = DG_ORDER_BLOCKS;  // resident blocks of 256 threads per SM
constexpr u32 kOrdMaxBlocks = 2048;  // k_order_scan: one column per block, 2 per thread

__device__ __forceinline__ void op_of(const u32* src, const u32* dst, u64 n, u64 j, u32& u, u32& v) {
  if (j < n) { u = src[j]; v = dst[j]; }
  else { u = dst[j - n]; v = src[j - n]; }  // undirected mirror op
}

__device__ __forceinline__ u32 part_of(u32 u, u32 nranks, u32 shift, u32 nparts) {
  const u32 row = nranks == 1 ? u : u / nranks;
  const u32 p = row >> shift;
  return p < nparts ? p : nparts - 1;  // (out-of-range IDs: the batch is rejected anyway)
}

__device__ __forceinline__ void range_of(u64 n_ops, u64& lo, u64& hi) {
  const u64 chunk = ((n_ops + gridDim.x - 1) / gridDim.x + 3) & ~3ull;  // (quads stay aligned)
  lo = (u64)blockIdx.x * chunk;
  if (lo > n_ops) lo = n_ops;
  hi = lo + chunk < n_ops ? lo + chunk : n_ops;
}

// The ops of one step (kOrdItems per thread, all loads issued before any is used):
// VEC (16-B aligned arrays, n % 4 == 0 for mirrors): two 16-B loads per array and
// thread, ops j0 + 4 (k kOrdThreads + t) + i; else one 4-B load per op, ops
// j0 + k kOrdThreads + t.  Bit k of `valid` marks item k as an op of [j0, hi).
// need_v: also load v (validation reads both endpoints; mirrors are validated at
// their original op, so their v is not needed then).
template <bool VEC>
__device__ __forceinline__ u32 load_step(const u32* __restrict__ src, const u32* __restrict__ dst,
                                         u64 n, u64 j0, u64 hi, bool need_v,
                                         u32 (&us)[kOrdItems], u32 (&vs)[kOrdItems]) {
  u32 valid = 0;
  if constexpr (VEC) {
#pragma unroll
    for (int k = 0; k < kOrdItems / 4; ++k) {
      const u64 j = j0 + 4 * ((u64)k * kOrdThreads + threadIdx.x);
      if (j + 3 < hi) {
        const bool m = j >= n;  // (n % 4 == 0: a quad never straddles n)
        const u64 jj = m ? j - n : j;
        const uint4 a = *reinterpret_cast<const uint4*>((m ? dst : src) + jj);
        us[4 * k] = a.x; us[4 * k + 1] = a.y; us[4 * k + 2] = a.z; us[4 * k + 3] = a.w;
        if (need_v || m) {
          const uint4 b = *reinterpret_cast<const uint4*>((m ? src : dst) + jj);
          vs[4 * k] = b.x; vs[4 * k + 1] = b.y; vs[4 * k + 2] = b.z; vs[4 * k + 3] = b.w;
        } else {
          vs[4 * k] = vs[4 * k + 1] = vs[4 * k + 2] = vs[4 * k + 3] = 0u;
        }
        valid |= 0xFu << (4 * k);
      } else {
#pragma unroll
        for (int i = 0; i < 4; ++i) {
          us[4 * k + i] = vs[4 * k + i] = 0u;
          if (j + i < hi) {
            op_of(src, dst, n, j + i, us[4 * k + i], vs[4 * k + i]);
            valid |= 1u << (4 * k + i);
          }
        }
      }
    }
  } else {
#pragma unroll
    for (int k = 0; k < kOrdItems; ++k) {
      const u64 j = j0 + (u64)k * kOrdThreads + threadIdx.x;
      us[k] = vs[k] = 0u;
      if (j < hi) {
        op_of(src, dst, n, j, us[k], vs[k]);
        valid |= 1u << k;
      }
    }
  }
  return valid;
}

// The weights of one step's ops, in load_step's order (mirror op j >= n: w[j - n]).
template <bool VEC>
__device__ __forceinline__ void load_w_step(const u32* __restrict__ w, u64 n, u64 j0, u64 hi,
                                            u32 (&ws)[kOrdItems]) {
  if constexpr (VEC) {
#pragma unroll
    for (int k = 0; k < kOrdItems / 4; ++k) {
      const u64 j = j0 + 4 * ((u64)k * kOrdThreads + threadIdx.x);
      if (j + 3 < hi) {
        const uint4 a = *reinterpret_cast<const uint4*>(w + (j >= n ? j - n : j));
        ws[4 * k] = a.x; ws[4 * k + 1] = a.y; ws[4 * k + 2] = a.z; ws[4 * k + 3] = a.w;
      } else {
#pragma unroll
        for (int i = 0; i < 4; ++i)
          ws[4 * k + i] = j + i < hi ? w[j + i >= n ? j + i - n : j + i] : 0u;
      }
    }
  } else {
#pragma unroll
    for (int k = 0; k < kOrdItems; ++k) {
      const u64 j = j0 + (u64)k * kOrdThreads + threadIdx.x;
      ws[k] = j < hi ? w[j >= n ? j - n : j] : 0u;
    }
  }
}

// ctl != nullptr: also the batch validation of k_validate (Q7: an endpoint >= nv
// rejects the batch; the per-batch counters are reset), so a validated delete reads
// its inputs once before the scatter instead of twice.
template <bool VEC>
__global__ void __launch_bounds__(kOrdThreads, kOrdBlocksPerSm) k_order_count(const u32* __restrict__ src,
                                                             const u32* __restrict__ dst, u64 n,
                                                             u64 n_ops, u32 nranks, u32 shift,
                                                             u32 nparts, u32* h, u32* totals,
                                                             u64 nv, u32 epoch, DevCtl* ctl) {
  __shared__ u32 hs[kMaxOrderParts];
  for (u32 p = threadIdx.x; p < nparts; p += blockDim.x) hs[p] = 0;
  if (ctl && blockIdx.x == 0 && threadIdx.x == 0) {
    ctl->count = 0;
    ctl->retry_count = 0;
  }
  __syncthreads();
  u64 lo, hi;
  range_of(n_ops, lo, hi);
  bool bad = false;
  // the next step's loads are issued before the current step is counted
  u32 us[kOrdItems], vs[kOrdItems];
  u32 valid = lo < hi ? load_step<VEC>(src, dst, n, lo, hi, ctl != nullptr, us, vs) : 0u;
  for (u64 j0 = lo; j0 < hi; j0 += kOrdStep) {
    u32 nus[kOrdItems], nvs[kOrdItems];
    const u32 nvalid =
        j0 + kOrdStep < hi ? load_step<VEC>(src, dst, n, j0 + kOrdStep, hi, ctl != nullptr, nus, nvs) : 0u;
#pragma unroll
    for (int k = 0; k < kOrdItems; ++k)
      if ((valid >> k) & 1u) {
        bad |= ((u64)us[k] >= nv) | ((u64)vs[k] >= nv);
        atomicAdd(&hs[part_of(us[k], nranks, shift, nparts)], 1u);
      }
#pragma unroll
    for (int k = 0; k < kOrdItems; ++k) { us[k] = nus[k]; vs[k] = nvs[k]; }
    valid = nvalid;
  }
  if (ctl && __any_sync(0xFFFFFFFFu, bad) && (threadIdx.x & 31) == 0)
    atomicMax(&ctl->fail_epoch, epoch);
  __syncthreads();
  for (u32 p = threadIdx.x; p < nparts; p += blockDim.x) {
    h[(size_t)blockIdx.x * kMaxOrderParts + p] = hs[p];
    if (hs[p]) atomicAdd(&totals[p], hs[p]);
  }
}

// one block per partition p, 1024 threads, count blocks 2t and 2t+1 per thread
__global__ void __launch_bounds__(1024) k_order_scan(u32* h, const u32* totals, u32 nb) {
  __shared__ u32 s[1024];
  __shared__ u32 base;
  const u32 p = blockIdx.x, t = threadIdx.x;
  if (t < 32) {  // first slot of partition p = sum of the totals before it
    u32 x = 0;
    for (u32 q = t; q < p; q += 32) x += totals[q];
    x = __reduce_add_sync(0xFFFFFFFFu, x);
    if (t == 0) base = x;
  }
  const u32 b0 = 2 * t, b1 = 2 * t + 1;
  const u32 o0 = b0 < nb ? h[(size_t)b0 * kMaxOrderParts + p] : 0u;
  const u32 o1 = b1 < nb ? h[(size_t)b1 * kMaxOrderParts + p] : 0u;
  s[t] = o0 + o1;
  __syncthreads();
  for (u32 off = 1; off < 1024; off <<= 1) {  // inclusive scan over the block pairs
    const u32 x = t >= off ? s[t - off] : 0u;
    __syncthreads();
    s[t] += x;
    __syncthreads();
  }
  const u32 ex = base + s[t] - o0 - o1;
  if (b0 < nb) h[(size_t)b0 * kMaxOrderParts + p] = ex;
  if (b1 < nb) h[(size_t)b1 * kMaxOrderParts + p] = ex + o0;
}

// Per step of 2048 ops the block first sorts the ops by partition in shared memory
// (rank by shared atomics, offsets by a block scan over the partitions), then writes
// them out in that order, so consecutive threads store consecutive slots of one
// partition's run (scattering op by op made every warp store touch 32 sectors:
// 0.31 ms per 2^24 ops).
// WT: the batch carries weights (an insert batch), moved with their ops.
template <bool VEC, bool WT>
__global__ void __launch_bounds__(kOrdThreads, kOrdBlocksPerSm) k_order_scatter(
    const u32* __restrict__ src, const u32* __restrict__ dst, const u32* __restrict__ w, u64 n,
    u64 n_ops, u32 nranks, u32 shift, u32 nparts, const u32* __restrict__ h,
    u32* __restrict__ osrc, u32* __restrict__ odst, u32* __restrict__ ow) {
  __shared__ u32 cur[kMaxOrderParts];   // next output slot of each partition
  __shared__ u32 cnt[kMaxOrderParts];   // this step: ops per partition, then their offsets
  __shared__ u32 st_u[kOrdStep], st_v[kOrdStep];
  __shared__ u32 st_w[WT ? kOrdStep : 1];
  __shared__ uint8_t st_p[kOrdStep];
  __shared__ u32 wsum[kOrdThreads / 32];
  static_assert(kMaxOrderParts == kOrdThreads, "one partition per thread in the scan");
  const u32 t = threadIdx.x, lane = t & 31u, wid = t >> 5;
  cur[t] = t < nparts ? h[(size_t)blockIdx.x * kMaxOrderParts + t] : 0u;
  u64 lo, hi;
  range_of(n_ops, lo, hi);
  // software pipeline: the next step's loads are issued once the current step's ops
  // are staged in shared memory, so they are in flight during its stores
  u32 us[kOrdItems], vs[kOrdItems], ws[kOrdItems];
  u32 valid = lo < hi ? load_step<VEC>(src, dst, n, lo, hi, true, us, vs) : 0u;
  if (WT && lo < hi) load_w_step<VEC>(w, n, lo, hi, ws);
  for (u64 j0 = lo; j0 < hi; j0 += kOrdStep) {
    cnt[t] = 0;
    __syncthreads();
    u32 ps[kOrdItems], rk[kOrdItems];
#pragma unroll
    for (int k = 0; k < kOrdItems; ++k) {
      const bool in = (valid >> k) & 1u;
      ps[k] = in ? part_of(us[k], nranks, shift, nparts) : kNil;
      rk[k] = in ? atomicAdd(&cnt[ps[k]], 1u) : 0u;
    }
    __syncthreads();
    // exclusive scan of cnt over the partitions (thread t holds partition t)
    const u32 c = cnt[t];
    u32 x = c;
#pragma unroll
    for (u32 o = 1; o < 32; o <<= 1) {
      const u32 y = __shfl_up_sync(0xFFFFFFFFu, x, o);
      if (lane >= o) x += y;
    }
    if (lane == 31) wsum[wid] = x;
    __syncthreads();
    u32 wbase = 0;
#pragma unroll
    for (u32 w = 0; w < kOrdThreads / 32; ++w) wbase += w < wid ? wsum[w] : 0u;
    const u32 off = wbase + x - c;  // first staging slot of partition t in this step
    __syncthreads();
    cnt[t] = off;
    __syncthreads();
#pragma unroll
    for (int k = 0; k < kOrdItems; ++k) {
      if (ps[k] == kNil) continue;
      const u32 at = cnt[ps[k]] + rk[k];
      st_u[at] = us[k];
      st_v[at] = vs[k];
      if (WT) st_w[at] = ws[k];
      st_p[at] = (uint8_t)ps[k];
    }
    valid = j0 + kOrdStep < hi ? load_step<VEC>(src, dst, n, j0 + kOrdStep, hi, true, us, vs) : 0u;
    if (WT && j0 + kOrdStep < hi) load_w_step<VEC>(w, n, j0 + kOrdStep, hi, ws);
    __syncthreads();
    const u32 m = (u32)(hi - j0 < kOrdStep ? hi - j0 : kOrdStep);
    for (u32 i = t; i < m; i += kOrdThreads) {  // runs of one partition are contiguous
      const u32 p = st_p[i];
      const u32 at = cur[p] + (i - cnt[p]);
      osrc[at] = st_u[i];
      odst[at] = st_v[i];
      if (WT) ow[at] = st_w[i];
    }
    __syncthreads();
    if (t < nparts) cur[t] += c;
  }
}

int order_blocks(int sms) {
  const int b = sms * kOrdBlocksPerSm;
  return b < (int)kOrdMaxBlocks ? b : (int)kOrdMaxBlocks;
}

}  // namespace

u32 order_shift(u64 rows) {
  u32 bits = 0;
  while (bits < 32 && (1ull << bits) < rows) ++bits;
  return bits > kOrderPartBits ? bits - kOrderPartBits : 0u;
}

size_t order_scratch_bytes(int sms) {
  return ((size_t)order_blocks(sms) + 1) * kMaxOrderParts * 4;
}

// scratch: order_scratch_bytes(sms) bytes; n_ops = (mirror ? 2n : n) < 2^32.
// ctl != nullptr: the count pass validates the batch (k_validate's job); `between`,
// when set, runs on the stream after that pass and before the scatter (the caller's
// snapshot of the verdict).
// w / ow (nullable): the batch's weights and their permuted copy (insert batches)
cudaError_t launch_order(const u32* src, const u32* dst, const u32* w, u64 n, bool mirror, u64 rows,
                         u32 nranks, void* scratch, u32* osrc, u32* odst, u32* ow, u64 nv,
                         u32 epoch, DevCtl* ctl, const std::function<cudaError_t()>& between,
                         int sms, cudaStream_t s) {
  const u64 n_ops = mirror ? 2 * n : n;
  const u32 shift = order_shift(rows);
  u32 nparts = (u32)(((rows ? rows : 1) + (1ull << shift) - 1) >> shift);
  if (nparts > kMaxOrderParts) nparts = kMaxOrderParts;
  if (nparts == 0) nparts = 1;
  const int nb = order_blocks(sms);
  u32* h = static_cast<u32*>(scratch);
  u32* totals = h + (size_t)nb * kMaxOrderParts;
  cudaError_t e = cudaMemsetAsync(totals, 0, kMaxOrderParts * 4, s);
  if (e != cudaSuccess) return e;
  const bool vec = ((reinterpret_cast<uintptr_t>(src) | reinterpret_cast<uintptr_t>(dst) |
                     reinterpret_cast<uintptr_t>(w)) & 15) == 0 &&
                   (!mirror || n % 4 == 0);
  if (vec)
    k_order_count<true><<<nb, kOrdThreads, 0, s>>>(src, dst, n, n_ops, nranks, shift, nparts, h,
                                                   totals, nv, epoch, ctl);
  else
    k_order_count<false><<<nb, kOrdThreads, 0, s>>>(src, dst, n, n_ops, nranks, shift, nparts, h,
                                                    totals, nv, epoch, ctl);
  if (between && (e = between()) != cudaSuccess) return e;
  k_order_scan<<<nparts, 1024, 0, s>>>(h, totals, (u32)nb);
#define DG_SCATTER(V_, W_)                                                                   \
  k_order_scatter<V_, W_><<<nb, kOrdThreads, 0, s>>>(src, dst, w, n, n_ops, nranks, shift, nparts, \
                                                     h, osrc, odst, ow)
  if (w) {
    if (vec) DG_SCATTER(true, true); else DG_SCATTER(false, true);
  } else {
    if (vec) DG_SCATTER(true, false); else DG_SCATTER(false, false);
  }
#undef DG_SCATTER
  note_kernel(3);
  return cudaGetLastError();
}

}  // namespace dg
