// kernels_graph.cu — table construction, export, statistics and vertex deletion.
#include <cub/device/device_scan.cuh>
#include <thrust/iterator/counting_iterator.h>
#include <thrust/iterator/transform_iterator.h>

#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

// ------------------------------------------------------ initial buckets (a0) ----
// #buckets of a new table = ceil(|A_u| / (lf * Bc)), one bucket when |A_u| is
// unknown.  lf is carried in thousandths so the
// ceiling is an exact integer decision (reading R-LF).
__global__ void k_initial_buckets(u64* nb, u64 count, u64 row0, const u32* hints_global,
                                  const u32* hints_local, u32 nranks, u32 rank, u32 lf_milli,
                                  u32 bc, u32 adaptive, u32 set) {
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 r = (u64)blockIdx.x * blockDim.x + threadIdx.x; r <= count; r += stride) {
    if (r == count) {
      nb[r] = 0;
      continue;
    }
    u64 hint = 0;
    if (hints_global) hint = hints_global[(row0 + r) * nranks + rank];
    else if (hints_local) hint = hints_local[r];
    if (adaptive) {
      nb[r] = class_size(hint, lf_milli, set);
      continue;
    }
    const u64 den = (u64)lf_milli * bc;
    u64 b = hint ? (hint * 1000 + den - 1) / den : 1;
    nb[r] = b ? b : 1;
  }
}

cudaError_t launch_initial_buckets(u64* nb, u64 count, u64 row0, const u32* hints_global,
                                   const u32* hints_local, u32 nranks, u32 rank, u32 lf_milli,
                                   u32 bc, u32 adaptive, u32 set, cudaStream_t s) {
  u64 blocks = (count + 1 + 255) / 256;
  if (blocks > 65535) blocks = 65535;
  k_initial_buckets<<<(unsigned)blocks, 256, 0, s>>>(nb, count, row0, hints_global, hints_local,
                                                     nranks, rank, lf_milli, bc, adaptive, set);
  note_kernel(1);
  return cudaGetLastError();
}

cudaError_t scan_exclusive_u64(const u64* in, u64* out, u64 count, void** temp,
                               size_t* temp_bytes, cudaStream_t s) {
  size_t need = 0;
  cudaError_t e = cub::DeviceScan::ExclusiveSum(nullptr, need, in, out, (int64_t)count, s);
  if (e != cudaSuccess) return e;
  if (need > *temp_bytes) {
    if (*temp) cudaFree(*temp);
    *temp = nullptr;
    *temp_bytes = 0;
    e = cudaMalloc(temp, need);
    if (e != cudaSuccess) return e;
    *temp_bytes = need;
  }
  note_kernel(2);
  return cub::DeviceScan::ExclusiveSum(*temp, need, in, out, (int64_t)count, s);
}

// buckets of class c in a packed (#buckets | class << 40) entry
// (home: uniform layouts keep chain 0 in the row's home bucket, so a row takes
// #buckets - 1 buckets from the pool)
struct ClassCount {
  const u64* nbc;
  u64 n;
  u32 c;
  u32 home;
  __host__ __device__ u64 operator()(u64 i) const {
    if (i >= n) return 0ull;
    const u64 v = nbc[i];
    return (u32)(v >> 40) == c ? (v & kNbMask) - home : 0ull;
  }
};

cudaError_t scan_class_offsets(const u64* nbc, u64 count, u32 c, u32 home, u64* off, void** temp,
                               size_t* temp_bytes, cudaStream_t s) {
  auto it = thrust::make_transform_iterator(thrust::counting_iterator<u64>(0),
                                            ClassCount{nbc, count, c, home});
  size_t need = 0;
  cudaError_t e = cub::DeviceScan::ExclusiveSum(nullptr, need, it, off, (int64_t)(count + 1), s);
  if (e != cudaSuccess) return e;
  if (need > *temp_bytes) {
    if (*temp) cudaFree(*temp);
    *temp = nullptr;
    *temp_bytes = 0;
    e = cudaMalloc(temp, need);
    if (e != cudaSuccess) return e;
    *temp_bytes = need;
  }
  note_kernel(2);
  return cub::DeviceScan::ExclusiveSum(*temp, need, it, off, (int64_t)(count + 1), s);
}

// Row r gets nbc[r] consecutive base buckets of its class c, starting at
// cb.base0[c] + cb.off[c][r]; each base bucket records its owner row.  `rows`
// (nullable) maps r to a directory row (re-sizing), else row = row0 + r.
// Uniform layouts (t.home set): chain 0 lives in the row's home bucket (all slots
// EMPTY, next NIL, owner = row), the other nb - 1 base buckets are consecutive from
// xbase in the pool, and the probe's chain-count byte nbs[row] = min(nb, 255).
__global__ void k_init_rows(Tables t, u64 row0, u64 count, const u32* rows, const u64* nbc,
                            ClassBases cb) {
  const u64 stride = (u64)gridDim.x * blockDim.x;
  const u32 home = t.home ? 1u : 0u;
  for (u64 r = (u64)blockIdx.x * blockDim.x + threadIdx.x; r < count; r += stride) {
    const u64 v = nbc[r];
    const u32 c = (u32)(v >> 40);
    const u32 n = (u32)(v & kNbMask);
    const u32 idx = by_class(cb.base0, c) + (u32)by_class(cb.off, c)[r];
    const u32 row = rows ? rows[r] : (u32)(row0 + r);
    DirEntry e;
    e.base = (c << kClassShift) | idx;
    e.nb = n;
    t.dir[row] = e;
    *deg_at(t, row) = 0;
    const u32 wc = by_class(cb.words, c);
    u32* pool = by_class(t.pool, c);
    for (u32 k = 0; k + home < n; ++k) pool[(u64)(idx + k) * wc + wc - 1] = row;
    if (home) {
      uint4* hb = reinterpret_cast<uint4*>(t.home + (u64)row * wc);
      const uint4 empty4 = make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
      for (u32 uu = 0; uu + 1 < wc / 4; ++uu) hb[uu] = empty4;
      hb[wc / 4 - 1] = make_uint4(kEmpty, kEmpty, kNil, 0u);  // (degree 0)
      t.nbs[row] = (uint8_t)(n < 255u ? n : 255u);
    }
    if (rows && t.hot_flags) atomicAnd(&t.hot_flags[row >> 5], ~(1u << (row & 31)));
  }
}

cudaError_t launch_init_rows(const Tables& t, u64 row0, u64 count, const u32* rows,
                             const u64* nbc, const ClassBases& cb, cudaStream_t s) {
  if (count == 0) return cudaSuccess;
  u64 blocks = (count + 255) / 256;
  if (blocks > 65535) blocks = 65535;
  k_init_rows<<<(unsigned)blocks, 256, 0, s>>>(t, row0, count, rows, nbc, cb);
  note_kernel(1);
  return cudaGetLastError();
}

// ---------------------------------------------------------- vertex insertion ----
__global__ void k_scatter_hints(u32* hint_new, u64 row0, u64 count, const u32* ids,
                                const u32* hints, u64 n, u32 nranks, u32 rank) {
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 i = (u64)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
    const u32 id = ids[i];
    if (id % nranks != rank) continue;
    const u64 row = id / nranks;
    if (row >= row0 && row < row0 + count) atomicMax(&hint_new[row - row0], hints ? hints[i] : 0u);
  }
}

cudaError_t launch_scatter_hints(u32* hint_new, u64 row0, u64 count, const u32* ids,
                                 const u32* hints, u64 n, u32 nranks, u32 rank, cudaStream_t s) {
  if (n == 0) return cudaSuccess;
  u64 blocks = (n + 255) / 256;
  if (blocks > 65535) blocks = 65535;
  k_scatter_hints<<<(unsigned)blocks, 256, 0, s>>>(hint_new, row0, count, ids, hints, n, nranks,
                                                   rank); note_kernel(1);
  return cudaGetLastError();
}

__global__ void k_max_id(const u32* ids, u64 n, u32* out) {
  u32 m = 0;
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 i = (u64)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) m = max(m, ids[i]);
  m = __reduce_max_sync(0xFFFFFFFFu, m);
  if ((threadIdx.x & 31) == 0) atomicMax(out, m);
}

cudaError_t launch_max_id(const u32* ids, u64 n, u32* out, cudaStream_t s) {
  cudaError_t e = cudaMemsetAsync(out, 0, sizeof(u32), s);
  if (e != cudaSuccess || n == 0) return e;
  u64 blocks = (n + 255) / 256;
  if (blocks > 1024) blocks = 1024;
  k_max_id<<<(unsigned)blocks, 256, 0, s>>>(ids, n, out); note_kernel(1);
  return cudaGetLastError();
}

// ------------------------------------------------------------------ degrees ----
// (uniform layouts: the last word of every home bucket, one 32-B sector per row)
__global__ void k_degrees(Tables t, u32* out) {
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 r = (u64)blockIdx.x * blockDim.x + threadIdx.x; r < t.rows; r += stride)
    out[r] = *deg_at(t, r);
}

cudaError_t launch_degrees(const Tables& t, u32* out, cudaStream_t s) {
  if (t.rows == 0) return cudaSuccess;
  u64 blocks = (t.rows + 255) / 256;
  if (blocks > 65535) blocks = 65535;
  k_degrees<<<(unsigned)blocks, 256, 0, s>>>(t, out); note_kernel(1);
  return cudaGetLastError();
}

// ------------------------------------------------------------ export (a12) ----
struct DegAt {
  const u32* deg;   // adaptive layout
  const u32* home;  // uniform layouts: degree = word hw-1 of home bucket i
  u32 hw;
  u64 rows;
  __host__ __device__ u64 operator()(u64 i) const {
    if (i >= rows) return 0ull;
    return hw ? (u64)home[i * hw + hw - 1] : (u64)deg[i];
  }
};

cudaError_t launch_export_offsets(const Tables& t, u64* ro, void** temp, size_t* temp_bytes,
                                  cudaStream_t s) {
  auto it = thrust::make_transform_iterator(thrust::counting_iterator<u64>(0), DegAt{t.deg, t.home, t.hw, t.rows});
  size_t need = 0;
  cudaError_t e = cub::DeviceScan::ExclusiveSum(nullptr, need, it, ro, (int64_t)(t.rows + 1), s);
  if (e != cudaSuccess) return e;
  if (need > *temp_bytes) {
    if (*temp) cudaFree(*temp);
    *temp = nullptr;
    *temp_bytes = 0;
    e = cudaMalloc(temp, need);
    if (e != cudaSuccess) return e;
    *temp_bytes = need;
  }
  note_kernel(2);
  return cub::DeviceScan::ExclusiveSum(*temp, need, it, ro, (int64_t)(t.rows + 1), s);
}

// One group per row walks every bucket chain of the row (the adjacency iterator,
// P:L431-436) and writes the live pairs compactly at row_offsets[row] (the set
// variant stores no weights: w gets 0).  Rows with more than kBigRowBuckets base
// buckets (hubs) are listed in big[1..] (count in big[0]) and exported by
// k_export_big, one block per row, so one group never walks a hub's thousands of
// buckets alone.  The order of a row's entries is unspecified.
template <int G, int S, bool A>
__device__ __forceinline__ u32 export_bucket(const Group<G>& g, const Geo<G, S, A>& gb,
                                             const uint4& q, u32* dst, u32* w, u64 pos) {
  typedef Lay<G, S> LY;
  const u32 below = (1u << g.gl) - 1u;
  u32 before = 0, total = 0;
#pragma unroll
  for (int j = 0; j < LY::SPU; ++j) {
    const u32 m = g.ballot(gb.has(g.gl, j) && LY::key(q, j) < kTomb);
    before += __popc(m & below);
    total += __popc(m);
  }
  u64 at = pos + before;
#pragma unroll
  for (int j = 0; j < LY::SPU; ++j) {
    if (gb.has(g.gl, j) && LY::key(q, j) < kTomb) {
      dst[at] = LY::key(q, j);
      if (w) w[at] = LY::val(q, j);
      ++at;
    }
  }
  return total;
}

// load lane gl's 16-B unit of bucket gb (lanes past a smaller adaptive bucket get EMPTY)
template <int G, int S, bool A>
__device__ __forceinline__ uint4 ld_unit(const Geo<G, S, A>& gb, u32 gl) {
  if (A && gl >= gb.units) return make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
  return ld_nc_v4(gb.p + 4 * gl);
}

template <int G, int S, bool A>
__global__ void __launch_bounds__(256) k_export_fill(Tables t, const u64* ro, u32* dst, u32* w,
                                                     u32* big) {
  const Group<G> g;
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  for (u64 row = gid; row < t.rows; row += ng) {
    const DirEntry de = t.dir[row];
    if (de.nb > kBigRowBuckets) {
      if (g.gl == 0) big[1 + atomicAdd(big, 1u)] = (u32)row;
      continue;
    }
    u64 pos = ro[row];
    for (u32 k = 0; k < de.nb; ++k) {
      u32 b = chain_head<A>(de.base, (u32)row, k);
      while (b != kNil) {
        const Geo<G, S, A> gb(t, b);
        const uint4 q = ld_unit(gb, g.gl);
        pos += export_bucket(g, gb, q, dst, w, pos);
        b = g.shfl(q.z, gb.units - 1);
      }
    }
  }
}

template <int G, int S, bool A>
__global__ void __launch_bounds__(256) k_export_big(Tables t, const u64* ro, u32* dst, u32* w,
                                                    const u32* big) {
  __shared__ unsigned long long cursor;
  const Group<G> g;
  const u32 gib = threadIdx.x / G, ngb = blockDim.x / G;
  const u32 nbig = big[0];
  for (u32 i = blockIdx.x; i < nbig; i += gridDim.x) {
    const u32 row = big[1 + i];
    const DirEntry de = t.dir[row];
    __syncthreads();
    if (threadIdx.x == 0) cursor = ro[row];
    __syncthreads();
    for (u32 k = gib; k < de.nb; k += ngb) {
      u32 b = chain_head<A>(de.base, row, k);
      while (b != kNil) {
        const Geo<G, S, A> gb(t, b);
        const uint4 q = ld_unit(gb, g.gl);
        u32 cnt = 0;
#pragma unroll
        for (int j = 0; j < Lay<G, S>::SPU; ++j)
          cnt += __popc(g.ballot(gb.has(g.gl, j) && Lay<G, S>::key(q, j) < kTomb));
        unsigned long long pos = 0;
        if (g.gl == 0 && cnt) pos = atomicAdd(&cursor, (unsigned long long)cnt);
        export_bucket(g, gb, q, dst, w, g.shfl(pos, 0));
        b = g.shfl(q.z, gb.units - 1);
      }
    }
  }
}

cudaError_t launch_export_fill(int lay, const Tables& t, const u64* ro, u32* dst, u32* w, u32* big,
                               int sms, cudaStream_t s) {
  if (t.rows == 0) return cudaSuccess;
  const int G = lay & 31;
  u64 blocks = (t.rows * G + 255) / 256;
  if (blocks > (u64)sms * 8) blocks = (u64)sms * 8;
  cudaError_t e = cudaMemsetAsync(big, 0, 4, s);
  if (e != cudaSuccess) return e;
  switch (lay) {
#define DG_CASE(G_, S_, A_)                                                               \
  case DG_LAYA(G_, S_, A_):                                                               \
    k_export_fill<G_, S_, A_><<<(unsigned)blocks, 256, 0, s>>>(t, ro, dst, w, big);       \
    k_export_big<G_, S_, A_><<<(unsigned)sms * 2, 256, 0, s>>>(t, ro, dst, w, big);       \
    break;
    DG_FOR_LAYOUTS_A(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(2);
  return cudaGetLastError();
}

// --------------------------------------------------------------- statistics ----
// one base-bucket chain: live / tombstone slots and its length
// per-thread accumulators of k_stats / k_stats_big
struct StatsAcc {
  unsigned long long linked = 0, live = 0, tombs = 0, maxc = 0, slots = 0, bytes = 0;
};

template <int G, int S, bool A>
__device__ __forceinline__ void stats_chain(const Tables& t, const Group<G>& g, u32 b,
                                            StatsAcc& a) {
  typedef Lay<G, S> LY;
  unsigned long long len = 0;
  while (b != kNil) {
    const Geo<G, S, A> gb(t, b);
    const uint4 q = ld_unit(gb, g.gl);
#pragma unroll
    for (int j = 0; j < LY::SPU; ++j) {
      const bool h = gb.has(g.gl, j);
      a.live += __popc(g.ballot(h && LY::key(q, j) < kTomb));
      a.tombs += __popc(g.ballot(h && LY::key(q, j) == kTomb));
    }
    ++len;
    a.slots += gb.bc();
    a.bytes += 16 * gb.units;
    b = g.shfl(q.z, gb.units - 1);
  }
  a.linked += len;
  if (len > a.maxc) a.maxc = len;
}

__device__ __forceinline__ void stats_flush(StatsOut* out, const StatsAcc& a) {
  if (a.linked | a.live | a.tombs) {
    atomicAdd(&out->linked_buckets, a.linked);
    atomicAdd(&out->live, a.live);
    atomicAdd(&out->tombs, a.tombs);
    atomicAdd(&out->slots, a.slots);
    atomicAdd(&out->bytes, a.bytes);
    atomicMax(&out->max_chain, a.maxc);
  }
}

// group per row; hub rows (> kBigRowBuckets base buckets) are split over the
// groups of one block by k_stats_big
template <int G, int S, bool A>
__global__ void __launch_bounds__(256) k_stats(Tables t, StatsOut* out, u32* big) {
  const Group<G> g;
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  unsigned long long nbase = 0;
  StatsAcc a;
  for (u64 row = gid; row < t.rows; row += ng) {
    const DirEntry de = t.dir[row];
    nbase += de.nb;
    if (de.nb > kBigRowBuckets) {
      if (g.gl == 0) big[1 + atomicAdd(big, 1u)] = (u32)row;
      continue;
    }
    for (u32 k = 0; k < de.nb; ++k) stats_chain<G, S, A>(t, g, chain_head<A>(de.base, (u32)row, k), a);
  }
  if (g.gl == 0) {
    if (nbase) atomicAdd(&out->base_buckets, nbase);
    stats_flush(out, a);
  }
}

template <int G, int S, bool A>
__global__ void __launch_bounds__(256) k_stats_big(Tables t, StatsOut* out, const u32* big) {
  const Group<G> g;
  const u32 gib = threadIdx.x / G, ngb = blockDim.x / G;
  StatsAcc a;
  const u32 nbig = big[0];
  for (u32 i = blockIdx.x; i < nbig; i += gridDim.x) {
    const u32 row = big[1 + i];
    const DirEntry de = t.dir[row];
    for (u32 k = gib; k < de.nb; k += ngb) stats_chain<G, S, A>(t, g, chain_head<A>(de.base, row, k), a);
  }
  if (g.gl == 0) stats_flush(out, a);
}

cudaError_t launch_stats(int lay, const Tables& t, StatsOut* out, u32* big, int sms, cudaStream_t s) {
  cudaError_t e = cudaMemsetAsync(out, 0, sizeof(StatsOut), s);
  if (e == cudaSuccess) e = cudaMemsetAsync(big, 0, 4, s);
  if (e != cudaSuccess || t.rows == 0) return e;
  const int G = lay & 31;
  u64 blocks = (t.rows * G + 255) / 256;
  if (blocks > (u64)sms * 8) blocks = (u64)sms * 8;
  switch (lay) {
#define DG_CASE(G_, S_, A_)                                                  \
  case DG_LAYA(G_, S_, A_):                                                  \
    k_stats<G_, S_, A_><<<(unsigned)blocks, 256, 0, s>>>(t, out, big);       \
    k_stats_big<G_, S_, A_><<<(unsigned)sms * 2, 256, 0, s>>>(t, out, big);  \
    break;
    DG_FOR_LAYOUTS_A(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(2);
  return cudaGetLastError();
}

// ------------------------------------------------------- vertex deletion (a9) ----
// Mark the batch in a |V|-bit bitmap D (all ranks mark every deleted ID, since
// incoming edges may live on any shard), validate it (Q7/Q11), and list each
// distinct ID owned by this rank once (duplicates are idempotent).
// The coarse filter (kVdelFilterBits bits, bit = id >> fshift) is the bitmap at a
// coarser grain: the purge sweep keeps it in shared memory and reads the fine bitmap
// only for keys whose coarse bit is set.
__global__ void k_vdel_mark(const u32* ids, u64 n, u64 nv, u32 epoch, u32* bitmap, u32* filter,
                            u32 fshift, u32* dedup, DevCtl* ctl, u32 nranks, u32 rank) {
  bool bad = false;
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 i = (u64)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride) {
    const u32 id = ids[i];
    if ((u64)id >= nv) {
      bad = true;
      continue;
    }
    const u32 bit = 1u << (id & 31);
    const u32 old = atomicOr(&bitmap[id >> 5], bit);
    if (!(old & bit)) {
      const u32 c = id >> fshift;
      atomicOr(&filter[c >> 5], 1u << (c & 31));
      if (id % nranks == rank) dedup[atomicAdd(&ctl->dedup_count, 1u)] = id;
    }
  }
  if (__any_sync(0xFFFFFFFFu, bad) && (threadIdx.x & 31) == 0) atomicMax(&ctl->fail_epoch, epoch);
}

cudaError_t launch_vdel_mark(const u32* ids, u64 n, u64 nv, u32 epoch, u32* bitmap, u32* filter,
                             u32 fshift, u32* dedup, DevCtl* ctl, u32 nranks, u32 rank, int sms,
                             cudaStream_t s) {
  if (n == 0) return cudaSuccess;
  u64 blocks = (n + 255) / 256;
  if (blocks > (u64)sms * 8) blocks = (u64)sms * 8;
  k_vdel_mark<<<(unsigned)blocks, 256, 0, s>>>(ids, n, nv, epoch, bitmap, filter, fshift, dedup,
                                               ctl, nranks, rank); note_kernel(1);
  return cudaGetLastError();
}

// Directed purge ("a follow-up lookup and delete of all deleted
// vertices in all hash tables"): one streaming pass over every allocated bucket
// of the pool (coalesced, G lanes per bucket); every live key in D becomes a
// tombstone and the owner row's degree drops by one.
// One launch per size class c: the pool of class c holds buckets of G units.
// H: the home pool (uniform layouts; bucket r = row r's chain 0) instead of pool
// `cls` (a second launch; one merged pass over both measured slower).
template <int G, int S, bool H = false>
__global__ void __launch_bounds__(256) k_vdel_sweep(Tables t, const u32* __restrict__ bitmap,
                                                    const u32* __restrict__ filter, u32 fshift,
                                                    u32 epoch, u32 cls) {
  typedef Lay<G, S> LY;
  constexpr int W = LY::W;
#ifndef DG_SWEEP_U
#define DG_SWEEP_U 4
#endif
  constexpr int U = DG_SWEEP_U;  // buckets in flight per group (memory-level parallelism)
#ifndef DG_SWEEP_SKIP
#define DG_SWEEP_SKIP 0
#endif
  __shared__ u32 sf[kVdelFilterBits / 32];
  const Group<G> g;
  if (ld_relaxed_u32(&t.ctl->fail_epoch) == epoch) return;
  for (u32 i = threadIdx.x; i < kVdelFilterBits / 32; i += blockDim.x) sf[i] = filter[i];
  __syncthreads();
  const u32 nbk = H ? (u32)t.rows : ld_relaxed_u32(&t.ctl->bump[cls]);
  u32* const pool = H ? t.home : by_class(t.pool, cls);
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  for (u64 b0 = gid; b0 < nbk; b0 += ng * U) {
#if DG_SWEEP_SKIP
    // slots fill in order and EMPTY slots only exist at the tail (the probe
    // invariant), so a bucket whose slot 0 is EMPTY holds no key: read its first
    // word only (one 32-B sector instead of the whole bucket)
    u32 live = 0;
#pragma unroll
    for (int k0 = 0; k0 < U; k0 += G) {
      const u32 k = k0 + g.gl;
      const u64 b = b0 + (u64)k * ng;
      const bool l = k < (u32)U && b < nbk && pool[b * W] != kEmpty;
      live |= g.ballot(l) << k0;
    }
#else
    constexpr u32 live = 0xFFFFFFFFu;
#endif
    uint4 q[U];
#pragma unroll
    for (int k = 0; k < U; ++k) {
      const u64 b = (live >> k) & 1u ? b0 + (u64)k * ng : nbk;
#ifdef DG_SWEEP_LDCS
      q[k] = b < nbk ? __ldcs(reinterpret_cast<const uint4*>(pool + b * W + 4 * g.gl))
                     : make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
#else
      q[k] = b < nbk ? *reinterpret_cast<const uint4*>(pool + b * W + 4 * g.gl)
                     : make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
#endif
    }
#pragma unroll
    for (int k = 0; k < U; ++k) {
      const u64 b = b0 + (u64)k * ng;
      u32* bp = pool + b * W;
      const uint4 x = q[k];
      const u32 owner = H ? (u32)b : g.shfl(x.w, G - 1);  // (home: word W-1 = degree)
      u32 dec = 0;
#pragma unroll
      for (int j = 0; j < LY::SPU; ++j) {
        const u32 kk = LY::key(x, j);
        if (!LY::has(g.gl, j) || kk >= kTomb) continue;
        const u32 c = kk >> fshift;
        if (((sf[c >> 5] >> (c & 31)) & 1u) && ((__ldg(bitmap + (kk >> 5)) >> (kk & 31)) & 1u) &&
            atomicCAS(bp + LY::word(g.gl, j), kk, kTomb) == kk)
          ++dec;
      }
      if (dec) atomicSub(deg_at(t, owner), dec);
    }
  }
}

cudaError_t launch_vdel_sweep(int lay, const Tables& t, const u32* bitmap, const u32* filter,
                              u32 fshift, u32 epoch, int sms, cudaStream_t s) {
  const unsigned blocks = (unsigned)sms * 8;
  if (lay & DG_ADAPTIVE_BIT) {  // one sweep per size class pool (32 / 64 / 128 B)
    if (lay & 32) {
      k_vdel_sweep<2, 1><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 0);
      k_vdel_sweep<4, 1><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 1);
      k_vdel_sweep<8, 1><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 2);
    } else {
      k_vdel_sweep<2, 0><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 0);
      k_vdel_sweep<4, 0><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 1);
      k_vdel_sweep<8, 0><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 2);
    }
    note_kernel(3);
    return cudaGetLastError();
  }
  switch (lay) {  // uniform layouts: the pool, then the home buckets
#define DG_CASE(G_, S_)                                                                      \
  case DG_LAY(G_, S_):                                                                       \
    k_vdel_sweep<G_, S_><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 0);        \
    k_vdel_sweep<G_, S_, true><<<blocks, 256, 0, s>>>(t, bitmap, filter, fshift, epoch, 0);  \
    break;
    DG_FOR_LAYOUTS(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(2);
  return cudaGetLastError();
}

// probe used by the undirected purge: delete key v from the table starting at b
template <int G, int S, bool A>
__device__ __forceinline__ int purge_delete(const Tables& t, const Group<G>& g, u32 b, u32 v) {
  typedef Lay<G, S> LY;
  while (true) {
    const Geo<G, S, A> gb(t, b);
    u32* bp = gb.p;
    const uint4 q = (A && g.gl >= gb.units) ? make_uint4(kEmpty, kEmpty, kEmpty, kEmpty)
                                            : ld_relaxed_v4(bp + 4 * g.gl);
    bool m = false, e = false;
    u32 wd = 0;
#pragma unroll
    for (int j = 0; j < LY::SPU; ++j) {
      const bool h = gb.has(g.gl, j);
      if (h && !m && LY::key(q, j) == v) { m = true; wd = LY::word(g.gl, j); }
      e |= h && LY::key(q, j) == kEmpty;
    }
    const u32 hit = g.ballot(m);
    if (hit) {
      const u32 l = __ffs(hit) - 1;
      u32 old = 0;
      if (g.gl == l) old = atomicCAS(bp + wd, v, kTomb);
      return g.shfl(old, l) == v ? 1 : 0;
    }
    if (g.ballot(e)) return 0;
    const u32 next = g.shfl(q.z, gb.units - 1);
    if (next == kNil) return 0;
    b = next;
  }
}

// The per-vertex purge kernels below are flattened to one group per (deleted
// vertex, base bucket): boff[k] = sum of the base-bucket counts of the first k
// distinct deleted vertices, so a hub's thousands of base buckets are cleared in
// parallel instead of by one group (the paper balances per vertex with an atomic
// queue, Alg2:L3-6; a bucket-granular split also balances hubs).
__global__ void k_vdel_nb(const u32* dedup, const DevCtl* ctl, u64 n_max, const DirEntry* dir,
                          u32 nranks, u64* nbarr) {
  const u32 cnt = ctl->dedup_count;
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 k = (u64)blockIdx.x * blockDim.x + threadIdx.x; k <= n_max; k += stride)
    nbarr[k] = k < cnt ? (u64)dir[dedup[k] / nranks].nb : 0ull;
}

cudaError_t launch_vdel_nb(const Tables& t, const u32* dedup, u64 n_max, u64* nbarr, int sms,
                           cudaStream_t s) {
  u64 blocks = (n_max + 1 + 255) / 256;
  if (blocks > (u64)sms * 8) blocks = (u64)sms * 8;
  k_vdel_nb<<<(unsigned)blocks, 256, 0, s>>>(dedup, t.ctl, n_max, t.dir, t.nranks, nbarr); note_kernel(1);
  return cudaGetLastError();
}

// largest k < cnt with boff[k] <= x
__device__ __forceinline__ u32 owner_of(const u64* boff, u32 cnt, u64 x) {
  u32 lo = 0, hi = cnt;  // boff[lo] <= x < boff[hi] (boff[cnt] = total)
  while (hi - lo > 1) {
    const u32 mid = (lo + hi) >> 1;
    if (boff[mid] <= x) lo = mid;
    else hi = mid;
  }
  return lo;
}

// Undirected purge, Alg. 2: for every deleted vertex u,
// iterate over A_u (L11-12) and delete u from A_v of every neighbour v (L13-17).
// Valid only for graphs kept symmetric (directed = 0, single rank).
template <int G, int S, bool A>
__global__ void __launch_bounds__(256) k_vdel_neighbors(Tables t, const u32* dedup,
                                                        const u64* boff, u32 epoch) {
  typedef Lay<G, S> LY;
  const Group<G> g;
  if (ld_relaxed_u32(&t.ctl->fail_epoch) == epoch) return;
  const u32 cnt = ld_relaxed_u32(&t.ctl->dedup_count);
  if (cnt == 0) return;
  const u64 total = boff[cnt];
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  for (u64 x = gid; x < total; x += ng) {
    const u32 k = owner_of(boff, cnt, x);
    const u32 u = dedup[k];
    u32 b = chain_head<A>(t.dir[u].base, u, (u32)(x - boff[k]));
    while (b != kNil) {
      const Geo<G, S, A> gb(t, b);
      const uint4 q = (A && g.gl >= gb.units) ? make_uint4(kEmpty, kEmpty, kEmpty, kEmpty)
                                              : ld_relaxed_v4(gb.p + 4 * g.gl);
#pragma unroll
      for (int j = 0; j < LY::SPU; ++j) {
        u32 lm = g.ballot(gb.has(g.gl, j) && LY::key(q, j) < kTomb);
        while (lm) {
          const u32 l = __ffs(lm) - 1;
          lm &= lm - 1;
          const u32 v = g.shfl(LY::key(q, j), l);
          const DirEntry dv = t.dir[v];
          if (purge_delete<G, S, A>(t, g, chain_head<A>(dv.base, v, bucket_of(u, dv.nb)), u) &&
              g.gl == 0)
            atomicSub(deg_at(t, v), 1u);
        }
      }
      b = g.shfl(q.z, gb.units - 1);
    }
  }
}

cudaError_t launch_vdel_neighbors(int lay, const Tables& t, const u32* dedup, const u64* boff,
                                  u32 epoch, int sms, cudaStream_t s) {
  const unsigned blocks = (unsigned)sms * 8;
  switch (lay) {
#define DG_CASE(G_, S_, A_)                                                               \
  case DG_LAYA(G_, S_, A_):                                                               \
    k_vdel_neighbors<G_, S_, A_><<<blocks, 256, 0, s>>>(t, dedup, boff, epoch);           \
    break;
    DG_FOR_LAYOUTS_A(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(1);
  return cudaGetLastError();
}

// Owner clear (Alg2:L18-22): walk A_u; chained buckets are reset to EMPTY and
// pushed on the free stack (dynamic memory reclaimed); base buckets
// are reset to EMPTY in place (Q9: static memory is kept but must not keep stale
// keys); degree := 0.  One group per (vertex, base bucket).
template <int G, bool A>
__global__ void __launch_bounds__(256) k_vdel_clear(Tables t, const u32* dedup, const u64* boff,
                                                    u32 epoch) {
  const Group<G> g;
  if (ld_relaxed_u32(&t.ctl->fail_epoch) == epoch) return;
  const u32 cnt = ld_relaxed_u32(&t.ctl->dedup_count);
  if (cnt == 0) return;
  const u64 total = boff[cnt];
  const uint4 empty4 = make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  for (u64 x = gid; x < total; x += ng) {
    const u32 k = owner_of(boff, cnt, x);
    const u32 row = dedup[k] / t.nranks;
    const u32 j = (u32)(x - boff[k]);
    u32 b = chain_head<A>(t.dir[row].base, row, j);
    bool base_bucket = true;
    while (b != kNil) {
      const Geo<G, 0, A> gb(t, b);
      const bool in = !A || g.gl < gb.units;
      u32* bp = gb.p + 4 * g.gl;
      const uint4 q = in ? ld_relaxed_v4(bp) : empty4;
      const u32 next = g.shfl(q.z, gb.units - 1);
      if (g.gl == gb.units - 1)  // (a home bucket's last word is the degree := 0)
        st_v4(bp, make_uint4(kEmpty, kEmpty, kNil, gb.home ? 0u : base_bucket ? row : kNil));
      else if (in) st_v4(bp, empty4);
      if (!base_bucket && g.gl == 0) {
        const u32 c = b >> kClassShift;
        by_class(t.stack, c)[atomicAdd(&t.ctl->stack_size[c], 1u)] = b;
      }
      base_bucket = false;
      b = next;
    }
    if (!t.hw && j == 0 && g.gl == 0) t.deg[row] = 0;  // (else the home-word store above)
  }
}

cudaError_t launch_vdel_clear(int lay, const Tables& t, const u32* dedup, const u64* boff,
                              u32 epoch, int sms, cudaStream_t s) {
  const unsigned blocks = (unsigned)sms * 8;
  if (lay & DG_ADAPTIVE_BIT) {
    k_vdel_clear<8, true><<<blocks, 256, 0, s>>>(t, dedup, boff, epoch);
    note_kernel(1);
    return cudaGetLastError();
  }
  switch (lay & 31) {
    case 2: k_vdel_clear<2, false><<<blocks, 256, 0, s>>>(t, dedup, boff, epoch); note_kernel(1); break;
    case 4: k_vdel_clear<4, false><<<blocks, 256, 0, s>>>(t, dedup, boff, epoch); note_kernel(1); break;
    case 8: k_vdel_clear<8, false><<<blocks, 256, 0, s>>>(t, dedup, boff, epoch); note_kernel(1); break;
    default: return cudaErrorInvalidValue;
  }
  return cudaGetLastError();
}

}  // namespace dg
