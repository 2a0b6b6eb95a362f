// kernels_tc.cu — triangle counting by per-vertex hash intersection (a13; §VI-C,
// P:L848-864): the query-bound application the paper runs on its structure.
//
//   rank(x) = (deg x, x);  N+(u) = {v in A_u : rank(v) > rank(u)}  (orientation)
//   count = sum over u, over pairs i < j of N+(u):  [ N+(u)[j] in A_{N+(u)[i]} ]
// Each triangle {a, b, c} with a the lowest rank is counted once, at u = a, for the
// pair {b, c}.  Because the graph is symmetric (undirected mode), c in A_b iff
// b in A_c, so the pair can probe either table; we probe A_{N+(u)[i]} for every
// later entry — one edgeExist per wedge.
//
// Steps (dg_triangle_count): the adjacency export (a12) gives CSR (ro, dst); then
//   k_tc_orient_count : warp per row, |N+(u)| (degree lookups of the neighbours)
//   scan              : oriented row offsets
//   k_tc_orient_fill  : warp per row, ballot-compacted N+(u) + end index per entry
//   k_tc_wedges       : one thread per oriented entry e = (u, i): probe the hash
//                       table of v_i for every later v_j of N+(u); whole buckets
//                       are read with 16-B loads, hits reduced per warp.
#include <cub/device/device_radix_sort.cuh>
#include <cub/device/device_scan.cuh>
#include <cub/device/device_select.cuh>
#include <thrust/iterator/counting_iterator.h>
#include <thrust/iterator/transform_iterator.h>

#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

__device__ __forceinline__ bool rank_less(u32 du, u32 u, u32 dv, u32 v) {
  return du < dv || (du == dv && u < v);
}

// warp per row; rows with more than kBigRowDegree neighbours (hubs) are listed in
// big[1..] (count big[0]) and oriented by the *_big kernels, one block per row.
__global__ void __launch_bounds__(256) k_tc_orient_count(const u64* ro, const u32* dst,
                                                         const u32* deg, u64 rows, u32 part,
                                                         u32 nparts, u64* ocnt, u32* big) {
  const u32 lane = threadIdx.x & 31;
  const u64 wid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nw = ((u64)gridDim.x * blockDim.x) >> 5;
  for (u64 u = wid; u < rows; u += nw) {
    u32 c = 0;
    if (u % nparts == part) {
      const u64 r0 = ro[u], r1 = ro[u + 1];
      if (r1 - r0 > kBigRowDegree) {
        if (lane == 0) big[1 + atomicAdd(big, 1u)] = (u32)u;
        continue;
      }
      const u32 du = deg[u];
      for (u64 k = r0 + lane; k < r1; k += 32) {
        const u32 v = dst[k];
        c += rank_less(du, (u32)u, __ldg(&deg[v]), v) ? 1u : 0u;
      }
      c = __reduce_add_sync(0xFFFFFFFFu, c);
    }
    if (lane == 0) ocnt[u] = c;
  }
  if (blockIdx.x == 0 && threadIdx.x == 0) ocnt[rows] = 0;
}

__global__ void __launch_bounds__(256) k_tc_orient_count_big(const u64* ro, const u32* dst,
                                                             const u32* deg, u64* ocnt,
                                                             const u32* big) {
  __shared__ u32 total;
  const u32 nbig = big[0];
  for (u32 i = blockIdx.x; i < nbig; i += gridDim.x) {
    const u32 u = big[1 + i];
    const u32 du = deg[u];
    __syncthreads();
    if (threadIdx.x == 0) total = 0;
    __syncthreads();
    u32 c = 0;
    for (u64 k = ro[u] + threadIdx.x; k < ro[u + 1]; k += blockDim.x) {
      const u32 v = dst[k];
      c += rank_less(du, u, __ldg(&deg[v]), v) ? 1u : 0u;
    }
    c = __reduce_add_sync(0xFFFFFFFFu, c);
    if ((threadIdx.x & 31) == 0 && c) atomicAdd(&total, c);
    __syncthreads();
    if (threadIdx.x == 0) ocnt[u] = total;
  }
}

__global__ void __launch_bounds__(256) k_tc_orient_fill(const u64* ro, const u32* dst,
                                                        const u32* deg, u64 rows, u32 part,
                                                        u32 nparts, const u64* oro, u32* oadj,
                                                        u32* oend) {
  const u32 lane = threadIdx.x & 31;
  const u64 wid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nw = ((u64)gridDim.x * blockDim.x) >> 5;
  for (u64 u = wid; u < rows; u += nw) {
    if (u % nparts != part) continue;
    if (ro[u + 1] - ro[u] > kBigRowDegree) continue;  // k_tc_orient_fill_big
    const u32 du = deg[u];
    u64 pos = oro[u];
    const u32 end = (u32)oro[u + 1];
    for (u64 k0 = ro[u]; k0 < ro[u + 1]; k0 += 32) {
      const u64 k = k0 + lane;
      bool keep = false;
      u32 v = 0;
      if (k < ro[u + 1]) {
        v = dst[k];
        keep = rank_less(du, (u32)u, __ldg(&deg[v]), v);
      }
      const u32 m = __ballot_sync(0xFFFFFFFFu, keep);
      if (keep) {
        const u64 at = pos + __popc(m & ((1u << lane) - 1u));
        oadj[at] = v;
        oend[at] = end;
      }
      pos += __popc(m);
    }
  }
}

// hub rows: warps of one block take 32-entry pieces; positions from a block cursor
// (the order of N+(u) is immaterial: every pair i < j is probed once)
__global__ void __launch_bounds__(256) k_tc_orient_fill_big(const u64* ro, const u32* dst,
                                                            const u32* deg, const u64* oro,
                                                            u32* oadj, u32* oend, const u32* big) {
  __shared__ unsigned long long cursor;
  const u32 lane = threadIdx.x & 31;
  const u32 nbig = big[0];
  for (u32 i = blockIdx.x; i < nbig; i += gridDim.x) {
    const u32 u = big[1 + i];
    const u32 du = deg[u];
    const u32 end = (u32)oro[u + 1];
    __syncthreads();
    if (threadIdx.x == 0) cursor = oro[u];
    __syncthreads();
    for (u64 k0 = ro[u] + (threadIdx.x & ~31u); k0 < ro[u + 1]; k0 += blockDim.x) {
      const u64 k = k0 + lane;
      bool keep = false;
      u32 v = 0;
      if (k < ro[u + 1]) {
        v = dst[k];
        keep = rank_less(du, u, __ldg(&deg[v]), v);
      }
      const u32 m = __ballot_sync(0xFFFFFFFFu, keep);
      unsigned long long pos = 0;
      if (lane == 0 && m) pos = atomicAdd(&cursor, (unsigned long long)__popc(m));
      pos = __shfl_sync(0xFFFFFFFFu, pos, 0);
      if (keep) {
        const u64 at = pos + __popc(m & ((1u << lane) - 1u));
        oadj[at] = v;
        oend[at] = end;
      }
    }
  }
}

// Wedge probes, organised like the edge-query kernel: a group of G lanes owns one
// oriented entry e = (u, i) at a time (32/G entries per warp, consecutive entries
// of a row have similar candidate counts); per step every lane takes one candidate
// w = N+(u)[j] and the group loads the G candidates' buckets of A_v together (one
// 16-B load per lane per candidate), then decides all G with group ballots.  Warp
// loops are warp-uniform so every intrinsic uses the full mask.  The rare probes
// whose key may sit further down a chain are walked by their own lane.
__global__ void k_iota(u32* out, u64 n) {
  for (u64 i = (u64)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += (u64)gridDim.x * blockDim.x)
    out[i] = (u32)i;
}

// perm (nullable): the entries in probe order — sorted by the probed vertex v, so the
// probes into one table A_v run close together in time and its buckets are read from
// DRAM about once instead of once per probe (launch_tc_probe_order)
template <int G, int S, bool A>
__global__ void __launch_bounds__(256, 4) k_tc_wedges(Tables t, const u32* __restrict__ oadj,
                                                      const u32* __restrict__ oend,
                                                      const u32* __restrict__ perm, u64 n_units,
                                                      unsigned long long* count) {
  typedef Lay<G, S> LY;
  typedef Geo<G, S, A> GEO;
  constexpr u32 FULL = 0xFFFFFFFFu;
  constexpr u32 GBITS = (G == 32) ? 0xFFFFFFFFu : ((1u << G) - 1u);
  constexpr int PER_WARP = 32 / G;
  const Group<G> g;
  u32 hits = 0;
  const u64 warp = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nwarps = ((u64)gridDim.x * blockDim.x) >> 5;
  for (u64 e0 = warp * PER_WARP; e0 < n_units; e0 += nwarps * PER_WARP) {
    const u64 ei = e0 + g.lane / G;               // this group's entry
    const bool ev = ei < n_units;
    const u64 e = (perm && ev) ? (u64)__ldg(perm + ei) : ei;
    const u32 v = ev ? __ldg(oadj + e) : 0u;
    const u32 ncand = ev ? __ldg(oend + e) - (u32)e - 1u : 0u;
    const uint2 dv = ev ? ld_nc_dir(t.dir + v) : make_uint2(0, 1);
    const u32 units = units_of<G, A>(dv.x);  // every probe of the group is into A_v
    const bool lastl = g.gl == units - 1;
    const bool inb = g.gl < units;
    const u32 maxc = __reduce_max_sync(FULL, ncand);
    for (u32 k0 = 0; k0 < maxc; k0 += G) {
      const bool act = k0 + g.gl < ncand;
      const u32 w = act ? __ldg(oadj + e + 1 + k0 + g.gl) : kEmpty;
      const u32 head = chain_head<A>(dv.x, v, bucket_of(w, dv.y));
      const u32 amask = __ballot_sync(FULL, act);
      uint4 q[G];
#pragma unroll
      for (int r = 0; r < G; ++r) {
        const u32 hr = __shfl_sync(FULL, head, g.base + r);
        if (((amask >> (g.base + r)) & 1u) && inb) q[r] = ld_nc_v4(GEO(t, hr).p + 4 * g.gl);
        else q[r] = make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
      }
      bool walk = false;
      u32 nxt = kNil;
#pragma unroll
      for (int r = 0; r < G; ++r) {
        const uint4 x = q[r];
        const u32 wr = __shfl_sync(FULL, w, g.base + r);
        const bool pr = (amask >> (g.base + r)) & 1u;
        bool m = false, e = false;
#pragma unroll
        for (int j = 0; j < LY::SPU; ++j) {
          const bool h = inb && (!lastl || j < LY::SPU / 2);
          m |= h && LY::key(x, j) == wr;
          e |= h && LY::key(x, j) == kEmpty;
        }
        const u32 hit = (__ballot_sync(FULL, pr && m) >> g.base) & GBITS;
        const u32 em = (__ballot_sync(FULL, e) >> g.base) & GBITS;
        const u32 next = __shfl_sync(FULL, x.z, g.base + units - 1);
        if (pr && g.gl == (u32)r) {
          if (hit) ++hits;
          else if (!em && next != kNil) { walk = true; nxt = next; }
        }
      }
      // rare: the key may sit further down the chain (edgeExist)
      if (walk) {
        u32 b = nxt;
        while (b != kNil) {
          const GEO gb(t, b);
          const uint4* bp = reinterpret_cast<const uint4*>(gb.p);
          bool found = false, ended = false;
          u32 nb2 = kNil;
#pragma unroll
          for (int c = 0; c < G; ++c) {
            if (A && (u32)c >= gb.units) break;
            const uint4 y = __ldg(bp + c);
#pragma unroll
            for (int j = 0; j < LY::SPU; ++j) {
              if (gb.has(c, j)) {
                found |= LY::key(y, j) == w;
                ended |= LY::key(y, j) == kEmpty;
              }
            }
            if ((u32)c == gb.units - 1) nb2 = y.z;
          }
          if (found) { ++hits; break; }
          if (ended) break;
          b = nb2;
        }
      }
    }
  }
  const u32 tot = __reduce_add_sync(FULL, hits);
  if ((threadIdx.x & 31) == 0 && tot) atomicAdd(count, (unsigned long long)tot);
}

cudaError_t launch_tc_orient_count(const Tables& t, const u64* ro, const u32* dst, u32 part,
                                   u32 nparts, u64* ocnt, u32* big, int sms, cudaStream_t s) {
  cudaError_t e = cudaMemsetAsync(big, 0, 4, s);
  if (e != cudaSuccess) return e;
  // uniform layouts keep degrees in the home buckets: snapshot them into t.deg (one
  // 32-B sector per row) so the orientation's random degree reads hit a dense array
  if (t.hw && (e = launch_degrees(t, t.deg, s)) != cudaSuccess) return e;
  k_tc_orient_count<<<(unsigned)sms * 8, 256, 0, s>>>(ro, dst, t.deg, t.rows, part, nparts, ocnt,
                                                      big);
  k_tc_orient_count_big<<<(unsigned)sms * 2, 256, 0, s>>>(ro, dst, t.deg, ocnt, big);
  note_kernel(2);
  return cudaGetLastError();
}

// big: the hub-row list left by launch_tc_orient_count
cudaError_t launch_tc_orient_fill(const Tables& t, const u64* ro, const u32* dst, u32 part,
                                  u32 nparts, const u64* oro, u32* oadj, u32* oend,
                                  const u32* big, int sms, cudaStream_t s) {
  k_tc_orient_fill<<<(unsigned)sms * 8, 256, 0, s>>>(ro, dst, t.deg, t.rows, part, nparts, oro, oadj,
                                                     oend);
  k_tc_orient_fill_big<<<(unsigned)sms * 2, 256, 0, s>>>(ro, dst, t.deg, oro, oadj, oend, big);
  note_kernel(2);
  return cudaGetLastError();
}

// ---------------------------------------------------------- flat wedges ----
// Load-balanced form of the wedge probes: the wedges of all entries with at least one
// candidate are numbered 0 .. W-1 in entry order (woff = exclusive scan of the entries'
// candidate counts over the compacted entry list `list` of (entry, probed vertex v)
// pairs), split into chunks of kTcChunk wedges taken grid-stride by the warps (so the
// warps work on neighbouring wedges at any moment: with the probe order the tables
// they probe are the same few), and every LANE probes one wedge: w = the candidate,
// A_v its entry's table, the lane reading the whole bucket with 16-B loads.  No warp waits on its longest entry (the per-entry
// kernel above runs each warp to the largest candidate count of its 32 / G entries)
// and there is no per-entry setup.
// Entry of each lane: lane j reads the start of entry k0 + 1 + j; the starts inside
// the 32-wedge window (and one at its end, bit 32) form a mask whose popcounts give
// every lane its entry and whose highest set bit its entry's start (entries are
// non-empty, so starts are distinct).  The next window's starts are loaded before the
// current window's probes run.
constexpr u32 kTcChunk = 256;  // wedges per chunk (8 windows of 32)

// chunk_k[c] = the entry holding wedge c * kTcChunk (every entry writes the chunks
// whose first wedge it holds)
__global__ void k_tc_chunk_entries(const u64* __restrict__ woff,
                                   const unsigned long long* n_list_dev, u32* chunk_k) {
  const u64 n_list = *n_list_dev;
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 k = (u64)blockIdx.x * blockDim.x + threadIdx.x; k < n_list; k += stride) {
    const u64 a = woff[k], b = woff[k + 1];
    for (u64 c = (a + kTcChunk - 1) / kTcChunk; c * kTcChunk < b; ++c) chunk_k[c] = (u32)k;
  }
}

template <int G, int S>
__global__ void __launch_bounds__(256) k_tc_wedges_flat(Tables t, const u32* __restrict__ oadj,
                                                        const uint2* __restrict__ list,
                                                        const u64* __restrict__ woff,
                                                        const u32* __restrict__ chunk_k,
                                                        const unsigned long long* n_list_dev,
                                                        unsigned long long* count) {
  typedef Lay<G, S> LY;
  typedef Geo<G, S, false> GEO;
  constexpr u32 FULL = 0xFFFFFFFFu;
  const u64 n_list = *n_list_dev;
  if (n_list == 0) return;
  const u64 W = woff[n_list];
  const u32 lane = threadIdx.x & 31u;
  const u64 warp = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nwarps = ((u64)gridDim.x * blockDim.x) >> 5;
  const u64 nchunks = (W + kTcChunk - 1) / kTcChunk;
  u32 hits = 0;
  for (u64 ch = warp; ch < nchunks; ch += nwarps) {
  // this chunk's wedges [x_lo, x_hi) in 32-wedge windows; k0 holds x_lo, s0 its start
  const u64 x_lo = ch * kTcChunk;
  const u64 x_hi = x_lo + kTcChunk < W ? x_lo + kTcChunk : W;
  u64 k0 = __ldg(chunk_k + ch);
  u64 s0 = woff[k0];
  const u32 upto = lane == 31 ? FULL : ((2u << lane) - 1u);
  // starts of entries k0+1 .. k0+32 relative to x0: bits 0..31 (lo) and bit 32 (hi)
  auto window = [&](u64 k0w, u64 x0, u32& mlo, u32& mhi) {
    const u64 kj = k0w + 1 + lane;
    u64 bit = 0;
    if (kj < n_list) {
      const u64 sj = woff[kj] - x0;
      if (sj <= 32) bit = 1ull << sj;
    }
    mlo = __reduce_or_sync(FULL, (u32)bit);
    mhi = __reduce_or_sync(FULL, (u32)(bit >> 32));
  };
  u32 mlo, mhi;
  window(k0, x_lo, mlo, mhi);
  for (u64 x0 = x_lo; x0 < x_hi; x0 += 32) {
    const u64 x = x0 + lane;
    const u32 mine = mlo & upto;
    const u64 k = k0 + __popc(mine);
    const u64 start = mine ? x0 + 31 - __clz(mine) : s0;
    // the next window: entry, start, and its starts' loads in flight during the probes
    const u64 k0n = k0 + __popc(mlo) + (mhi & 1u);
    const u64 s0n = (mhi & 1u) ? x0 + 32 : (mlo ? x0 + 31 - __clz(mlo) : s0);
    u32 nlo = 0, nhi = 0;
    if (x0 + 32 < x_hi) window(k0n, x0 + 32, nlo, nhi);
    if (x < x_hi) {
      const uint2 ev = __ldg(list + k);  // (entry, probed vertex)
      const u32 w = __ldg(oadj + ev.x + 1 + (x - start));
      const uint2 dv = ld_nc_dir(t.dir + ev.y);
      u32 b = chain_head<false>(dv.x, ev.y, bucket_of(w, dv.y));
      // edgeExist: the chain of A_v that w hashes to
      while (b != kNil) {
        const uint4* bp = reinterpret_cast<const uint4*>(GEO(t, b).p);
        uint4 y[G];
#pragma unroll
        for (int c2 = 0; c2 < G; ++c2) y[c2] = __ldg(bp + c2);
        bool found = false;
#pragma unroll
        for (int c2 = 0; c2 < G; ++c2) {
#pragma unroll
          for (int j = 0; j < LY::SPU; ++j) {
            if (!LY::has(c2, j)) continue;
            found |= LY::key(y[c2], j) == w;
          }
        }
        if (found) { ++hits; break; }
        // EMPTY slots form the chain's suffix: the chain ends in this
        // bucket iff its last slot is EMPTY (one compare instead of one per slot)
        if (LY::key(y[G - 1], LY::SPU / 2 - 1) == kEmpty) break;
        b = y[G - 1].z;
      }
    }
    k0 = k0n;
    s0 = s0n;
    mlo = nlo;
    mhi = nhi;
  }
  }
  const u32 tot = __reduce_add_sync(FULL, hits);
  if (lane == 0 && tot) atomicAdd(count, (unsigned long long)tot);
}

namespace {
struct EntryPair {  // entry e -> (e, probed vertex oadj[e])
  const u32* oadj;
  __host__ __device__ uint2 operator()(u32 e) const { return make_uint2(e, oadj[e]); }
};
struct HasCand {  // the entry has at least one later candidate
  const u32* oend;
  __host__ __device__ bool operator()(const uint2& p) const { return oend[p.x] > p.x + 1; }
};
struct CandOf {  // candidates of the k-th listed entry
  const u32* oend;
  const uint2* list;
  u64 n;
  __host__ __device__ u64 operator()(u64 k) const {
    return k < n ? (u64)(oend[list[k].x] - list[k].x - 1) : 0ull;
  }
};
}  // namespace

u64 tc_chunk_count(u64 wedges) { return wedges / kTcChunk + 1; }

// list: entries with >= 1 candidate, in `order` (nullable: entry order); woff: their
// wedge offsets (n_list + 1); n_list_dev / *n_list: their number.  Synchronises s.
cudaError_t launch_tc_flat_prepare(const u32* oadj, const u32* oend, const u32* order, u64 n_units,
                                   uint2* list, u64* woff, unsigned long long* n_list_dev,
                                   u64* n_list, void** temp, size_t* temp_bytes, cudaStream_t s) {
  *n_list = 0;
  if (n_units == 0 || n_units >= (1ull << 31)) return cudaSuccess;
  const int n = (int)n_units;
  size_t need = 0;
  cudaError_t e;
  auto grow = [&](size_t want) -> cudaError_t {
    if (want <= *temp_bytes) return cudaSuccess;
    if (*temp) cudaFree(*temp);
    *temp = nullptr;
    *temp_bytes = 0;
    cudaError_t r = cudaMalloc(temp, want);
    if (r == cudaSuccess) *temp_bytes = want;
    return r;
  };
  if (order) {
    auto in = thrust::make_transform_iterator(order, EntryPair{oadj});
    e = cub::DeviceSelect::If(nullptr, need, in, list, n_list_dev, n, HasCand{oend}, s);
    if (e != cudaSuccess || (e = grow(need)) != cudaSuccess) return e;
    e = cub::DeviceSelect::If(*temp, need, in, list, n_list_dev, n, HasCand{oend}, s);
  } else {
    auto in = thrust::make_transform_iterator(thrust::counting_iterator<u32>(0), EntryPair{oadj});
    e = cub::DeviceSelect::If(nullptr, need, in, list, n_list_dev, n, HasCand{oend}, s);
    if (e != cudaSuccess || (e = grow(need)) != cudaSuccess) return e;
    e = cub::DeviceSelect::If(*temp, need, in, list, n_list_dev, n, HasCand{oend}, s);
  }
  if (e != cudaSuccess) return e;
  unsigned long long nl = 0;
  if ((e = cudaMemcpyAsync(&nl, n_list_dev, 8, cudaMemcpyDeviceToHost, s)) != cudaSuccess) return e;
  if ((e = cudaStreamSynchronize(s)) != cudaSuccess) return e;
  *n_list = nl;
  auto it = thrust::make_transform_iterator(thrust::counting_iterator<u64>(0),
                                            CandOf{oend, list, (u64)nl});
  need = 0;
  e = cub::DeviceScan::ExclusiveSum(nullptr, need, it, woff, (int64_t)(nl + 1), s);
  if (e != cudaSuccess || (e = grow(need)) != cudaSuccess) return e;
  e = cub::DeviceScan::ExclusiveSum(*temp, need, it, woff, (int64_t)(nl + 1), s);
  note_kernel(3);
  return e;
}

// chunk_k: (total wedges / kTcChunk + 1) u32 (tc_chunk_count)
cudaError_t launch_tc_wedges_flat(int lay, const Tables& t, const u32* oadj, const uint2* list,
                                  const u64* woff, u32* chunk_k,
                                  const unsigned long long* n_list_dev,
                                  unsigned long long* count, int sms, cudaStream_t s) {
  k_tc_chunk_entries<<<(unsigned)sms * 8, 256, 0, s>>>(woff, n_list_dev, chunk_k);
  note_kernel(1);
  switch (lay) {
#define DG_CASE(G_, S_)                                                                     \
  case DG_LAY(G_, S_):                                                                      \
    k_tc_wedges_flat<G_, S_><<<(unsigned)sms * 8, 256, 0, s>>>(t, oadj, list, woff, chunk_k, \
                                                             n_list_dev, count);           \
    break;
    DG_FOR_LAYOUTS(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(1);
  return cudaGetLastError();
}

// Probe order of the wedge kernel: the oriented entries sorted by their probed vertex
// oadj[e] (CUB radix sort of (v, e) pairs over the bits of the row count).  keys /
// vals: 2 x n_units u32 each (double buffers); returns the sorted entry ids in *perm.
cudaError_t launch_tc_probe_order(const u32* oadj, u64 n_units, u64 rows, u32* keys, u32* vals,
                                  const u32** perm, void** temp, size_t* temp_bytes,
                                  cudaStream_t s) {
  if (n_units == 0 || n_units >= (1ull << 31)) { *perm = nullptr; return cudaSuccess; }
  const int n = (int)n_units;
  int bits = 1;
  while (bits < 32 && (1ull << bits) < rows) ++bits;
  cudaError_t e = cudaMemcpyAsync(keys, oadj, n_units * 4, cudaMemcpyDeviceToDevice, s);
  if (e != cudaSuccess) return e;
  k_iota<<<(unsigned)((n_units + 255) / 256 < 65535 ? (n_units + 255) / 256 : 65535), 256, 0, s>>>(vals, n_units);
  cub::DoubleBuffer<u32> kb(keys, keys + n_units), vb(vals, vals + n_units);
  size_t need = 0;
  e = cub::DeviceRadixSort::SortPairs(nullptr, need, kb, vb, n, 0, bits, s);
  if (e != cudaSuccess) return e;
  if (need > *temp_bytes) {
    if (*temp) cudaFree(*temp);
    *temp = nullptr;
    *temp_bytes = 0;
    if ((e = cudaMalloc(temp, need)) != cudaSuccess) return e;
    *temp_bytes = need;
  }
  e = cub::DeviceRadixSort::SortPairs(*temp, need, kb, vb, n, 0, bits, s);
  note_kernel(2);
  *perm = vb.Current();
  return e;
}

cudaError_t launch_tc_wedges(int lay, const Tables& t, const u32* oadj, const u32* oend,
                             const u32* perm, u64 n_units, unsigned long long* count, int sms,
                             cudaStream_t s) {
  if (n_units == 0) return cudaSuccess;
  const int G = lay & 31;
  u64 blocks = (n_units * G + 255) / 256;
  if (blocks > (u64)sms * 4) blocks = (u64)sms * 4;
  switch (lay) {
#define DG_CASE(G_, S_, A_)                                                                 \
  case DG_LAYA(G_, S_, A_):                                                                 \
    k_tc_wedges<G_, S_, A_><<<(unsigned)blocks, 256, 0, s>>>(t, oadj, oend, perm, n_units, count); \
    break;
    DG_FOR_LAYOUTS_A(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(1);
  return cudaGetLastError();
}

}  // namespace dg
