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
#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

__device__ __forceinline__ bool rank_less(u32 du, u32 u, u32 dv, u32 v) {
  return du < dv || (du == dv && u < v);
}

__global__ void __launch_bounds__(256) k_tc_orient_count(const u64* ro, const u32* dst,
                                                         const u32* deg, u64 rows, u32 part,
                                                         u32 nparts, u64* ocnt) {
  const u32 lane = threadIdx.x & 31;
  const u64 wid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nw = ((u64)gridDim.x * blockDim.x) >> 5;
  for (u64 u = wid; u < rows; u += nw) {
    u32 c = 0;
    if (u % nparts == part) {
      const u32 du = deg[u];
      for (u64 k = ro[u] + lane; k < ro[u + 1]; k += 32) {
        const u32 v = dst[k];
        c += rank_less(du, (u32)u, __ldg(&deg[v]), v) ? 1u : 0u;
      }
      c = __reduce_add_sync(0xFFFFFFFFu, c);
    }
    if (lane == 0) ocnt[u] = c;
  }
  if (blockIdx.x == 0 && threadIdx.x == 0) ocnt[rows] = 0;
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

template <int G>
__global__ void __launch_bounds__(256) k_tc_wedges(Tables t, const u32* __restrict__ oadj,
                                                   const u32* __restrict__ oend, u64 n_units,
                                                   unsigned long long* count) {
  constexpr int W = Group<G>::W;
  u32 hits = 0;
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 e = (u64)blockIdx.x * blockDim.x + threadIdx.x; e < n_units; e += stride) {
    const u32 v = oadj[e];
    const u32 end = oend[e];
    const uint2 dv = ld_nc_dir(t.dir + v);
    for (u32 k = (u32)e + 1; k < end; ++k) {
      const u32 w = __ldg(oadj + k);
      u32 b = dv.x + bucket_of(w, dv.y);
      while (true) {  // edgeExist(v, w): walk the chain of w's bucket in A_v
        const uint4* bp = reinterpret_cast<const uint4*>(t.pool + (u64)b * W);
        bool found = false, ended = false;
        u32 next = kNil;
#pragma unroll
        for (int c = 0; c < G; ++c) {
          const uint4 q = __ldg(bp + c);
          found |= q.x == w;
          ended |= q.x == kEmpty;
          if (c < G - 1) {
            found |= q.z == w;
            ended |= q.z == kEmpty;
          } else {
            next = q.z;
          }
        }
        if (found) {
          ++hits;
          break;
        }
        if (ended || next == kNil) break;
        b = next;
      }
    }
  }
  const u32 tot = __reduce_add_sync(0xFFFFFFFFu, hits);
  if ((threadIdx.x & 31) == 0 && tot) atomicAdd(count, (unsigned long long)tot);
}

cudaError_t launch_tc_orient_count(const Tables& t, const u64* ro, const u32* dst, u32 part,
                                   u32 nparts, u64* ocnt, int sms, cudaStream_t s) {
  k_tc_orient_count<<<(unsigned)sms * 8, 256, 0, s>>>(ro, dst, t.deg, t.rows, part, nparts, ocnt);
  note_kernel(1);
  return cudaGetLastError();
}

cudaError_t launch_tc_orient_fill(const Tables& t, const u64* ro, const u32* dst, u32 part,
                                  u32 nparts, const u64* oro, u32* oadj, u32* oend, int sms,
                                  cudaStream_t s) {
  k_tc_orient_fill<<<(unsigned)sms * 8, 256, 0, s>>>(ro, dst, t.deg, t.rows, part, nparts, oro, oadj,
                                                     oend);
  note_kernel(1);
  return cudaGetLastError();
}

cudaError_t launch_tc_wedges(int G, const Tables& t, const u32* oadj, const u32* oend, u64 n_units,
                             unsigned long long* count, int sms, cudaStream_t s) {
  if (n_units == 0) return cudaSuccess;
  u64 blocks = (n_units + 255) / 256;
  if (blocks > (u64)sms * 8) blocks = (u64)sms * 8;
  switch (G) {
    case 2: k_tc_wedges<2><<<(unsigned)blocks, 256, 0, s>>>(t, oadj, oend, n_units, count); break;
    case 4: k_tc_wedges<4><<<(unsigned)blocks, 256, 0, s>>>(t, oadj, oend, n_units, count); break;
    case 8: k_tc_wedges<8><<<(unsigned)blocks, 256, 0, s>>>(t, oadj, oend, n_units, count); break;
    default: return cudaErrorInvalidValue;
  }
  note_kernel(1);
  return cudaGetLastError();
}

}  // namespace dg
