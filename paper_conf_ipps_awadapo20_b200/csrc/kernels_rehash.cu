// kernels_rehash.cu — per-vertex table re-sizing (P:L309-313:
// "maintain low-cost metrics per vertex to determine the chain-length and
// periodically perform rehashing if it exceeds a given threshold").
//
// An insert that walks more than `hot_steps` chained buckets flags its row
// (k_edges).  Before the next insert batch the host re-sizes the flagged rows:
//   k_hot_sizes    : new #base buckets = max(nb+1, ceil(2*deg / (lf*Bc))), old nb, deg
//                    (degree-adaptive layout: the size class is chosen again for 2*deg,
//                    so a growing row moves up to larger buckets)
//   k_hot_export   : live pairs of the flagged tables -> (src, dst, w) lists
//   k_hot_release  : every bucket of the old tables (base and chained) reset to
//                    EMPTY and pushed on the free stack
//   k_init_rows    : new directory entries over a fresh consecutive base range
// and the exported pairs are inserted again with the ordinary insert kernel.  The
// logical graph is unchanged (same keys, same values, exact degrees); only chain
// lengths (and any tombstones of those rows) go away.
#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

__global__ void k_hot_sizes(Tables t, u32 n, u32 lf_milli, u32 bc, u32 flush, u32 adaptive,
                            u32 set, u64* nbnew, u64* nbold, u64* degs) {
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 k = (u64)blockIdx.x * blockDim.x + threadIdx.x; k <= n; k += stride) {
    if (k == n) {
      nbnew[k] = nbold[k] = degs[k] = 0;
      continue;
    }
    const u32 row = t.hot_list[k];
    const DirEntry de = t.dir[row];
    const u64 d = *deg_at(t, row);
    if (adaptive) {  // size class and #buckets by the initial rule (k_initial_buckets)
      u64 v = class_size(flush ? d : 2 * d, lf_milli, set);
      const u32 oc = de.base >> kClassShift;
      if (!flush && (u32)(v >> 40) == oc && (v & kNbMask) < (u64)de.nb + 1)
        v = ((u64)oc << 40) | ((u64)de.nb + 1);
      nbnew[k] = v;
      nbold[k] = de.nb;
      degs[k] = d;
      continue;
    }
    const u64 den = (u64)lf_milli * bc;
    u64 want;
    if (flush) {  // tombstone flush: the initial-size rule for the live keys
      want = d ? (d * 1000 + den - 1) / den : 1;
    } else {      // re-size: room to double before chaining again
      want = (2 * d * 1000 + den - 1) / den;
      if (want < (u64)de.nb + 1) want = (u64)de.nb + 1;
    }
    nbnew[k] = want;
    nbold[k] = de.nb;
    degs[k] = d;
  }
}

// largest k < cnt with off[k] <= x
__device__ __forceinline__ u32 seg_of(const u64* off, u32 cnt, u64 x) {
  u32 lo = 0, hi = cnt;
  while (hi - lo > 1) {
    const u32 mid = (lo + hi) >> 1;
    if (off[mid] <= x) lo = mid;
    else hi = mid;
  }
  return lo;
}

// one group per (flagged row, old base bucket): walk the chain, append live pairs
template <int G, int S, bool A>
__global__ void __launch_bounds__(256) k_hot_export(Tables t, u32 n, const u64* obo,
                                                    unsigned long long* cursor, u32* osrc,
                                                    u32* odst, u32* ow, u32 rank) {
  typedef Lay<G, S> LY;
  const Group<G> g;
  const u64 total = obo[n];
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  const u32 below = (1u << g.gl) - 1u;
  for (u64 x = gid; x < total; x += ng) {
    const u32 k = seg_of(obo, n, x);
    const u32 row = t.hot_list[k];
    const u32 gid_u = row * t.nranks + rank;  // global source id
    u32 b = chain_head<A>(t.dir[row].base, row, (u32)(x - obo[k]));
    while (b != kNil) {
      const Geo<G, S, A> gb(t, b);
      const uint4 q = (A && g.gl >= gb.units) ? make_uint4(kEmpty, kEmpty, kEmpty, kEmpty)
                                              : ld_relaxed_v4(gb.p + 4 * g.gl);
      u32 before = 0, cnt = 0;
#pragma unroll
      for (int j = 0; j < LY::SPU; ++j) {
        const u32 m = g.ballot(gb.has(g.gl, j) && LY::key(q, j) < kTomb);
        before += __popc(m & below);
        cnt += __popc(m);
      }
      unsigned long long pos = 0;
      if (g.gl == 0 && cnt) pos = atomicAdd(cursor + k, (unsigned long long)cnt);
      u64 at = g.shfl(pos, 0) + before;
#pragma unroll
      for (int j = 0; j < LY::SPU; ++j) {
        if (gb.has(g.gl, j) && LY::key(q, j) < kTomb) {
          osrc[at] = gid_u;
          odst[at] = LY::key(q, j);
          ow[at] = LY::val(q, j);
          ++at;
        }
      }
      b = g.shfl(q.z, gb.units - 1);
    }
  }
}

// every bucket of the old tables -> EMPTY, onto the free stack (base ones too: the
// row moves to a new base range); a home bucket stays the row's (emptied here)
template <int G, bool A>
__global__ void __launch_bounds__(256) k_hot_release(Tables t, u32 n, const u64* obo) {
  const Group<G> g;
  const u64 total = obo[n];
  const uint4 empty4 = make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  for (u64 x = gid; x < total; x += ng) {
    const u32 k = seg_of(obo, n, x);
    const u32 row = t.hot_list[k];
    u32 b = chain_head<A>(t.dir[row].base, row, (u32)(x - obo[k]));
    while (b != kNil) {
      const Geo<G, 0, A> gb(t, b);
      const bool in = !A || g.gl < gb.units;
      u32* bp = gb.p + 4 * g.gl;
      const uint4 q = in ? ld_relaxed_v4(bp) : empty4;
      const u32 next = g.shfl(q.z, gb.units - 1);
      if (in) st_v4(bp, empty4);
      if (g.gl == 0 && !gb.home) {
        const u32 c = b >> kClassShift;
        by_class(t.stack, c)[atomicAdd(&t.ctl->stack_size[c], 1u)] = b;
      }
      b = next;
    }
  }
}

// Tombstone flush ("Tombstones can later be completely flushed out of
// the data structure"): one streaming pass over every allocated bucket; a bucket
// holding a tombstone flags its owner row (bucket word W-1) for a compacting
// re-build (the rows are then re-sized with flush = 1).
// (H: the home pool of a uniform layout)
template <int G, int S, bool H = false>
__global__ void __launch_bounds__(256) k_tomb_sweep(Tables t, u32 cls) {
  typedef Lay<G, S> LY;
  const Group<G> g;
  const u32 nbk = H ? (u32)t.rows : ld_relaxed_u32(&t.ctl->bump[cls]);
  const u32* const pool = H ? t.home : by_class(t.pool, cls);
  const u64 gid = ((u64)blockIdx.x * blockDim.x + threadIdx.x) / G;
  const u64 ng = ((u64)gridDim.x * blockDim.x) / G;
  for (u64 b = gid; b < nbk; b += ng) {
    const uint4 x = *reinterpret_cast<const uint4*>(pool + b * LY::W + 4 * g.gl);
    bool tomb = false;
#pragma unroll
    for (int j = 0; j < LY::SPU; ++j) tomb |= LY::has(g.gl, j) && LY::key(x, j) == kTomb;
    const u32 owner = H ? (u32)b : g.shfl(x.w, G - 1);  // (home: word W-1 = degree)
    if (g.ballot(tomb) && g.gl == 0) {
      const u32 bit = 1u << (owner & 31);
      if (!(atomicOr(&t.hot_flags[owner >> 5], bit) & bit)) {
        const u32 k = atomicAdd(&t.ctl->hot_count, 1u);
        if (k < t.hot_cap) t.hot_list[k] = owner;
      }
    }
  }
}

cudaError_t launch_tomb_sweep(int lay, const Tables& t, int sms, cudaStream_t s) {
  const unsigned blocks = (unsigned)sms * 8;
  if (lay & DG_ADAPTIVE_BIT) {  // one sweep per size class pool
    if (lay & 32) {
      k_tomb_sweep<2, 1><<<blocks, 256, 0, s>>>(t, 0);
      k_tomb_sweep<4, 1><<<blocks, 256, 0, s>>>(t, 1);
      k_tomb_sweep<8, 1><<<blocks, 256, 0, s>>>(t, 2);
    } else {
      k_tomb_sweep<2, 0><<<blocks, 256, 0, s>>>(t, 0);
      k_tomb_sweep<4, 0><<<blocks, 256, 0, s>>>(t, 1);
      k_tomb_sweep<8, 0><<<blocks, 256, 0, s>>>(t, 2);
    }
    note_kernel(3);
    return cudaGetLastError();
  }
  switch (lay) {
#define DG_CASE(G_, S_)                                       \
  case DG_LAY(G_, S_):                                        \
    k_tomb_sweep<G_, S_><<<blocks, 256, 0, s>>>(t, 0);        \
    k_tomb_sweep<G_, S_, true><<<blocks, 256, 0, s>>>(t, 0);  \
    break;
    DG_FOR_LAYOUTS(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(2);
  return cudaGetLastError();
}

cudaError_t launch_hot_sizes(const Tables& t, u32 n, u32 lf_milli, u32 bc, u32 flush, u32 adaptive,
                             u32 set, u64* nbnew, u64* nbold, u64* degs, cudaStream_t s) {
  const unsigned blocks = (n + 256) / 256;
  k_hot_sizes<<<blocks, 256, 0, s>>>(t, n, lf_milli, bc, flush, adaptive, set, nbnew, nbold, degs);
  note_kernel(1);
  return cudaGetLastError();
}

cudaError_t launch_hot_export(int lay, const Tables& t, u32 n, const u64* obo,
                              unsigned long long* cursor, u32* osrc, u32* odst, u32* ow, u32 rank,
                              int sms, cudaStream_t s) {
  const unsigned blocks = (unsigned)sms * 8;
  switch (lay) {
#define DG_CASE(G_, S_, A_)                                                                \
  case DG_LAYA(G_, S_, A_):                                                                \
    k_hot_export<G_, S_, A_><<<blocks, 256, 0, s>>>(t, n, obo, cursor, osrc, odst, ow, rank); \
    break;
    DG_FOR_LAYOUTS_A(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(1);
  return cudaGetLastError();
}

cudaError_t launch_hot_release(int lay, const Tables& t, u32 n, const u64* obo, int sms,
                               cudaStream_t s) {
  const unsigned blocks = (unsigned)sms * 8;
  if (lay & DG_ADAPTIVE_BIT) {
    k_hot_release<8, true><<<blocks, 256, 0, s>>>(t, n, obo);
    note_kernel(1);
    return cudaGetLastError();
  }
  switch (lay & 31) {
    case 2: k_hot_release<2, false><<<blocks, 256, 0, s>>>(t, n, obo); break;
    case 4: k_hot_release<4, false><<<blocks, 256, 0, s>>>(t, n, obo); break;
    case 8: k_hot_release<8, false><<<blocks, 256, 0, s>>>(t, n, obo); break;
    default: return cudaErrorInvalidValue;
  }
  note_kernel(1);
  return cudaGetLastError();
}

}  // namespace dg
