// kernels_check.cu — structural invariants of the per-vertex hash tables (debug /
// test entry point dg_check_invariants; not on the hot path).
//
// What the lock-free insert's correctness rests on, checked directly in the table
// memory:
//   * EMPTY slots form a suffix of every chain ("empty locations can only
//     exist at the end of each bucket's list") — the probe's early stop and the
//     next-slot retry both depend on it;
//   * every live key sits in the chain its hash selects, bucket_of(v, nb);
//   * no live key repeats inside a chain (key uniqueness, fn3 P:L235-236);
//   * no self-loop (Alg1:L3) and no key >= the vertex capacity;
//   * every bucket's owner word is its row (the purge sweep reads it);
//   * degree[row] == live keys of the row;
//   * chains end (no cycle: a chain longer than the pool is reported broken).
// One warp per row, one lane per chain of the row (chains j = lane, lane + 32, ...);
// each lane walks its chain with scalar loads.
#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

namespace {

constexpr u32 kDupCheckMaxBuckets = 64;  // longer chains: duplicates not checked (counted)

__device__ __forceinline__ void bump(unsigned long long* c, unsigned long long v = 1) {
  if (v) atomicAdd(c, v);
}

template <int G, int S, bool A>
__global__ void __launch_bounds__(256) k_check(Tables t, u64 nv, u32 rank, InvariantsOut* out,
                                              u64 max_len) {
  typedef Lay<G, S> LY;
  typedef Geo<G, S, A> GEO;
  const u32 lane = threadIdx.x & 31u;
  const u64 warp = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nwarps = ((u64)gridDim.x * blockDim.x) >> 5;
  for (u64 row = warp; row < t.rows; row += nwarps) {
    const DirEntry de = t.dir[row];
    const u64 gid = row * t.nranks + rank;  // global vertex id of the row
    // uniform layouts: the probe's chain-count byte must agree with the directory
    if (!A && lane == 0 && t.nbs[row] != (de.nb < 255u ? de.nb : 255u))
      bump(&out->owner_mismatch);
    unsigned long long live = 0, tombs = 0, buckets = 0;
    bool bad = false;
    for (u32 j = lane; j < de.nb; j += 32) {
      u32 b = chain_head<A>(de.base, (u32)row, j);
      u64 len = 0;
      bool seen_empty = false, not_suffix = false;
      while (b != kNil) {
        if (++len > max_len) {
          bump(&out->broken_chains);
          bad = true;
          break;
        }
        const GEO gb(t, b);
        // (a home bucket's owner is its index: its last word is the row's degree)
        if (!gb.home && gb.p[gb.owner_word()] != (u32)row) {
          bump(&out->owner_mismatch);
          bad = true;
        }

        for (u32 uu = 0; uu < gb.units; ++uu) {
#pragma unroll
          for (int k = 0; k < LY::SPU; ++k) {
            if (!gb.has(uu, k)) continue;
            const u32 key = gb.p[LY::word(uu, k)];
            if (key == kEmpty) {
              seen_empty = true;
              continue;
            }
            if (seen_empty) not_suffix = true;
            if (key == kTomb) {
              ++tombs;
              continue;
            }
            ++live;
            if ((u64)key >= nv) { bump(&out->keys_out_of_range); bad = true; }
            if ((u64)key == gid) { bump(&out->self_loops); bad = true; }
            if (bucket_of(key, de.nb) != j) { bump(&out->misplaced_keys); bad = true; }
          }
        }
        ++buckets;
        b = gb.p[gb.next_word()];
      }
      if (not_suffix) {
        bump(&out->empty_not_suffix);
        bad = true;
      }
      // duplicates inside the chain: every live key against every later slot
      if (len > kDupCheckMaxBuckets) {
        bump(&out->dup_unchecked_chains);
        continue;
      }
      for (u32 b1 = chain_head<A>(de.base, (u32)row, j); b1 != kNil;) {
        const GEO g1(t, b1);
        for (u32 uu = 0; uu < g1.units; ++uu) {
          for (int k = 0; k < LY::SPU; ++k) {
            if (!g1.has(uu, k)) continue;
            const u32 key = g1.p[LY::word(uu, k)];
            if (key >= kTomb) continue;
            // later slots of this bucket, then the later buckets
            bool first = true;
            for (u32 b2 = b1; b2 != kNil;) {
              const GEO g2(t, b2);
              for (u32 u2 = 0; u2 < g2.units; ++u2) {
                for (int k2 = 0; k2 < LY::SPU; ++k2) {
                  if (!g2.has(u2, k2)) continue;
                  if (first && (u2 < uu || (u2 == uu && k2 <= k))) continue;
                  if (g2.p[LY::word(u2, k2)] == key) { bump(&out->duplicate_keys); bad = true; }
                }
              }
              first = false;
              b2 = g2.p[g2.next_word()];
            }
          }
        }
        b1 = g1.p[g1.next_word()];
      }
    }
    // per-row totals (warp reduction)
    for (int o = 16; o; o >>= 1) {
      live += __shfl_xor_sync(0xFFFFFFFFu, live, o);
      tombs += __shfl_xor_sync(0xFFFFFFFFu, tombs, o);
      buckets += __shfl_xor_sync(0xFFFFFFFFu, buckets, o);
    }
    bad = __any_sync(0xFFFFFFFFu, bad);
    if (lane == 0) {
      if (live != *deg_at(t, row)) {
        bump(&out->degree_mismatch);
        bad = true;
      }
      bump(&out->live_pairs, live);
      bump(&out->tombstones, tombs);
      bump(&out->buckets, buckets);
      bump(&out->chains, de.nb);
      bump(&out->rows);
      if (bad) atomicMin(&out->first_bad_row, (unsigned long long)row);
    }
  }
}

}  // namespace

cudaError_t launch_check(int lay, const Tables& t, u64 nv, u32 rank, InvariantsOut* out, int sms,
                         cudaStream_t s) {
  cudaError_t e = cudaMemsetAsync(out, 0, sizeof(InvariantsOut), s);
  if (e != cudaSuccess) return e;
  e = cudaMemsetAsync(&out->first_bad_row, 0xFF, 8, s);
  if (e != cudaSuccess || t.rows == 0) return e;
  u64 blocks = (t.rows * 32 + 255) / 256;
  if (blocks > (u64)sms * 16) blocks = (u64)sms * 16;
  u64 max_len = 0;  // a chain longer than every pool together is a cycle
  for (int c = 0; c < kClasses; ++c) max_len += t.cap[c];
  max_len += 1;
  switch (lay) {
#define DG_CASE(G_, S_, A_)                                                                   \
  case DG_LAYA(G_, S_, A_):                                                                   \
    k_check<G_, S_, A_><<<(unsigned)blocks, 256, 0, s>>>(t, nv, rank, out, max_len);          \
    break;
    DG_FOR_LAYOUTS_A(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
  note_kernel(1);
  return cudaGetLastError();
}

}  // namespace dg
