// kernels_edges.cu — batched edge insert / delete / query (the hot path).
//
// Method (§IV-B..C): each op (u, v[, w]) locates A_u through the vertex
// dictionary (Alg1:L8 `graph[current_src]`), hashes v to a bucket of A_u and walks
// that bucket's chain.  Insert = key-unique "replace":
// overwrite the value of an existing key, else install the pair in the first
// EMPTY slot, linking a new bucket at the tail when the chain is full
// (P:L414-418).  Delete = overwrite the key with a tombstone.
// Tombstones are skipped, never reused, so EMPTY slots only exist at the tail of
// a chain and every probe stops at the first EMPTY.
//
// B200 execution design (differs from the paper's one-op-per-warp
// WCWS):
//   * a warp stages 32 consecutive ops of the batch with one coalesced load per
//     input array;
//   * every lane loads the directory entry of ITS op and issues an L2 prefetch of
//     the op's first bucket, so 32 directory gathers and 32 bucket gathers per
//     warp are in flight at once (memory-level parallelism is the bound);
//   * a "group" of G = bucket_bytes/16 lanes then probes the G ops of its lanes one
//     after another, each lane holding 16 B of the bucket (one 128-B bucket = one
//     coalesced request of 8 lanes); 32/G groups per warp probe independently;
//   * a new pair is installed with one 64-bit CAS on (key, value); a deletion is a
//     32-bit CAS key -> tombstone, so exactly one of several racing deleters wins
//     and degrees stay exact (Alg1:L9-10);
//   * degree updates are one fire-and-forget atomic per added/removed key; batch
//     counters are reduced per warp.
#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

enum { OP_INSERT = 0, OP_DELETE = 1, OP_QUERY = 2 };

// ----------------------------------------------------------- allocator (a8) ----
// Phase-concurrent free stack + bump cursor: during an insert
// phase buckets are only popped, during a vertex-deletion phase only pushed, so
// a single cursor per direction is ABA-free.
__device__ __forceinline__ u32 alloc_bucket(const Tables& t, u32 stack_size) {
  u32 i = atomicAdd(&t.ctl->pop_count, 1u);
  if (i < stack_size) return t.stack[stack_size - 1 - i];
  u32 j = atomicAdd(&t.ctl->bump, 1u);
  return j < t.cap ? j : kNil;
}

// ------------------------------------------------------------ probe: insert ----
// returns 1 = key added, 0 = existing key replaced, -1 = no bucket available
template <int G>
__device__ __forceinline__ int probe_insert(const Tables& t, const Group<G>& g, u32 row, u32 b,
                                            u32 v, u32 w, u32& spare, u32 stack_size) {
  constexpr int W = Group<G>::W;
  while (true) {
    u32* bp = t.pool + (u64)b * W;
    const uint4 q = ld_relaxed_v4(bp + 4 * g.gl);
    const bool lastl = g.last();
    const bool m0 = q.x == v, m1 = !lastl && q.z == v;
    const u32 hit = g.ballot(m0 || m1);
    if (hit) {  // replace: key exists
      const u32 l = __ffs(hit) - 1;
      if (g.gl == l) st_relaxed_u32(bp + 4 * g.gl + (m0 ? 1 : 3), w);
      return 0;
    }
    const bool e0 = q.x == kEmpty, e1 = !lastl && q.z == kEmpty;
    const u32 em = g.ballot(e0 || e1);
    if (em) {  // first EMPTY slot of the chain: install (v, w)
      const u32 l = __ffs(em) - 1;
      const u32 woff = 4 * g.gl + (e0 ? 0 : 2);
      unsigned long long old = 0;
      if (g.gl == l)
        old = atomicCAS(reinterpret_cast<unsigned long long*>(bp + woff), kEmptyPair,
                        (unsigned long long)pack_pair(v, w));
      old = g.shfl(old, l);
      if (old == kEmptyPair) return 1;
      if ((u32)old == v) {  // a racing op installed the same key: replace
        if (g.gl == l) st_relaxed_u32(bp + woff + 1, w);
        return 0;
      }
      continue;  // slot taken by another key: re-read this bucket
    }
    const u32 next = g.shfl(q.z, G - 1);
    if (next != kNil) {
      b = next;
      continue;
    }
    // chain full: link a new bucket at the tail
    if (spare == kNil) {
      u32 s = 0;
      if (g.gl == 0) s = alloc_bucket(t, stack_size);
      spare = g.shfl(s, 0);
      if (spare == kNil) return -1;
    }
    u32 old = 0;
    if (lastl) {
      st_relaxed_u32(t.pool + (u64)spare * W + Group<G>::OWNER, row);
      old = atomicCAS(bp + Group<G>::NEXT, kNil, spare);
    }
    old = g.shfl(old, G - 1);
    if (old == kNil) {
      b = spare;
      spare = kNil;
    } else {
      b = old;  // another op linked first; keep our spare for later
    }
  }
}

// ------------------------------------------------------------ probe: delete ----
template <int G>
__device__ __forceinline__ int probe_delete(const Tables& t, const Group<G>& g, u32 b, u32 v) {
  constexpr int W = Group<G>::W;
  while (true) {
    u32* bp = t.pool + (u64)b * W;
    const uint4 q = ld_relaxed_v4(bp + 4 * g.gl);
    const bool lastl = g.last();
    const bool m0 = q.x == v, m1 = !lastl && q.z == v;
    const u32 hit = g.ballot(m0 || m1);
    if (hit) {
      const u32 l = __ffs(hit) - 1;
      u32 old = 0;
      if (g.gl == l) old = atomicCAS(bp + 4 * g.gl + (m0 ? 0 : 2), v, kTomb);
      return g.shfl(old, l) == v ? 1 : 0;
    }
    const bool e0 = q.x == kEmpty, e1 = !lastl && q.z == kEmpty;
    if (g.ballot(e0 || e1)) return 0;
    const u32 next = g.shfl(q.z, G - 1);
    if (next == kNil) return 0;
    b = next;
  }
}

// ------------------------------------------------------------- probe: query ----
template <int G>
__device__ __forceinline__ bool probe_query(const Tables& t, const Group<G>& g, u32 b, u32 v,
                                            u32& val) {
  constexpr int W = Group<G>::W;
  while (true) {
    const u32* bp = t.pool + (u64)b * W;
    const uint4 q = ld_nc_v4(bp + 4 * g.gl);
    const bool lastl = g.last();
    const bool m0 = q.x == v, m1 = !lastl && q.z == v;
    const u32 hit = g.ballot(m0 || m1);
    if (hit) {
      const u32 l = __ffs(hit) - 1;
      val = g.shfl(m0 ? q.y : q.w, l);
      return true;
    }
    const bool e0 = q.x == kEmpty, e1 = !lastl && q.z == kEmpty;
    if (g.ballot(e0 || e1)) return false;
    const u32 next = g.shfl(q.z, G - 1);
    if (next == kNil) return false;
    b = next;
  }
}

// ------------------------------------------------------------- main kernel ----
template <int G, int OP>
__global__ void __launch_bounds__(kEdgeBlock) k_edges(Tables t, EdgeBatch a) {
  const Group<G> g;
  if (OP != OP_QUERY) {
    if (ld_relaxed_u32(&t.ctl->fail_epoch) == a.epoch) return;  // batch rejected (Q7)
  }
  const u32 stack_size = (OP == OP_INSERT) ? ld_relaxed_u32(&t.ctl->stack_size) : 0u;
  const u64 warp = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nwarps = ((u64)gridDim.x * blockDim.x) >> 5;
  u64 my_count = 0;
  u32 spare = kNil;
  bool bad_range = false;

  for (u64 chunk = warp; chunk * 32 < a.n_ops; chunk += nwarps) {
    // ---- stage 32 ops of the batch (coalesced), one per lane
    const u64 j = chunk * 32 + g.lane;
    const bool valid = j < a.n_ops;
    u64 opid = j;
    u32 u = 0, v = 0, w = 0;
    if (valid) {
      if (a.idx) opid = a.idx[j];
      u64 i = opid;
      const bool rev = opid >= a.n;  // undirected mirror op
      if (rev) i = opid - a.n;
      u = a.src[i];
      v = a.dst[i];
      if (OP == OP_INSERT && a.w) w = a.w[i];
      if (rev) { const u32 x = u; u = v; v = x; }
    }
    bool active = valid && u != v;  // self-loops are never stored (Alg1:L3)
    if (OP == OP_QUERY && valid && ((u64)u >= a.nv || (u64)v >= a.nv)) {
      active = false;
      bad_range = true;
    }
    const u32 row = (t.nranks == 1) ? u : u / t.nranks;
    // ---- every lane gathers its op's directory entry and prefetches its bucket
    u32 bkt = 0;
    if (active) {
      // base/nb never change during an edge phase; only deg is written (atomics)
      const uint4 de = (OP == OP_QUERY) ? ld_nc_dir(t.dir + row) : ld_dir(t.dir + row);
      bkt = de.x + bucket_of(v, de.y);
      prefetch_l2(t.pool + (u64)bkt * Group<G>::W);
    }
    // ---- each group probes the G ops held by its lanes, one after another
    u32 res = 0, resw = 0;
#pragma unroll 1
    for (int r = 0; r < G; ++r) {
      if (!g.shfl((int)active, r)) continue;
      const u32 rv = g.shfl(v, r);
      const u32 rb = g.shfl(bkt, r);
      const u32 rrow = g.shfl(row, r);
      if (OP == OP_INSERT) {
        const u32 rw = g.shfl(w, r);
        const u64 ropid = g.shfl(opid, r);
        const int s = probe_insert<G>(t, g, rrow, rb, rv, rw, spare, stack_size);
        if (g.gl == 0) {
          if (s == 1) {
            atomicAdd(&t.dir[rrow].deg, 1u);
            ++my_count;
          } else if (s < 0) {
            a.retry_out[atomicAdd(&t.ctl->retry_count, 1u)] = ropid;
          }
        }
      } else if (OP == OP_DELETE) {
        const int s = probe_delete<G>(t, g, rb, rv);
        if (s && g.gl == 0) {
          atomicSub(&t.dir[rrow].deg, 1u);
          ++my_count;
        }
      } else {
        u32 val = 0;
        const bool f = probe_query<G>(t, g, rb, rv, val);
        if (g.gl == (u32)r) {
          res = f ? 1u : 0u;
          resw = f ? val : 0u;
        }
      }
    }
    if (OP == OP_QUERY && valid) {
      a.found[j] = (uint8_t)res;
      if (a.wout) a.wout[j] = resw;
    }
  }
  // ---- epilogue: hand back an unused spare bucket, reduce the batch counter
  if (OP == OP_INSERT && spare != kNil && g.gl == 0)
    t.ret_list[atomicAdd(&t.ctl->ret_count, 1u)] = spare;
  if (OP == OP_QUERY) {
    if (__any_sync(0xFFFFFFFFu, bad_range) && g.lane == 0)
      atomicMax(&t.ctl->fail_epoch, a.epoch);
  } else {
    const u64 tot = __reduce_add_sync(0xFFFFFFFFu, (u32)my_count);
    if (g.lane == 0 && tot) atomicAdd(reinterpret_cast<unsigned long long*>(&t.ctl->count), tot);
  }
}

// ---------------------------------------------------------------- helpers ----
// Validation (Q7) for mutating batches: any endpoint >= capacity rejects the
// batch; also resets the per-batch counters (they are only written by kernels
// that run after this one on the stream).
__global__ void k_validate(const u32* __restrict__ src, const u32* __restrict__ dst, u64 n,
                           u64 nv, u32 epoch, DevCtl* ctl) {
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    ctl->count = 0;
    ctl->retry_count = 0;
  }
  bool bad = false;
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 i = (u64)blockIdx.x * blockDim.x + threadIdx.x; i < n; i += stride)
    bad |= ((u64)src[i] >= nv) | ((u64)dst[i] >= nv);
  if (__any_sync(0xFFFFFFFFu, bad) && (threadIdx.x & 31) == 0) atomicMax(&ctl->fail_epoch, epoch);
}

// After an insert phase: drop the popped entries from the free stack, clamp the
// bump cursor, and push the spare buckets that were handed back.
__global__ void k_fixup_alloc(Tables t) {
  __shared__ u32 s_ss, s_rc;
  DevCtl* c = t.ctl;
  if (threadIdx.x == 0) {
    const u32 pc = c->pop_count, ss = c->stack_size;
    s_ss = pc >= ss ? 0u : ss - pc;
    s_rc = c->ret_count;
    if (c->bump > t.cap) c->bump = t.cap;
  }
  __syncthreads();
  for (u32 k = threadIdx.x; k < s_rc; k += blockDim.x) t.stack[s_ss + k] = t.ret_list[k];
  __syncthreads();
  if (threadIdx.x == 0) {
    c->stack_size = s_ss + s_rc;
    c->pop_count = 0;
    c->ret_count = 0;
  }
}

// ---------------------------------------------------------------- launchers ----
template <int G, int OP>
static int grid_for() {
  static int blocks_per_sm = -1;
  if (blocks_per_sm < 0) {
    int b = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, k_edges<G, OP>, kEdgeBlock, 0) !=
            cudaSuccess || b <= 0)
      b = 1;
    blocks_per_sm = b;
  }
  return blocks_per_sm;
}

template <int G, int OP>
static cudaError_t launch_g(const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  if (a.n_ops == 0) return cudaSuccess;
  const u64 warps_needed = (a.n_ops + 31) / 32;
  const u64 per_block = kEdgeBlock / 32;
  u64 blocks = (warps_needed + per_block - 1) / per_block;
  const u64 maxb = (u64)sms * grid_for<G, OP>();
  if (blocks > maxb) blocks = maxb;
  k_edges<G, OP><<<(unsigned)blocks, kEdgeBlock, 0, s>>>(t, a);
  return cudaGetLastError();
}

template <int OP>
static cudaError_t launch_op(int G, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  switch (G) {
    case 2: return launch_g<2, OP>(t, a, sms, s);
    case 4: return launch_g<4, OP>(t, a, sms, s);
    case 8: return launch_g<8, OP>(t, a, sms, s);
    default: return cudaErrorInvalidValue;
  }
}

cudaError_t launch_insert(int G, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  return launch_op<OP_INSERT>(G, t, a, sms, s);
}
cudaError_t launch_delete(int G, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  return launch_op<OP_DELETE>(G, t, a, sms, s);
}
cudaError_t launch_query(int G, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  return launch_op<OP_QUERY>(G, t, a, sms, s);
}

u64 max_groups(int G, int sms) {
  // upper bound on groups resident in one launch (bounds the spare-return list)
  return (u64)sms * 2048 / (u64)G;
}

cudaError_t launch_validate(const u32* src, const u32* dst, u64 n, u64 nv, u32 epoch, DevCtl* ctl,
                            int sms, cudaStream_t s) {
  u64 blocks = (n + 255) / 256;
  if (blocks > (u64)sms * 8) blocks = (u64)sms * 8;
  if (blocks == 0) blocks = 1;
  k_validate<<<(unsigned)blocks, 256, 0, s>>>(src, dst, n, nv, epoch, ctl);
  return cudaGetLastError();
}

cudaError_t launch_fixup_alloc(const Tables& t, cudaStream_t s) {
  k_fixup_alloc<<<1, 256, 0, s>>>(t);
  return cudaGetLastError();
}

}  // namespace dg
