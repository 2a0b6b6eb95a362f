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
#include <atomic>

#include "dg_common.cuh"
#include "kernels.h"

namespace dg {

static std::atomic<unsigned long long> g_launches{0};
void note_kernel(int n) { g_launches.fetch_add((unsigned long long)n, std::memory_order_relaxed); }
uint64_t kernel_launches() { return g_launches.load(std::memory_order_relaxed); }

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
// Full chain walk from the head bucket b (slow path; the fast path in k_edges
// handles single-bucket chains).  The key must be absent from the whole chain
// before it is installed (uniqueness); it is installed with
// a 64-bit CAS in the FIRST free slot of the chain: the first tombstone when
// tombstones are reused (the paper's two-stage option), else the
// first EMPTY.  Any failed slot CAS re-scans the chain from the head:
// two inserts of one key then always contend for the same slot.
// returns 1 = key added, 0 = existing key replaced, -1 = no bucket available
template <int G>
__device__ __forceinline__ int probe_insert(const Tables& t, const Group<G>& g, u32 row,
                                            const u32 head, u32 v, u32 w, u32& spare,
                                            u32 stack_size, bool reuse) {
  constexpr int W = Group<G>::W;
  u32 b = head;
  u32* ff = nullptr;         // first free slot seen (pair address), group-uniform
  unsigned long long ffo = 0;  // its current contents
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
    if (!ff) {
      const bool f0 = e0 || (reuse && q.x == kTomb);
      const bool f1 = e1 || (reuse && !lastl && q.z == kTomb);
      const u32 fm = g.ballot(f0 || f1);
      if (fm) {
        const u32 l = __ffs(fm) - 1;
        const u64 addr = (u64)(bp + 4 * g.gl + (f0 ? 0 : 2));
        const unsigned long long cur = f0 ? pack_pair(q.x, q.y) : pack_pair(q.z, q.w);
        ff = reinterpret_cast<u32*>(g.shfl(addr, l));
        ffo = g.shfl(cur, l);
      }
    }
    const u32 next = g.shfl(q.z, G - 1);
    if (em || next == kNil) {
      // end of the chain: the key is absent
      if (ff) {
        unsigned long long old = 0;
        if (g.gl == 0)
          old = atomicCAS(reinterpret_cast<unsigned long long*>(ff), ffo,
                          (unsigned long long)pack_pair(v, w));
        old = g.shfl(old, 0);
        if (old == ffo) return 1;
        if ((u32)old == v) {  // a racing op installed the same key there: replace
          if (g.gl == 0) st_relaxed_u32(ff + 1, w);
          return 0;
        }
        ff = nullptr;  // slot taken by another key: re-scan from the head
        b = head;
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
        b = old;  // another op linked first (earlier slots cannot free up); keep our spare
      }
      continue;
    }
    b = next;
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
// Per warp iteration (32 ops):
//   1. lane L stages op L (coalesced) and gathers its directory entry;
//   2. each group of G lanes loads the head buckets of its G ops back to back
//      (G independent 128-bit loads per lane: G*32/G = 32 buckets in flight per warp);
//   3. with group ballots it decides every op whose chain is a single bucket (the
//      common case at the paper's load factor): hit/miss for queries, the slot to
//      tombstone for deletes, replace-or-install slot for inserts;
//   4. every lane issues the CAS of its own op — one warp-wide atomic instruction;
//   5. ops with longer chains or lost CASes take the sequential chain walk.
enum { ST_DONE = 0, ST_CAS = 1, ST_SLOW = 2 };

template <int G, int OP>
__global__ void __launch_bounds__(kEdgeBlock, 4) k_edges(Tables t, EdgeBatch a) {
  constexpr int W = Group<G>::W;
  const Group<G> g;
  if (OP != OP_QUERY) {
    if (ld_relaxed_u32(&t.ctl->fail_epoch) == a.epoch) return;  // batch rejected (Q7)
  }
  const u32 stack_size = (OP == OP_INSERT) ? ld_relaxed_u32(&t.ctl->stack_size) : 0u;
  const bool reuse = a.reuse_tombstones != 0;
  const u64 warp = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nwarps = ((u64)gridDim.x * blockDim.x) >> 5;
  u32 my_count = 0;
  u32 spare = kNil;
  bool bad_range = false;

  for (u64 chunk = warp; chunk * 32 < a.n_ops; chunk += nwarps) {
    // ---- 1. stage one op per lane
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
    u32 head = 0;
    if (active) {
      // base/nb never change during an edge phase; only deg is written (atomics)
      const uint4 de = (OP == OP_QUERY) ? ld_nc_dir(t.dir + row) : ld_dir(t.dir + row);
      head = de.x + bucket_of(v, de.y);
    }
    // ---- 2. head buckets of the group's G ops, all loads in flight together.
    // The fast path (2-4) is branch-free across groups: every warp intrinsic uses
    // the full mask and each lane reads from the lanes of its own group.
    constexpr u32 FULL = 0xFFFFFFFFu;
    constexpr u32 GBITS = (G == 32) ? 0xFFFFFFFFu : ((1u << G) - 1u);
    const u32 amask = __ballot_sync(FULL, active);
    uint4 q[G];
#pragma unroll
    for (int r = 0; r < G; ++r) {
      const u32 hr = __shfl_sync(FULL, head, g.base + r);
      const u32* p = t.pool + (u64)hr * W + 4 * g.gl;
      if ((amask >> (g.base + r)) & 1u) q[r] = (OP == OP_QUERY) ? ld_nc_v4(p) : ld_relaxed_v4(p);
      else q[r] = make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
    }
    // ---- 3. decide single-bucket chains
    u32 state = ST_DONE;
    u32 res_val = 0;                 // query: value; found in res_found
    bool res_found = false;
    u32* cas_addr = nullptr;
    unsigned long long cas_old = 0;
    const bool lastl = g.last();
#pragma unroll
    for (int r = 0; r < G; ++r) {
      const uint4 x = q[r];
      const u32 srcl = g.base + r;
      const bool ar = (amask >> srcl) & 1u;
      const u32 vr = __shfl_sync(FULL, v, srcl);
      const u32 hr = __shfl_sync(FULL, head, srcl);
      u32* bp = t.pool + (u64)hr * W + 4 * g.gl;
      const bool m0 = ar && x.x == vr, m1 = ar && !lastl && x.z == vr;
      const u32 hit = (__ballot_sync(FULL, m0 || m1) >> g.base) & GBITS;
      const bool e0 = x.x == kEmpty, e1 = !lastl && x.z == kEmpty;
      const u32 em = (__ballot_sync(FULL, e0 || e1) >> g.base) & GBITS;
      const u32 next = __shfl_sync(FULL, x.z, g.base + G - 1);
      const bool whole = em != 0 || next == kNil;  // the head bucket is the whole chain
      const u32 lh = hit ? __ffs(hit) - 1 : 0;
      const bool mine = g.gl == (u32)r;
      if (OP == OP_QUERY) {
        const u32 val = __shfl_sync(FULL, m0 ? x.y : x.w, g.base + lh);
        if (mine && ar) {
          res_found = hit != 0;
          res_val = val;
          if (!hit && !whole) state = ST_SLOW;
        }
      } else if (OP == OP_DELETE) {
        const u64 ka = __shfl_sync(FULL, (unsigned long long)(bp + (m0 ? 0 : 2)), g.base + lh);
        if (mine && ar) {
          if (hit) { state = ST_CAS; cas_addr = reinterpret_cast<u32*>(ka); }
          else if (!whole) state = ST_SLOW;
        }
      } else {  // insert
        const u32 wr = __shfl_sync(FULL, w, srcl);
        if (hit && g.gl == lh) st_relaxed_u32(bp + (m0 ? 1 : 3), wr);  // replace
        const bool f0 = e0 || (reuse && x.x == kTomb);
        const bool f1 = e1 || (reuse && !lastl && x.z == kTomb);
        const u32 fm = (__ballot_sync(FULL, f0 || f1) >> g.base) & GBITS;
        const u32 lf = fm ? __ffs(fm) - 1 : 0;
        const unsigned long long cur = f0 ? pack_pair(x.x, x.y) : pack_pair(x.z, x.w);
        const u64 sa = __shfl_sync(FULL, (unsigned long long)(bp + (f0 ? 0 : 2)), g.base + lf);
        const unsigned long long so = __shfl_sync(FULL, cur, g.base + lf);
        if (mine && ar && !hit) {
          if (whole && fm) { state = ST_CAS; cas_addr = reinterpret_cast<u32*>(sa); cas_old = so; }
          else state = ST_SLOW;
        }
      }
    }
    // ---- 4. one CAS per lane, all in flight together
    if (state == ST_CAS) {
      if (OP == OP_DELETE) {
        if (atomicCAS(cas_addr, v, kTomb) == v) {
          atomicSub(&t.dir[row].deg, 1u);
          ++my_count;
        }
        state = ST_DONE;  // a lost CAS means another op deleted the key (Q5)
      } else if (OP == OP_INSERT) {
        const unsigned long long old =
            atomicCAS(reinterpret_cast<unsigned long long*>(cas_addr), cas_old,
                      (unsigned long long)pack_pair(v, w));
        if (old == cas_old) {
          atomicAdd(&t.dir[row].deg, 1u);
          ++my_count;
          state = ST_DONE;
        } else if ((u32)old == v) {  // a racing op installed the same key: replace
          st_relaxed_u32(cas_addr + 1, w);
          state = ST_DONE;
        } else {
          state = ST_SLOW;
        }
      }
    }
    // ---- 5. sequential chain walks for the rest
    u32 slow = g.ballot(state == ST_SLOW);
    while (slow) {
      const u32 r = __ffs(slow) - 1;
      slow &= slow - 1;
      const u32 vr = g.shfl(v, r);
      const u32 hr = g.shfl(head, r);
      const u32 rowr = g.shfl(row, r);
      if (OP == OP_INSERT) {
        const u32 wr = g.shfl(w, r);
        const int s = probe_insert<G>(t, g, rowr, hr, vr, wr, spare, stack_size, reuse);
        if (g.gl == r) {
          if (s == 1) {
            atomicAdd(&t.dir[row].deg, 1u);
            ++my_count;
          } else if (s < 0) {
            a.retry_out[atomicAdd(&t.ctl->retry_count, 1u)] = opid;
          }
        }
      } else if (OP == OP_DELETE) {
        const int s = probe_delete<G>(t, g, hr, vr);
        if (s && g.gl == r) {
          atomicSub(&t.dir[row].deg, 1u);
          ++my_count;
        }
      } else {
        u32 val = 0;
        const bool f = probe_query<G>(t, g, hr, vr, val);
        if (g.gl == r) { res_found = f; res_val = f ? val : 0u; }
      }
    }
    if (OP == OP_QUERY && valid) {
      a.found[j] = res_found ? 1 : 0;
      if (a.wout) a.wout[j] = res_found ? res_val : 0u;
    }
  }
  // ---- epilogue: hand back an unused spare bucket, reduce the batch counter
  if (OP == OP_INSERT && spare != kNil && g.gl == 0)
    t.ret_list[atomicAdd(&t.ctl->ret_count, 1u)] = spare;
  if (OP == OP_QUERY) {
    if (__any_sync(0xFFFFFFFFu, bad_range) && g.lane == 0)
      atomicMax(&t.ctl->fail_epoch, a.epoch);
  } else {
    const u32 tot = __reduce_add_sync(0xFFFFFFFFu, my_count);
    if (g.lane == 0 && tot)
      atomicAdd(reinterpret_cast<unsigned long long*>(&t.ctl->count), (unsigned long long)tot);
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
  k_edges<G, OP><<<(unsigned)blocks, kEdgeBlock, 0, s>>>(t, a); note_kernel(1);
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
  k_validate<<<(unsigned)blocks, 256, 0, s>>>(src, dst, n, nv, epoch, ctl); note_kernel(1);
  return cudaGetLastError();
}

cudaError_t launch_fixup_alloc(const Tables& t, cudaStream_t s) {
  k_fixup_alloc<<<1, 256, 0, s>>>(t); note_kernel(1);
  return cudaGetLastError();
}

}  // namespace dg
