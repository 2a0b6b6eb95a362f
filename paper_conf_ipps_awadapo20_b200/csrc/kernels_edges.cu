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
//   * uniform layouts: lane L reads its row's chain count from an L2-resident byte
//     array; a key that hashes to chain 0 goes straight to the row's HOME bucket
//     (addressed by row) without a directory access, the others read
//     the directory entry for their chain's first bucket; the degree-adaptive layout
//     reads the directory entry first;
//   * a "group" of G = bucket_bytes/16 lanes then probes the G ops of its lanes one
//     after another, each lane holding 16 B of the bucket (one 128-B bucket = one
//     coalesced request of 8 lanes); 32/G groups per warp probe independently;
//   * a new pair is installed with one 64-bit CAS on (key, value) into the chain's
//     first free slot; after a lost CAS on an EMPTY slot the next slot of the bucket
//     is tried with a 32-bit key CAS (EMPTY -> key) followed by a plain value store
//     (legal under phase concurrency: no reader runs during an insert phase;
//     DESIGN.md §4.2).  The set variant always installs with a 32-bit key CAS.  A
//     deletion is a 32-bit CAS key -> tombstone, so exactly one of several racing
//     deleters wins and degrees stay exact (Alg1:L9-10);
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

// After a lost install CAS on an EMPTY slot, try the next slot of the bucket once
// before re-scanning (measured on B200, cfg2: src-sorted bulk build 10.98 -> 6.8 ms,
// random 2^24 insert 1.20 -> 1.21 ms; walking the whole bucket spills registers and
// costs random inserts 6%)
#ifndef DG_SLOT_WALK
#define DG_SLOT_WALK 1
#endif
// Speculative chain-0 probe in the MAIN round, bit OP (insert 1, delete 2, query 4):
// measured slower on B200 (profiles/r02/ab/spec/: cfg2 query 0.633 -> 0.837 ms, insert
// 1.21 -> 1.34 ms; cfg3, where every key is in chain 0, 0.577 -> 0.587 ms): off
#ifndef DG_SPEC_HOME
#define DG_SPEC_HOME 0
#endif
#ifndef DG_SLOT_WALK_ONCE
#define DG_SLOT_WALK_ONCE 1
#endif
#ifndef DG_SLOT_WALK_MAIN
#define DG_SLOT_WALK_MAIN 1
#endif


// ----------------------------------------------------------- allocator (a8) ----
// Phase-concurrent free stack + bump cursor: during an insert
// phase buckets are only popped, during a vertex-deletion phase only pushed, so
// a single cursor per direction is ABA-free.  Pops take stack entries from the top
// (index stack_size - 1 - i for the i-th pop); past the stack, buckets come from the
// bump cursor.  Stack sizes are fixed during an insert phase.

// Per-warp bucket chunks: a warp takes `chunk` consecutive pops of a class's free
// stack (or, once the stack is exhausted, `chunk` consecutive bump slots) with ONE
// atomic and hands them to its extending lanes over later rounds.  Chain growth is
// otherwise serialised on the two allocator counters of the class: in the cfg4 R-MAT
// insert batches (~3% of ops extend a chain) per-warp-round atomics on one address
// took a fifth of the kernel's stall samples.  The unused rest of every chunk goes
// back with the spare buckets at kernel end.  Chunk state lives in shared memory
// (warp-uniform, touched only when a lane extends), per size class:
// {pos, end, mode (0 = stack, 1 = bump), stack size at kernel start}.
constexpr u32 kChunk = 32;  // largest chunk; a launch uses a.chunk (small batches less)

__device__ __forceinline__ u32* warp_chunk(u32 c) {
  __shared__ u32 s_chunk[kEdgeBlock / 32][kClasses][4];
  return s_chunk[threadIdx.x >> 5][c];
}

// lane 0 of each warp, at kernel start (stack sizes are fixed during an insert phase)
template <bool A>
__device__ __forceinline__ void init_chunks(const Tables& t) {
  for (u32 c = 0; c < (A ? (u32)kClasses : 1u); ++c) {
    u32* sc = warp_chunk(c);
    const u32 ss = ld_relaxed_u32(&t.ctl->stack_size[c]);
    sc[0] = sc[1] = 0;
    sc[2] = ss ? 0u : 1u;
    sc[3] = ss;
  }
}

__device__ __forceinline__ u32 chunk_id(const Tables& t, u32 c, u32 mode, u32 ss, u32 k) {
  if (mode == 0) return by_class(t.stack, c)[ss - 1 - k];
  return k < by_class(t.cap, c) ? (c << kClassShift) | k : kNil;
}

// Called by the whole warp; returns a bucket id of class c (NIL when the pool is
// exhausted) for lanes with `want`, NIL for the others.
template <bool A>
__device__ __forceinline__ u32 alloc_bucket_chunk(const Tables& t, bool want, u32 c, u32 chunk) {
  const u32 lane = threadIdx.x & 31u;
  const u32 below = (1u << lane) - 1u;
  u32 id = kNil;
  bool need = want;
  while (true) {
    const u32 nm = __ballot_sync(0xFFFFFFFFu, need);
    if (nm == 0) break;
    // serve the lanes of one class per pass (uniform layouts: class 0 only)
    const u32 cc = A ? __shfl_sync(0xFFFFFFFFu, c, __ffs(nm) - 1) : 0u;
    const bool mine = need && (!A || c == cc);
    const u32 m = A ? __ballot_sync(0xFFFFFFFFu, mine) : nm;
    u32* sc = warp_chunk(cc);
    const u32 n = __popc(m), rank = __popc(m & below);
    const u32 pos = sc[0], end = sc[1], mode = sc[2], ss = sc[3];
    const u32 avail = end - pos;
    const u32 take = n < avail ? n : avail;
    if (mine && rank < take) {
      id = chunk_id(t, cc, mode, ss, pos + rank);
      need = false;
    }
    __syncwarp();
    if (lane == 0) {
      sc[0] = pos + take;
      if (n > avail) {  // refill: the chunk is used up
        bool stack = mode == 0;
        if (stack) {
          const u32 i0 = atomicAdd(&t.ctl->pop_count[cc], chunk);
          if (i0 < ss) {
            sc[0] = i0;
            sc[1] = i0 + chunk < ss ? i0 + chunk : ss;
          } else {
            stack = false;
          }
        }
        if (!stack) {
          const u32 b0 = atomicAdd(&t.ctl->bump[cc], chunk);
          sc[0] = b0;
          sc[1] = b0 + chunk;
          sc[2] = 1;
        }
      }
    }
    __syncwarp();
  }
  return id;
}

// hand the unused rest of the warp's chunks back (kernel end; whole warp)
template <bool A>
__device__ __forceinline__ void release_chunks(const Tables& t) {
  const u32 lane = threadIdx.x & 31u;
  for (u32 c = 0; c < (A ? (u32)kClasses : 1u); ++c) {
    const u32* sc = warp_chunk(c);
    const u32 pos = sc[0], end = sc[1], mode = sc[2], ss = sc[3];
    for (u32 k = pos + lane; k < end; k += 32) {
      const u32 id = chunk_id(t, c, mode, ss, k);
      if (id != kNil) t.ret_list[atomicAdd(&t.ctl->ret_count, 1u)] = id;
    }
  }
}

// ------------------------------------------------------------- main kernel ----
// Per warp iteration (32 ops of the batch):
//   1. lane L stages op L (coalesced loads) and gathers its directory entry; its
//      op starts at the head bucket b = base + hash(v) mod nb of A_u;
//   2. rounds, until no op of the warp is pending:
//      a. each group of G lanes loads the CURRENT bucket of each of its G pending ops
//         (G independent 16-B loads per lane: up to 32 buckets in flight per warp);
//      b. with full-warp ballots/shuffles (each lane reads its own group's lanes;
//         no divergence, no group-masked syncs) every op is decided from its
//         bucket: key found / chain ended / continue to `next`;
//      c. the lane that owns an op performs its atomic: the delete CAS
//         key -> tombstone, the insert CAS of (key, value) into the chain's first
//         free slot, or the allocation + CAS-link of a new tail bucket — all lanes
//         of the warp in one instruction.
//   The insert follows Alg. 1's replace: the whole chain is scanned
//   for the key before a new pair is installed; the install targets the FIRST free
//   slot (first tombstone when tombstones are reused, else the first
//   EMPTY); a failed install CAS tries the next slot of the bucket once
//   (when the lost slot was EMPTY) and otherwise re-scans from the head, so two
//   inserts of one key always contend for the same slot.
enum { ACT_NONE = 0, ACT_CAS_DEL = 1, ACT_CAS_INS = 2, ACT_EXTEND = 3 };

// One pass of the round loop over the 32 ops of a warp (one per lane).  MAIN:
// exactly one round; ops that still need work (a chain to walk, a lost CAS, a
// chain extension) are returned as deferred and re-run from scratch later in a
// dense backlog chunk, so a few slow ops no longer cost a whole extra round for
// the other 31 lanes.  !MAIN: rounds until every op of the warp is done.
// Lanes per op group: L lanes share one bucket of G 16-B units, each lane holding
// K = G/L units (for 128-B buckets L = 4: two 16-B loads per lane, 8 ops decided
// per warp step).
// (measured on B200, cfg2 2^24 batches: insert 1.54 -> 1.39 ms and query 0.68 ->
// 0.62 ms with L = 4; delete is faster with L = 8: 1.08 vs 1.54 ms)
template <int G, int OP>
struct Lanes {
#if defined(DG_LANES_PER_BUCKET)
  static constexpr int L = (DG_LANES_PER_BUCKET < G) ? DG_LANES_PER_BUCKET : G;
#elif defined(DG_QUERY_LANES)  // A/B switch: query lanes only
  static constexpr int L = OP == OP_QUERY ? ((DG_QUERY_LANES < G) ? DG_QUERY_LANES : G)
                                          : (G >= 8 && OP != OP_DELETE) ? G / 2 : G;
#else
  static constexpr int L = (G >= 8 && OP != OP_DELETE) ? G / 2 : G;
#endif
  static constexpr int K = G / L;
};

// A: degree-adaptive layout (bucket geometry from the id's size class, G = 8 lanes
// cover the largest class; lanes past a smaller bucket load nothing).
template <int G, int S, int OP, bool MAIN, bool A>
__device__ __forceinline__ bool run_ops(const Tables& t, const EdgeBatch& a,
                                        const Group<Lanes<G, OP>::L>& g, const bool valid,
                                        const u64 opid, const u64 j, const bool reuse, u32& my_count, u32& spare,
                                        bool& bad_range) {
  typedef Lay<G, S> LY;
  typedef Geo<G, S, A> GEO;
  constexpr int L = Lanes<G, OP>::L;
  constexpr int K = Lanes<G, OP>::K;
  constexpr u32 FULL = 0xFFFFFFFFu;
  constexpr u32 GBITS = (L == 32) ? 0xFFFFFFFFu : ((1u << L) - 1u);
  bool deferred = false;
  // ---- 1. stage one op per lane
  u32 u = 0, v = 0, w = 0;
  if (valid) {
    u64 i = opid;
    const bool rev = opid >= a.n;  // undirected mirror op
    if (rev) i = opid - a.n;
    u = a.src[i];
    v = a.dst[i];
    if (OP == OP_INSERT && a.w) w = a.w[i];
    if (rev) { const u32 x = u; u = v; v = x; }
  }
  bool pend = valid && u != v;  // self-loops are never stored (Alg1:L3)
  if (OP == OP_QUERY && valid && ((u64)u >= a.nv || (u64)v >= a.nv)) {
    pend = false;
    bad_range = true;
  }
  const u32 row = (t.nranks == 1) ? u : u / t.nranks;
  u32 head = 0;
  u32 nbase = 0;
  // MAIN round, uniform layouts: speculate that the key hashes to chain 0 — the home
  // bucket's loads go out together with the chain-count byte's instead of after it;
  // an op whose key hashes to another chain is deferred to the backlog
  constexpr bool SPEC = MAIN && !A && ((DG_SPEC_HOME >> OP) & 1);
  u32 nbb_spec = 0;
  if (pend) {
    // base/nb never change during an edge phase; only deg is written (atomics)
    if constexpr (SPEC) {
      nbb_spec = __ldg(t.nbs + row);
      head = kHomeBit | row;
    } else if constexpr (A) {
      const uint2 de = (OP == OP_QUERY) ? ld_nc_dir(t.dir + row) : ld_dir(t.dir + row);
      head = de.x + bucket_of(v, de.y);
      nbase = de.y;
    } else {
      // uniform layouts: the row's chain count from the L2-resident byte array; a key
      // of chain 0 goes straight to the row's home bucket, the others read the
      // directory for the chain's first bucket
      const u32 nbb = __ldg(t.nbs + row);
      const u32 j0 = nbb < 255u ? bucket_of(v, nbb) : 1u;
      if (j0 == 0) {
        head = kHomeBit | row;
        nbase = nbb;
      } else {
        const uint2 de = (OP == OP_QUERY) ? ld_nc_dir(t.dir + row) : ld_dir(t.dir + row);
        head = chain_head<false>(de.x, row, bucket_of(v, de.y));
        nbase = de.y;
      }
    }
  }
  u32 cur = head;
  bool found = false;
  u32 val = 0;
  u32 steps = 0;                   // insert: chain buckets walked
  u32* ff = nullptr;               // insert: first free slot of the chain (pair address)
  unsigned long long ffo = 0;      //         and its contents when scanned

  // ---- 2. rounds
  while (true) {
    const u32 pm = __ballot_sync(FULL, pend);
    if (pm == 0) break;
    // a. current buckets of the group's pending ops: lane gl holds units gl*K .. gl*K+K-1
    uint4 q[L][K];
#pragma unroll
    for (int r = 0; r < L; ++r) {
      const u32 cr = __shfl_sync(FULL, cur, g.base + r);
      const GEO gr(t, cr);
      const u32* p = gr.p + 4 * K * g.gl;
      const bool pr = (pm >> (g.base + r)) & 1u;
#pragma unroll
      for (int c = 0; c < K; ++c) {
        if (pr && (!A || K * g.gl + c < gr.units))
          q[r][c] = (OP == OP_QUERY) ? ld_nc_v4(p + 4 * c) : ld_relaxed_v4(p + 4 * c);
        else q[r][c] = make_uint4(kEmpty, kEmpty, kEmpty, kEmpty);
      }
    }
    // the ops decided this round (speculation: those whose key hashes to chain 0)
    u32 pmd = pm;
    if constexpr (SPEC) {
      const bool ok = !pend || (nbb_spec < 255u && bucket_of(v, nbb_spec) == 0u);
      pmd = pm & __ballot_sync(FULL, ok);
      nbase = nbb_spec;
    }
    // b. decide: each lane scans its 2K slots in order, the group combines by ballot
    int act = ACT_NONE;
#pragma unroll
    for (int r = 0; r < L; ++r) {
      const u32 srcl = g.base + r;
      const bool pr = (pmd >> srcl) & 1u;
      const u32 vr = __shfl_sync(FULL, v, srcl);
      const u32 cr = __shfl_sync(FULL, cur, srcl);
      const u32 units = units_of<G, A>(cr);
      bool lhit = false, lempty = false, lfree = false;
      u32 hslot = 0, hval = 0, fslot = 0;   // key word indices in the bucket
      unsigned long long fcont = 0;
#pragma unroll
      for (int c = 0; c < K; ++c) {
        const uint4 x = q[r][c];
        const u32 uu = K * g.gl + c;               // 16-B unit index in the bucket
#pragma unroll
        for (int k = 0; k < LY::SPU; ++k) {
          if (!GEO::has_u(units, uu, k)) continue;  // (next, owner) words of the last unit
          const u32 kk = LY::key(x, k);
          if (pr && !lhit && kk == vr) { lhit = true; hslot = LY::word(uu, k); hval = LY::val(x, k); }
          const bool e = kk == kEmpty;
          lempty |= e;
          if (!lfree && (e || (reuse && kk == kTomb))) {
            lfree = true; fslot = LY::word(uu, k);
            fcont = S ? (unsigned long long)kk : pack_pair(kk, LY::val(x, k));
          }
        }
      }
      const u32 hit = (__ballot_sync(FULL, lhit) >> g.base) & GBITS;
      const u32 em = (__ballot_sync(FULL, lempty) >> g.base) & GBITS;
      // the last unit (odd index) is unit K-1 of lane (units-1)/K
      const u32 next = __shfl_sync(FULL, q[r][K - 1].z, g.base + (units - 1) / K);
      const bool end = em != 0 || next == kNil;  // EMPTY slots only exist at the tail
      const u32 lh = hit ? __ffs(hit) - 1 : 0;
      const bool mine = pr && g.gl == (u32)r;
      if (OP == OP_QUERY) {
        const u32 hv = __shfl_sync(FULL, hval, g.base + lh);
        if (mine) {
          if (hit) { found = true; val = hv; pend = false; }
          else if (end) pend = false;
          else cur = next;
        }
      } else if (OP == OP_DELETE) {
        const u32 hs = __shfl_sync(FULL, hslot, g.base + lh);
        if (mine) {
          if (hit) { act = ACT_CAS_DEL; ff = GEO(t, cur).p + hs; }
          else if (end) pend = false;
          else cur = next;
        }
      } else {  // insert
        const u32 wr = __shfl_sync(FULL, w, srcl);
        if (!S && lhit && g.gl == lh) st_relaxed_u32(GEO(t, cr).p + hslot + 1, wr);  // replace
        const u32 fm = (__ballot_sync(FULL, lfree) >> g.base) & GBITS;
        const u32 lf = fm ? __ffs(fm) - 1 : 0;
        const u32 sslot = __shfl_sync(FULL, fslot, g.base + lf);
        const unsigned long long so = __shfl_sync(FULL, fcont, g.base + lf);
        if (mine) {
          if (hit) {
            pend = false;
          } else {
            if (!ff && fm) { ff = GEO(t, cur).p + sslot; ffo = so; }
            if (end) {
              act = ff ? ACT_CAS_INS : ACT_EXTEND;
            } else {
              cur = next;
              // a long chain in an over-full table (more keys than base slots):
              // flag the row for re-sizing before the next batch (per-vertex chain
              // metric + rehash)
              if (++steps == t.hot_steps && t.hot_flags) {
                const u32 dr = ld_relaxed_u32(deg_ptr<G, A>(t, row));
                if (dr > nbase * GEO::bc_u(units)) {  // (home chains hold one less)
                  const u32 bit = 1u << (row & 31);
                  if (!(atomicOr(&t.hot_flags[row >> 5], bit) & bit)) {
                    const u32 k = atomicAdd(&t.ctl->hot_count, 1u);
                    if (k < t.hot_cap) t.hot_list[k] = row;
                    atomicAdd(&t.ctl->hot_pairs, dr);
                  }
                }
              }
            }
          }
        }
      }
    }
    // c. one atomic per lane, all in flight together
    if (OP == OP_DELETE && act == ACT_CAS_DEL) {
      if (atomicCAS(ff, v, kTomb) == v) {
        atomicSub(deg_ptr<G, A>(t, row), 1u);
        ++my_count;
      }
      pend = false;  // a lost CAS means another op deleted the key (Q5)
    }
    if (OP == OP_INSERT && act == ACT_CAS_INS) {
      // map: one 64-bit CAS installs (key, value); set: a 32-bit CAS installs the key
      const u32 okey = S ? atomicCAS(ff, (u32)ffo, v)
                         : (u32)atomicCAS(reinterpret_cast<unsigned long long*>(ff), ffo,
                                          (unsigned long long)pack_pair(v, w));
      if (okey == (u32)ffo) {
        atomicAdd(deg_ptr<G, A>(t, row), 1u);
        ++my_count;
        pend = false;
      } else if (okey == v) {  // a racing op installed the same key: replace
        if (!S) st_relaxed_u32(ff + 1, w);
        pend = false;
      } else {
#if DG_SLOT_WALK
        // The slot went to another key.  If it was EMPTY in this op's view it lies in
        // the tail bucket `cur`, every slot before it holds a key other than v (the
        // scan, and the CAS return for this one) and EMPTY slots form the chain's
        // suffix, so v may go into the NEXT slot of the bucket: a key CAS
        // EMPTY -> v that succeeds finds the rest of the chain empty, hence v
        // nowhere else.  Ops racing on one bucket (src-sorted batches) then install
        // one per slot in one round instead of re-scanning from the head each time.
        if (DG_SLOT_WALK_MAIN || !MAIN) {
          if ((u32)ffo == kEmpty) {
            // word index of the slot in its bucket from the address (pools are aligned
            // to the bucket size), so no bucket pointer is kept live; the slots end
            // before the (next, owner) words, or before the header of a home bucket
            const u32 nw = 4 * units_of<G, A>(cur);
            const u32 lim = nw - 2u;
            u32 off = (u32)(reinterpret_cast<uintptr_t>(ff) >> 2) & (nw - 1u);
            u32* p = ff;
#if DG_SLOT_WALK_ONCE
            if ((off += (S ? 1u : 2u)) < lim) {  // one further slot, then re-scan
#else
            while ((off += (S ? 1u : 2u)) < lim) {
#endif
              p += S ? 1 : 2;
              const u32 k2 = atomicCAS(p, kEmpty, v);
              if (k2 == kEmpty) {
                atomicAdd(deg_ptr<G, A>(t, row), 1u);
                ++my_count;
              }
              if (k2 == kEmpty || k2 == v) {  // installed, or a racing op's v: replace
                if (!S) st_relaxed_u32(p + 1, w);
                pend = false;
                off = nw;  // ends the walk (no `break`: the ONCE form is an `if`)
              }
            }
          }
        }
        if (pend) {  // bucket full (or the slot was a tombstone): re-scan from the head
          cur = head;
          ff = nullptr;
        }
#else
        cur = head;  // the slot went to another key: re-scan from the head
        ff = nullptr;
#endif
      }
    }
    if (OP == OP_INSERT) {
      // chain full: link a new bucket at the tail (a8), of the row's class
      const bool ext = act == ACT_EXTEND;
      const u32 cls = A ? cur >> kClassShift : 0u;
      if (A && ext && spare != kNil && (spare >> kClassShift) != cls) {  // spare of another class
        t.ret_list[atomicAdd(&t.ctl->ret_count, 1u)] = spare;
        spare = kNil;
      }
      const bool want = ext && spare == kNil;
      if (__any_sync(FULL, want)) {
        const u32 got = alloc_bucket_chunk<A>(t, want, cls, a.chunk);
        if (want) spare = got;
      }
    }
    if (OP == OP_INSERT && act == ACT_EXTEND) {
      if (spare == kNil) {  // pool exhausted: the host grows it and re-runs this op
        const u32 k = atomicAdd(&t.ctl->retry_count, 1u);
        if (k < a.retry_cap) a.retry_out[k] = opid;
        pend = false;
      } else {
        const GEO gs(t, spare), gc(t, cur);
        st_relaxed_u32(gs.p + gs.owner_word(), row);
        const u32 old = atomicCAS(gc.p + gc.next_word(), kNil, spare);
        if (old == kNil) {
          cur = spare;
          spare = kNil;
        } else {
          cur = old;  // another op linked first (no earlier slot can free up); keep ours
        }
      }
    }
    if (MAIN) {
      deferred = pend;
      break;
    }
  }
  if (OP == OP_QUERY && valid && !deferred) {
    a.found[j] = found ? 1 : 0;
    if (a.wout) a.wout[j] = found ? val : 0u;
  }
  return deferred;
}

#ifndef DG_INPUT_PF
#define DG_INPUT_PF 0  // (measured: no gain on cfg2, -1% on cfg3)
#endif
#ifndef DG_QUERY_PREFETCH
#define DG_QUERY_PREFETCH 0
#endif
#ifndef DG_DELETE_PREFETCH
#define DG_DELETE_PREFETCH 0
#endif
#ifndef DG_INSERT_PREFETCH
#define DG_INSERT_PREFETCH 0
#endif
template <int OP>
struct Prefetch {
  static constexpr bool on = OP == OP_QUERY    ? DG_QUERY_PREFETCH != 0
                             : OP == OP_DELETE ? DG_DELETE_PREFETCH != 0
                                               : DG_INSERT_PREFETCH != 0;
};

// resident blocks per SM the register allocation targets (measured on B200, cfg2
// 2^24 batches: insert 1.41 -> 1.35 ms and query 0.625 -> 0.603 ms at 3 blocks of
// 256 threads, 85 registers, no spills; delete is faster at 4: 1.07 vs 1.12 ms)
#ifndef DG_MINB_INS
#define DG_MINB_INS 4  // round 2 (home buckets): 4 blocks with a 148-B spill beat 3 blocks
#endif                 // at 80 registers, cfg2 insert 1.242 -> 1.206 ms (profiles/r02/ab)
#ifndef DG_MINB_QRY
#define DG_MINB_QRY 3
#endif
#ifndef DG_MINB_DEL  // (round 2, locality-ordered deletes: 5 blocks 0.666 -> 0.652 ms on cfg2,
#define DG_MINB_DEL 5  //  6 blocks 0.80 ms; profiles/r02/ab/occupancy/)
#endif
template <int OP>
struct MinBlocks {
  static constexpr int v = OP == OP_INSERT ? DG_MINB_INS : OP == OP_QUERY ? DG_MINB_QRY : DG_MINB_DEL;
};
// the allocator fixup of k_fixup by ONE block (the last of k_edges, small batches)
__device__ __forceinline__ void fixup_block(const Tables& t, u32* pub, u32 epoch);

// Software grid barrier (every block of the launch is resident: launch_g caps the grid
// at the occupancy bound and launches it cooperatively): arrivals on ctl->bar_count,
// the last arrival bumps the generation.  A barrier that is not complete after ~4 s traps (a CUDA error that
// makes the handle sticky-bad) instead of hanging.
__device__ __forceinline__ void grid_barrier(DevCtl* c) {
  __syncthreads();
  if (threadIdx.x == 0) {
    volatile u32* gen = &c->bar_gen;
    const u32 g0 = *gen;
    __threadfence();
    if (atomicAdd(&c->bar_count, 1u) == gridDim.x - 1) {
      c->bar_count = 0;
      __threadfence();
      atomicAdd(&c->bar_gen, 1u);
    } else {
      const long long t0 = clock64();
      while (*gen == g0) {
        __nanosleep(64);
        if (clock64() - t0 > (8ll << 30)) __trap();
      }
    }
    __threadfence();
  }
  __syncthreads();
}

// Fused validation of a small mutating batch (Q7, k_validate's job): every block
// checks a share of the batch, then a grid barrier, so no block mutates before the
// whole batch is known to be in range.
__device__ __forceinline__ void fused_validate(const EdgeBatch& a, DevCtl* c) {
  bool bad = false;
  const u64 stride = (u64)gridDim.x * blockDim.x;
  for (u64 i = (u64)blockIdx.x * blockDim.x + threadIdx.x; i < a.n; i += stride)
    bad |= ((u64)a.src[i] >= a.nv) | ((u64)a.dst[i] >= a.nv);
  if (__syncthreads_or(bad) && threadIdx.x == 0) atomicMax(&c->fail_epoch, a.epoch);
  if (blockIdx.x == 0 && threadIdx.x == 0) {  // (no block adds to them before the barrier)
    c->count = 0;
    c->retry_count = 0;
  }
  grid_barrier(c);
}

template <int G, int S, int OP, bool A>
__global__ void __launch_bounds__(kEdgeBlock, MinBlocks<OP>::v) k_edges(Tables t, EdgeBatch a) {
  constexpr u32 FULL = 0xFFFFFFFFu;
  const Group<Lanes<G, OP>::L> g;
  if (OP != OP_QUERY && a.fuse_validate) fused_validate(a, t.ctl);
  bool skip = false;
  if (OP != OP_QUERY) {
    if (ld_relaxed_u32(&t.ctl->fail_epoch) == a.epoch) skip = true;  // batch rejected (Q7)
  }
  if (OP == OP_INSERT && a.sorted_path && ld_relaxed_u32(&t.ctl->unsorted_epoch) != a.epoch)
    skip = true;  // src-sorted batch: k_insert_sorted installs it
  if (skip) {
    if (OP == OP_INSERT && !A && a.pub) fixup_block(t, a.pub, a.epoch);  // (every block: a no-op
    return;                                                            //  but for the last)
  }
  const bool reuse = a.reuse_tombstones != 0;
  const u64 warp = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nwarps = ((u64)gridDim.x * blockDim.x) >> 5;
  u32 my_count = 0;
  u32 spare = kNil;  // a fresh bucket this lane allocated but could not link
  bool bad_range = false;
  if (OP == OP_INSERT && g.lane == 0) init_chunks<A>(t);  // empty bucket chunks
  __syncwarp();
  // per-warp backlog of deferred op ids (shared memory)
  __shared__ unsigned long long backlog[kEdgeBlock / 32][64];
  unsigned long long* bl = backlog[threadIdx.x >> 5];
  const u32 below = (1u << g.lane) - 1u;
  u32 nbl = 0;  // warp-uniform
  for (u64 chunk = warp; chunk * 32 < a.n_ops; chunk += nwarps) {
    const u64 j = chunk * 32 + g.lane;
    const bool valid = j < a.n_ops;
#if DG_INPUT_PF
    // the next chunk's input lines (32 ops = one 128-B line per array) into L2 now, so
    // its staging loads do not wait on DRAM (no registers held across the iteration)
    if (!a.idx && g.lane < 3) {
      const u64 nx = (chunk + nwarps) * 32;
      if (nx < a.n) {
        const u32* arr = g.lane == 0 ? a.src : g.lane == 1 ? a.dst : a.w;
        if (arr) prefetch_l2(arr + nx);
      }
    }
#endif
    const u64 opid = valid ? (a.idx ? a.idx[j] : j) : 0;
    // (off by default) load the NEXT chunk's sources now and prefetch their directory
    // entries into L2 after this chunk is probed, so the next chunk's directory gather
    // overlaps this chunk's probe.  Measured on cfg2: query 0.603 -> 0.658 ms, insert +
    // delete with it as well 1.20/1.07 -> 1.24/1.18 ms: the extra request per op costs
    // more than the latency it hides.
    const u64 nj = j + (u64)nwarps * 32;
    const bool pf = Prefetch<OP>::on && !a.idx && nj < a.n_ops;
    const u32 nsrc = pf ? (nj < a.n ? __ldg(a.src + nj) : __ldg(a.dst + (nj - a.n))) : 0u;
    const bool d = run_ops<G, S, OP, true, A>(t, a, g, valid, opid, j, reuse, my_count, spare,
                                           bad_range);
    if (pf && (u64)nsrc < a.nv) prefetch_l2(t.dir + (t.nranks == 1 ? nsrc : nsrc / t.nranks));
    const u32 dm = __ballot_sync(FULL, d);
    if (d) bl[nbl + __popc(dm & below)] = OP == OP_QUERY ? j : opid;
    nbl += __popc(dm);
    __syncwarp();
    if (nbl >= 32) {
      nbl -= 32;
      const u64 op2 = bl[nbl + g.lane];
      __syncwarp();
      run_ops<G, S, OP, false, A>(t, a, g, true, op2, op2, reuse, my_count, spare,
                                  bad_range);
    }
  }
  while (nbl > 0) {  // drain the backlog
    const u32 take = nbl < 32 ? nbl : 32;
    nbl -= take;
    const bool valid = g.lane < take;
    const u64 op2 = valid ? bl[nbl + g.lane] : 0;
    __syncwarp();
    run_ops<G, S, OP, false, A>(t, a, g, valid, op2, op2, reuse, my_count, spare,
                                bad_range);
  }
  // ---- epilogue: hand back unused spare buckets, reduce the batch counter
  if (OP == OP_INSERT && spare != kNil) t.ret_list[atomicAdd(&t.ctl->ret_count, 1u)] = spare;
  if (OP == OP_INSERT) {
    __syncwarp();
    release_chunks<A>(t);
  }
  if (OP == OP_QUERY) {
    if (__any_sync(FULL, bad_range) && g.lane == 0) atomicMax(&t.ctl->fail_epoch, a.epoch);
  } else {
    const u32 tot = __reduce_add_sync(FULL, my_count);
    if (g.lane == 0 && tot)
      atomicAdd(reinterpret_cast<unsigned long long*>(&t.ctl->count), (unsigned long long)tot);
  }
  if (OP == OP_INSERT && !A && a.pub) fixup_block(t, a.pub, a.epoch);
}

// ------------------------------------------------- src-sorted batches (a3) ----
// Same-source grouping (Alg1:L4-8: a warp groups the edges of one source
// into one call on its table; bulk build from sorted COO).  When the
// batch's sources are non-decreasing (checked by k_validate), all ops of a row are
// consecutive, so the warp whose 32-op chunk holds the START of a row can own the
// row for the whole batch: no other warp touches its tables.  The owner processes
// the row's ops 32 at a time; ops that hash to one chain form a group that walks the
// chain once, and the group's distinct new keys take the chain's next free slots in
// rank order (plain stores: the chain is private) — extension buckets are allocated
// and linked for the overflow in the same pass.  Chains stay prefix-filled (EMPTY
// slots only at the tail) because every group fills from the first free
// slot on, in order, before the next group of that chain runs.  Rows with many
// chains (nb > a.excl_chains: hubs, whose ops spread over many chains and would make
// one warp walk a long run alone) go through the lock-free per-op path of k_edges
// (run_ops) in every chunk, as in unsorted batches.
//
// resident blocks per SM (measured on the cfg2 src-sorted bulk build, kernel ms: 3 blocks
// at 80 registers 3.59; 4: 3.22; 5: 3.16; 6 (40 registers + spills): 3.10; 8: 3.11)
#ifndef DG_SORTED_MINB
#define DG_SORTED_MINB 6
#endif
#ifndef DG_SORTED_PREMATCH
#define DG_SORTED_PREMATCH 1
#endif
#ifndef DG_SORTED_PF  // load the next chunk's inputs while the current one is installed
#define DG_SORTED_PF 0    // (measured: 4.41 -> 4.51 ms on the cfg2 sorted build: registers)
#endif
#ifndef DG_SORTED_TMA  // stage the next chunk's inputs in shared memory with bulk copies
#define DG_SORTED_TMA 0   // (measured: 3.87 -> 3.99 ms on the cfg2 sorted build)
#endif
#ifndef DG_SORTED_DENSE  // owned rows in dense passes (else: chunk pass + tail-row passes)
#define DG_SORTED_DENSE 2
#endif

// one warp's staged 32-op chunk: src (with the 4 ops before the chunk), dst, weight
struct alignas(16) SortedStage {
  u32 src[36];
  u32 dst[32];
  u32 w[32];
};

// position of the n-th (0-based) set bit of m
__device__ __forceinline__ u32 nth_bit(u32 m, u32 n) {
  for (u32 k = 0; k < n; ++k) m &= m - 1;
  return __ffs(m) - 1;
}

// Exclusive-ownership install of the active lanes' ops (one op per lane; the warp
// owns every row involved).  Returns nothing; counts into my_count.
template <int G, int S, bool A>
__device__ __forceinline__ void install_owned(const Tables& t, const EdgeBatch& a, bool act,
                                              u64 opid, u32 row, u32 v, u32 w, u32 base,
                                              u32 nb, u32& my_count) {
  typedef Lay<G, S> LY;
  typedef Geo<G, S, A> GEO;
  constexpr u32 FULL = 0xFFFFFFFFu;
  const u32 lane = threadIdx.x & 31u;
  const u32 below = (1u << lane) - 1u;
  // duplicates of one key among the lanes: the last one (batch order) writes (Q1).
  // A 32-bit hash match first: the exact 64-bit match only when two lanes' hashes
  // collide (duplicate keys are rare; equal keys always have equal hashes).
  const u32 below0 = (1u << lane) - 1u;
  u32 dm = 1u << lane;
#if DG_SORTED_PREMATCH
  const u32 h32 = act ? (v ^ (row * 0x9E3779B1u)) : (0xFFFFFF00u | lane);
  const u32 hm = __match_any_sync(FULL, h32);
  if (__any_sync(FULL, act && (hm & ~(1u << lane))))
#endif
  {
    const u64 kk = act ? (((u64)row << 32) | v) : (~0ull - lane);
    dm = __match_any_sync(FULL, kk);
  }
  (void)below0;
  const bool writer = act && (dm >> lane) == 1u;  // highest lane of its key
  // walk the op's chain: the key, or the first free (EMPTY) slot and the tail bucket
  u32 j = 0, b = kNil, hit_word = kNil, tail = kNil, e = 0;
  if (writer) {
    j = bucket_of(v, nb);
    b = chain_head<A>(base, row, j);
    while (true) {
      const GEO gb(t, b);
      u32 first_empty = kNil;
      u32 next = kNil;
      for (u32 uu = 0; uu < gb.units; ++uu) {
        const uint4 x = ld_relaxed_v4(gb.p + 4 * uu);
#pragma unroll
        for (int k = 0; k < LY::SPU; ++k) {
          if (!gb.has(uu, k)) continue;
          const u32 key = LY::key(x, k);
          if (key == v && hit_word == kNil) hit_word = LY::word(uu, k);
          if (key == kEmpty && first_empty == kNil) first_empty = uu * LY::SPU + k;
        }
        if (uu == gb.units - 1) next = x.z;
      }
      if (hit_word != kNil) { tail = b; break; }
      if (first_empty != kNil) { tail = b; e = first_empty; break; }  // EMPTY: the chain ends here
      if (next == kNil) { tail = b; e = gb.bc(); break; }             // full tail bucket
      b = next;
    }
  }
  const bool hit = writer && hit_word != kNil;
  if (hit && !S) st_relaxed_u32(GEO(t, tail).p + hit_word + 1, w);  // replace
  const bool fresh = writer && !hit;
  // groups: the fresh keys of one chain, ranked in lane (= batch) order.  Owned rows
  // have <= 256 chains, so (row, chain) packs exactly into 32 bits below 2^24 rows
  // (a 32-bit match is cheaper than a 64-bit one)
  u32 gm;
  if (t.rows < (1ull << 24) - 1)
    gm = __match_any_sync(FULL, fresh ? (row << 8 | j) : (0xFFFFFFFFu - lane));
  else
    gm = __match_any_sync(FULL, fresh ? (((u64)row << 32) | j) : (~0ull - 64 - lane));
  gm &= __ballot_sync(FULL, fresh);
  const u32 r = __popc(gm & below);
  const u32 bct = fresh ? GEO(t, tail).bc() : 0u;
  const u32 cls = A ? (tail >> kClassShift) : 0u;
  const u32 avail = fresh ? bct - e : 0u;
  // overflow: ranks >= avail go to new pool buckets of bcn slots (the row's class)
  const u32 bcn = bct;
  const bool over = fresh && r >= avail;
  const u32 q = over ? r - avail : 0u;
  const bool want = over && q % bcn == 0;  // the first key of each new bucket allocates it
  u32 got = kNil;
  if (__any_sync(FULL, want)) got = alloc_bucket_chunk<A>(t, want, cls, a.chunk);
  // the new buckets of the group, k-th held by the lane of rank avail + k*bcn
  const u32 kb = over ? q / bcn : 0u;
  u32 mine = kNil, pred = tail;
  {
    const u32 src_mine = over ? nth_bit(gm, avail + kb * bcn) : lane;
    const u32 src_pred = (over && kb > 0) ? nth_bit(gm, avail + (kb - 1) * bcn) : lane;
    const u32 m1 = __shfl_sync(FULL, got, src_mine);
    const u32 m2 = __shfl_sync(FULL, got, src_pred);
    if (over) {
      mine = m1;
      if (kb > 0) pred = m2;
    }
  }
  // a group whose allocation failed anywhere: its overflow ops retry later (the host
  // grows the pool), and the buckets it did get are handed back
  const bool fail = over && mine == kNil;
  const u32 failm = __ballot_sync(FULL, fail);
  const bool group_failed = over && (failm & gm) != 0;
  if (want && got != kNil && group_failed) {
    t.ret_list[atomicAdd(&t.ctl->ret_count, 1u)] = got;
  }
  if (over && group_failed) {
    const u32 k = atomicAdd(&t.ctl->retry_count, 1u);
    if (k < a.retry_cap) a.retry_out[k] = opid;
  }
  if (want && got != kNil && !group_failed) {  // link: pred.next = got, owner word = row
    const GEO gn(t, got), gp(t, pred);
    gn.p[gn.owner_word()] = row;
    gp.p[gp.next_word()] = got;
  }
  const bool store = fresh && !group_failed;
  if (store) {
    const u32 bk = over ? mine : tail;
    const u32 slot = over ? q % bcn : e + r;
    u32* p = GEO(t, bk).p + (S ? slot : 2 * slot);
    if (S) *p = v;
    else *reinterpret_cast<unsigned long long*>(p) = pack_pair(v, w);
    ++my_count;
  }
  // one degree update per group (Alg1:L9-10): its leader adds the group's installs
  const u32 sm = __ballot_sync(FULL, store) & gm;
  if (store && (sm & below) == 0) atomicAdd(deg_ptr<G, A>(t, row), __popc(sm));
  __syncwarp();  // the stores are visible to the warp's next walk
}

template <int G, int S, bool A>
__global__ void __launch_bounds__(kEdgeBlock, DG_SORTED_MINB) k_insert_sorted(Tables t, EdgeBatch a) {
  constexpr u32 FULL = 0xFFFFFFFFu;
  const Group<Lanes<G, OP_INSERT>::L> g;
  if (ld_relaxed_u32(&t.ctl->fail_epoch) == a.epoch) return;      // rejected (Q7)
  if (ld_relaxed_u32(&t.ctl->unsorted_epoch) == a.epoch) return;  // k_edges runs it
  const bool reuse = a.reuse_tombstones != 0;
  const u64 warp = ((u64)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const u64 nwarps = ((u64)gridDim.x * blockDim.x) >> 5;
  const u32 lane = g.lane;
  u32 my_count = 0;
  u32 spare = kNil;
  bool bad_range = false;
  if (g.lane == 0) init_chunks<A>(t);
  __syncwarp();
  const u64 n = a.n;  // sorted path: directed, no mirror, no index list
  // inputs of the chunk: src, dst, weight of the lane's op, the op before the chunk
  auto load_in = [&](u64 c, u32& u_, u32& v_, u32& w_, u32& p_) {
    const u64 i_ = c * 32 + lane;
    const bool ok = i_ < n;
    u_ = ok ? a.src[i_] : kNil;
    v_ = ok ? a.dst[i_] : kNil;
    w_ = (ok && a.w) ? a.w[i_] : 0u;
    p_ = (c * 32 < n && c) ? a.src[c * 32 - 1] : kNil;
  };
  u32 nu = 0, nv = 0, nw = 0, np = 0;
  if (DG_SORTED_PF) load_in(warp, nu, nv, nw, np);
#if DG_SORTED_TMA
  // Double-buffered per-warp staging: while chunk c is installed, the TMA engine
  // copies chunk c + nwarps into the other stage (full 32-op chunks of 16-B aligned
  // arrays; other chunks load directly).
  __shared__ SortedStage s_stage[kEdgeBlock / 32][2];
  __shared__ unsigned long long s_bar[kEdgeBlock / 32][2];
  const u32 wib = threadIdx.x >> 5;
  const bool tma_ok =
      ((reinterpret_cast<uintptr_t>(a.src) | reinterpret_cast<uintptr_t>(a.dst) |
        reinterpret_cast<uintptr_t>(a.w)) & 15u) == 0;
  if (tma_ok && lane == 0) {
    mbar_init(&s_bar[wib][0], 1);
    mbar_init(&s_bar[wib][1], 1);
  }
  __syncwarp();
  // warp-uniform: stage chunk c into stage st; false = not staged (load it directly)
  auto stage_in = [&](u64 c, u32 st) -> bool {
    if (!tma_ok || (c + 1) * 32 > n) return false;
    if (lane == 0) {
      const u32 pre = c ? 4u : 0u;  // the 4 ops before the chunk (for `prev`)
      SortedStage& sg = s_stage[wib][st];
      fence_proxy_async_smem();  // this warp's earlier reads of the stage come first
      mbar_expect_tx(&s_bar[wib][st], (32u + pre) * 4u + 128u + (a.w ? 128u : 0u));
      bulk_g2s(sg.src + 4 - pre, a.src + c * 32 - pre, (32u + pre) * 4u, &s_bar[wib][st]);
      bulk_g2s(sg.dst, a.dst + c * 32, 128u, &s_bar[wib][st]);
      if (a.w) bulk_g2s(sg.w, a.w + c * 32, 128u, &s_bar[wib][st]);
    }
    return true;
  };
  u32 st = 0, parity = 0;  // parity bit s: the phase to wait for on stage s
  bool staged = stage_in(warp, 0);
#endif
  for (u64 chunk = warp; chunk * 32 < n; chunk += nwarps) {
    const u64 lo = chunk * 32;
    const u64 i = lo + lane;
    const bool valid = i < n;
    u32 u, v, w, prev;  // (prev: the row of the op before the chunk)
#if DG_SORTED_TMA
    __syncwarp();  // every lane has read the other stage (previous iteration)
    const bool staged_next = stage_in(chunk + nwarps, st ^ 1u);
    if (staged) {
      mbar_wait(&s_bar[wib][st], (parity >> st) & 1u);
      parity ^= 1u << st;
      const SortedStage& sg = s_stage[wib][st];
      u = sg.src[4 + lane];
      v = sg.dst[lane];
      w = a.w ? sg.w[lane] : 0u;
      prev = lo ? sg.src[3] : kNil;
    } else {
      load_in(chunk, u, v, w, prev);
    }
    staged = staged_next;
    st ^= 1u;
#else
    if (DG_SORTED_PF) {
      u = nu; v = nv; w = nw; prev = np;
      load_in(chunk + nwarps, nu, nv, nw, np);  // consumed next iteration
    } else {
      load_in(chunk, u, v, w, prev);
    }
#endif
    const u32 row = (t.nranks == 1) ? u : u / t.nranks;
    uint2 de = make_uint2(0, 0);  // {base (uniform: xbase), nb}
    if (valid) de = ld_dir(t.dir + row);
    const bool excl = valid && de.y <= a.excl_chains;
    // 1. rows with many chains: the per-op lock-free path, every chunk its own ops
    const bool cas = valid && !excl;
    if (__any_sync(FULL, cas))
      run_ops<G, S, OP_INSERT, false, A>(t, a, g, cas, i, i, reuse, my_count, spare, bad_range);
#if DG_SORTED_DENSE == 2
    // 2. rows that start in this chunk: all their ops, in dense passes of 32
    //    consecutive ops from the first row start on (a pass holds several rows; the
    //    last row may run past the chunk).  Pass 0 takes the chunk's ops from the
    //    registers (shifted by shuffles) and the tail row's next ops from memory.
    const u32 starts = __ballot_sync(FULL, valid && (lo == 0 || u != prev));
    if (starts) {
      const u32 off = __ffs(starts) - 1;
      const u32 tail_row = __shfl_sync(FULL, u, 31);  // started here (sorted), or kNil
      const u32 trow = __shfl_sync(FULL, row, 31);
      const uint2 tde = make_uint2(__shfl_sync(FULL, de.x, 31), __shfl_sync(FULL, de.y, 31));
      const bool tail_ex = tail_row != kNil && tde.y <= a.excl_chains;
      const u32 sl = (lane + off) & 31u;
      u32 s2 = __shfl_sync(FULL, u, sl), v2 = __shfl_sync(FULL, v, sl);
      u32 w2 = __shfl_sync(FULL, w, sl), r2 = __shfl_sync(FULL, row, sl);
      uint2 de2 = make_uint2(__shfl_sync(FULL, de.x, sl), __shfl_sync(FULL, de.y, sl));
      bool in = __shfl_sync(FULL, valid ? 1 : 0, sl) != 0;
      u64 i2 = lo + off + lane;
      for (bool first = true;; first = false) {
        if (!first || lane + off >= 32) {  // beyond the chunk: the tail row's next ops
          const bool ok2 = tail_ex && i2 < n;  // (the three loads in parallel)
          s2 = ok2 ? a.src[i2] : kNil;
          v2 = ok2 ? a.dst[i2] : 0u;
          w2 = (ok2 && a.w) ? a.w[i2] : 0u;
          in = ok2 && s2 == tail_row;
          r2 = trow;
          de2 = tde;
        }
        install_owned<G, S, A>(t, a, in && de2.y <= a.excl_chains && v2 != s2, i2, r2, v2, w2,
                               de2.x, de2.y, my_count);
        if (!tail_ex || !__shfl_sync(FULL, in ? 1 : 0, 31) || i2 - lane + 32 >= n) break;
        i2 += 32;
      }
    }
#elif DG_SORTED_DENSE
    // 2. rows that start in this chunk: all their ops, in dense passes of 32
    //    consecutive ops from the first row start on (the last row may run past the
    //    chunk; a pass holds several rows)
    const u32 starts = __ballot_sync(FULL, valid && (lo == 0 || u != prev));
    if (starts) {
      const u32 tail_row = __shfl_sync(FULL, u, 31);  // started here (sorted), or kNil
      const u32 tail_nb = __shfl_sync(FULL, de.y, 31);
      for (u64 p0 = lo + (__ffs(starts) - 1);; p0 += 32) {
        const u64 i2 = p0 + lane;
        const bool ok2 = i2 < n;  // (the three loads in parallel: one round trip)
        const u32 s2 = ok2 ? a.src[i2] : kNil;
        const u32 v2 = ok2 ? a.dst[i2] : 0u;
        const u32 w2 = (ok2 && a.w) ? a.w[i2] : 0u;
        const bool in = ok2 && (i2 < lo + 32 || s2 == tail_row);
        const u32 r2 = (t.nranks == 1) ? s2 : s2 / t.nranks;
        uint2 de2 = make_uint2(0, 0);
        if (in) de2 = ld_dir(t.dir + r2);
        install_owned<G, S, A>(t, a, in && de2.y <= a.excl_chains && v2 != s2, i2, r2, v2, w2,
                               de2.x, de2.y, my_count);
        if (!__shfl_sync(FULL, in ? 1 : 0, 31) || p0 + 32 >= n || tail_nb > a.excl_chains)
          break;  // the last row ended (or is not owned)
      }
    }
#else
    // 2. rows this chunk owns (started in it): the whole row, 32 ops at a time
    const bool owned = excl && (lo == 0 || u != prev);
    install_owned<G, S, A>(t, a, owned && u != v, i, row, v, w, de.x, de.y, my_count);
    // the last owned row may continue past the chunk
    const u32 tail_row = __shfl_sync(FULL, u, 31);
    const bool cont = __shfl_sync(FULL, owned ? 1 : 0, 31) != 0 && lo + 32 < n;
    if (cont) {
      const uint2 tde = make_uint2(__shfl_sync(FULL, de.x, 31), __shfl_sync(FULL, de.y, 31));
      const u32 trow = (t.nranks == 1) ? tail_row : tail_row / t.nranks;
      for (u64 lo2 = lo + 32; lo2 < n; lo2 += 32) {
        const u64 i2 = lo2 + lane;
        const bool ok2 = i2 < n;  // (the three loads in parallel: one round trip)
        const u32 s2 = ok2 ? a.src[i2] : kNil;
        const u32 v2r = ok2 ? a.dst[i2] : 0u;
        const u32 w2r = (ok2 && a.w) ? a.w[i2] : 0u;
        const bool in = ok2 && s2 == tail_row;
        const u32 v2 = in ? v2r : 0u;
        const u32 w2 = in ? w2r : 0u;
        install_owned<G, S, A>(t, a, in && v2 != tail_row, i2, trow, v2, w2, tde.x, tde.y,
                               my_count);
        if (__ballot_sync(FULL, in) != FULL) break;  // the run ended in this sub-chunk
      }
    }
#endif
  }
  if (spare != kNil) t.ret_list[atomicAdd(&t.ctl->ret_count, 1u)] = spare;
  __syncwarp();
  release_chunks<A>(t);
  const u32 tot = __reduce_add_sync(FULL, my_count);
  if (lane == 0 && tot)
    atomicAdd(reinterpret_cast<unsigned long long*>(&t.ctl->count), (unsigned long long)tot);
}

// ---------------------------------------------------------------- helpers ----
// Validation (Q7) for mutating batches: any endpoint >= capacity rejects the
// batch; also resets the per-batch counters (they are only written by kernels
// that run after this one on the stream).
template <bool VEC>
__global__ void __launch_bounds__(256) k_validate(const u32* __restrict__ src,
                                                 const u32* __restrict__ dst, u64 n, u64 nv,
                                                 u32 epoch, DevCtl* ctl) {
  // kQ quads (VEC: 16-B loads, arrays 16-B aligned) or kQ * 4 single ops per thread and
  // step, all loads issued before any is consumed
  constexpr int kQ = 2;
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    ctl->count = 0;
    ctl->retry_count = 0;
  }
  const u32 lane = threadIdx.x & 31u;
  bool bad = false, unsorted = false;
  const u64 step = (u64)gridDim.x * blockDim.x * kQ * 4;
  for (u64 i0 = (u64)blockIdx.x * blockDim.x * kQ * 4; i0 < n; i0 += step) {
    if constexpr (VEC) {
      uint4 a[kQ], b[kQ];
      u32 prev[kQ];
#pragma unroll
      for (int k = 0; k < kQ; ++k) {
        const u64 i = i0 + 4 * ((u64)k * blockDim.x + threadIdx.x);
        if (i + 3 < n) {
          a[k] = *reinterpret_cast<const uint4*>(src + i);
          b[k] = *reinterpret_cast<const uint4*>(dst + i);
        } else {  // the tail quad
          a[k].x = i < n ? src[i] : 0u;      b[k].x = i < n ? dst[i] : 0u;
          a[k].y = i + 1 < n ? src[i + 1] : a[k].x;  b[k].y = i + 1 < n ? dst[i + 1] : 0u;
          a[k].z = i + 2 < n ? src[i + 2] : a[k].y;  b[k].z = i + 2 < n ? dst[i + 2] : 0u;
          a[k].w = a[k].z;                   b[k].w = 0u;
          if (i >= n) a[k] = make_uint4(0xFFFFFFFFu, 0xFFFFFFFFu, 0xFFFFFFFFu, 0xFFFFFFFFu);
        }
        prev[k] = lane == 0 && i > 0 && i < n ? src[i - 1] : 0u;  // (the warp's left neighbour)
      }
#pragma unroll
      for (int k = 0; k < kQ; ++k) {
        const u64 i = i0 + 4 * ((u64)k * blockDim.x + threadIdx.x);
        const u32 left = __shfl_up_sync(0xFFFFFFFFu, a[k].w, 1);
        if (i < n) {
          const u32 mx = max(max(a[k].x, a[k].y), max(a[k].z, a[k].w));
          const u32 my = max(max(b[k].x, b[k].y), max(b[k].z, b[k].w));
          bad |= ((u64)mx >= nv) | ((u64)my >= nv);
          unsorted |= a[k].y < a[k].x || a[k].z < a[k].y || a[k].w < a[k].z ||
                      (i > 0 && a[k].x < (lane == 0 ? prev[k] : left));
        }
      }
    } else {
      u32 us[kQ * 4], vs[kQ * 4], prev[kQ * 4];
#pragma unroll
      for (int k = 0; k < kQ * 4; ++k) {
        const u64 i = i0 + (u64)k * blockDim.x + threadIdx.x;
        us[k] = i < n ? src[i] : 0u;
        vs[k] = i < n ? dst[i] : 0u;
        prev[k] = lane == 0 && i > 0 && i < n ? src[i - 1] : 0u;
      }
#pragma unroll
      for (int k = 0; k < kQ * 4; ++k) {
        const u64 i = i0 + (u64)k * blockDim.x + threadIdx.x;
        const u32 left = __shfl_up_sync(0xFFFFFFFFu, us[k], 1);
        if (i < n) {
          bad |= ((u64)us[k] >= nv) | ((u64)vs[k] >= nv);
          unsorted |= i > 0 && us[k] < (lane == 0 ? prev[k] : left);
        }
      }
    }
  }
  if (__any_sync(0xFFFFFFFFu, bad) && lane == 0) atomicMax(&ctl->fail_epoch, epoch);
  if (__any_sync(0xFFFFFFFFu, unsorted) && lane == 0) atomicMax(&ctl->unsorted_epoch, epoch);
}

// After an insert phase: drop the popped entries from each class's free stack,
// clamp the bump cursors, and push the spare buckets that were handed back onto the
// stack of their class.
__global__ void k_fixup_alloc(Tables t, bool copied) {
  __shared__ u32 s_ss[kClasses], s_rc;
  DevCtl* c = t.ctl;
  if (threadIdx.x < kClasses) {
    const u32 k = threadIdx.x;
    const u32 pc = c->pop_count[k], ss = c->stack_size[k];
    s_ss[k] = pc >= ss ? 0u : ss - pc;
    if (c->bump[k] > by_class(t.cap, k)) c->bump[k] = by_class(t.cap, k);
  }
  if (threadIdx.x == 0) s_rc = c->ret_count;
  __syncthreads();
  if (copied) {  // uniform layouts: k_fixup_copy already pushed them
    if (threadIdx.x == 0) s_ss[0] += s_rc;
  } else {
    for (u32 k = threadIdx.x; k < s_rc; k += blockDim.x) {
      const u32 id = t.ret_list[k];
      const u32 cl = id >> kClassShift;
      by_class(t.stack, cl)[atomicAdd(&s_ss[cl], 1u)] = id;
    }
  }
  __syncthreads();
  if (threadIdx.x < kClasses) {
    c->stack_size[threadIdx.x] = s_ss[threadIdx.x];
    c->pop_count[threadIdx.x] = 0;
  }
  if (threadIdx.x == 0) c->ret_count = 0;
}

// ---------------------------------------------------------------- launchers ----
template <int G, int S, int OP, bool A>
static int grid_for() {
  static int blocks_per_sm = -1;
  if (blocks_per_sm < 0) {
    int b = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, k_edges<G, S, OP, A>, kEdgeBlock, 0) !=
            cudaSuccess || b <= 0)
      b = 1;
    blocks_per_sm = b;
  }
  return blocks_per_sm;
}

template <int G, int S, bool A>
static cudaError_t launch_sorted(const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  static int bps = -1;
  if (bps < 0) {
    int b = 0;
    if (cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, k_insert_sorted<G, S, A>, kEdgeBlock, 0) !=
            cudaSuccess || b <= 0)
      b = 1;
    bps = b;
  }
  const u64 warps = (a.n + 31) / 32;
  u64 blocks = (warps + kEdgeBlock / 32 - 1) / (kEdgeBlock / 32);
  const u64 maxb = (u64)sms * bps;
  if (blocks > maxb) blocks = maxb;
  k_insert_sorted<G, S, A><<<(unsigned)blocks, kEdgeBlock, 0, s>>>(t, a);
  note_kernel(1);
  return cudaGetLastError();
}

template <int G, int S, int OP, bool A>
static cudaError_t launch_g(const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  if (a.n_ops == 0) return cudaSuccess;
  const u64 warps_needed = (a.n_ops + 31) / 32;
  const u64 per_block = kEdgeBlock / 32;
  u64 blocks = (warps_needed + per_block - 1) / per_block;
  const u64 maxb = (u64)sms * grid_for<G, S, OP, A>();
  if (blocks > maxb) blocks = maxb;
  // bucket chunk per warp: ~1/4 of the ops a warp handles, 1..kChunk (a small batch
  // would otherwise strand most of every chunk)
  const u64 per_warp = a.n_ops / (blocks * per_block);
  EdgeBatch ab = a;
  ab.chunk = (u32)(per_warp / 4 < 1 ? 1 : per_warp / 4 > kChunk ? kChunk : per_warp / 4);
  if (OP == OP_INSERT && ab.sorted_path) {
    // exactly one of the two kernels does the work (k_validate's sortedness verdict)
    const cudaError_t e = launch_sorted<G, S, A>(t, ab, sms, s);
    if (e != cudaSuccess) return e;
  } else {
    ab.sorted_path = 0;
  }
  if (OP != OP_QUERY && ab.fuse_validate) {
    // the fused validation's grid barrier needs every block resident: a cooperative
    // launch guarantees it even when other kernels (another handle's, another
    // stream's) hold part of the GPU
    Tables tt = t;
    void* args[] = {&tt, &ab};
    const cudaError_t e = cudaLaunchCooperativeKernel((const void*)k_edges<G, S, OP, A>,
                                                      dim3((unsigned)blocks), dim3(kEdgeBlock),
                                                      args, 0, s);
    note_kernel(1);
    return e;
  }
  k_edges<G, S, OP, A><<<(unsigned)blocks, kEdgeBlock, 0, s>>>(t, ab); note_kernel(1);
  return cudaGetLastError();
}

template <int OP>
static cudaError_t launch_op(int lay, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  switch (lay) {
#define DG_CASE(G, S, A) case DG_LAYA(G, S, A): return launch_g<G, S, OP, A>(t, a, sms, s);
    DG_FOR_LAYOUTS_A(DG_CASE)
#undef DG_CASE
    default: return cudaErrorInvalidValue;
  }
}

cudaError_t launch_insert(int lay, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  return launch_op<OP_INSERT>(lay, t, a, sms, s);
}
cudaError_t launch_delete(int lay, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  return launch_op<OP_DELETE>(lay, t, a, sms, s);
}
cudaError_t launch_query(int lay, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s) {
  return launch_op<OP_QUERY>(lay, t, a, sms, s);
}

u64 spare_bound(u64 n_ops, int ncls, int G, int sms) {
  // a launch of n_ops ops takes at most one bucket per extending op (linked or kept
  // as its lane's spare) plus, per warp and size class, the unused rest of its last
  // chunk (< one bucket per op of the warp): small batches need far less than the
  // machine-wide bound
  const u64 small = n_ops * (1 + (u64)ncls) + 4096;
  const u64 big = max_groups(G, sms);
  return small < big ? small : big;
}

u64 max_groups(int G, int sms) {
  // upper bound on the buckets an insert launch takes beyond the ones it links: each
  // resident thread may hold one spare bucket, each resident warp the unused rest of
  // a chunk (kChunk - 1)
  (void)G;
  return (u64)sms * 2048 * 2;
}

cudaError_t launch_validate(const u32* src, const u32* dst, u64 n, u64 nv, u32 epoch, DevCtl* ctl,
                            int sms, cudaStream_t s) {
  u64 blocks = (n + 2047) / 2048;
  if (blocks > (u64)sms * 8) blocks = (u64)sms * 8;
  if (blocks == 0) blocks = 1;
  if (((reinterpret_cast<uintptr_t>(src) | reinterpret_cast<uintptr_t>(dst)) & 15) == 0)
    k_validate<true><<<(unsigned)blocks, 256, 0, s>>>(src, dst, n, nv, epoch, ctl);
  else
    k_validate<false><<<(unsigned)blocks, 256, 0, s>>>(src, dst, n, nv, epoch, ctl);
  note_kernel(1);
  return cudaGetLastError();
}

// What the host reads from mapped memory after an insert (no copy, no event; it may
// lag behind the stream): the re-sizing counters and, tagged with the batch's epoch,
// the allocator cursors (the host bounds the cursors of launches not yet published).
// Layout (u32): [0] hot_count, [1] hot_pairs, [2..4] bump per class, [5] epoch
// (written last, after a fence, so a host that sees the epoch sees the cursors).
__device__ __forceinline__ void publish(const DevCtl* c, u32* out, u32 epoch) {
  volatile u32* o = out;
  o[0] = c->hot_count;
  o[1] = c->hot_pairs;
  for (int k = 0; k < kClasses; ++k) o[2 + k] = c->bump[k];
  __threadfence_system();
  o[5] = epoch;
}

// Every block of the launch calls this at its end; the last one to arrive (a fenced
// counter) pushes the returned spare buckets onto the free stack, moves the cursors
// and publishes them (uniform layouts; the launcher uses it for small batches, where
// one block copies the few returned buckets quickly).
__device__ __forceinline__ void fixup_block(const Tables& t, u32* pub, u32 epoch) {
  __shared__ bool last;
  __threadfence();
  __syncthreads();
  if (threadIdx.x == 0) last = atomicAdd(&t.ctl->fixup_done, 1u) == gridDim.x - 1;
  __syncthreads();
  if (!last) return;
  __threadfence();
  DevCtl* c = t.ctl;
  const u32 pc = ld_relaxed_u32(&c->pop_count[0]), ss = ld_relaxed_u32(&c->stack_size[0]);
  const u32 rc = ld_relaxed_u32(&c->ret_count);
  const u32 base = pc >= ss ? 0u : ss - pc;
  for (u32 k = threadIdx.x; k < rc; k += blockDim.x) t.stack[0][base + k] = t.ret_list[k];
  __syncthreads();
  if (threadIdx.x != 0) return;
  __threadfence();
  c->stack_size[0] = base + rc;
  c->pop_count[0] = 0;
  c->ret_count = 0;
  if (c->bump[0] > t.cap[0]) c->bump[0] = t.cap[0];
  publish(c, pub, epoch);
  c->fixup_done = 0;
}

// Uniform layouts, ONE launch: every block copies its share of the returned spare
// buckets onto the free stack (k_fixup_copy's work); the last block to finish (a
// fenced counter) moves the cursors (k_fixup_alloc's work) and publishes the
// re-sizing counters to `hot_out` (mapped host memory, nullable), so the host reads
// them without a copy or an event per insert batch.
__global__ void k_fixup(Tables t, u32* hot_out, u32 epoch) {
  DevCtl* c = t.ctl;
  const u32 pc = c->pop_count[0], ss = c->stack_size[0], rc = c->ret_count;
  const u32 base = pc >= ss ? 0u : ss - pc;
  const u32 stride = gridDim.x * blockDim.x;
  for (u32 k = blockIdx.x * blockDim.x + threadIdx.x; k < rc; k += stride)
    t.stack[0][base + k] = t.ret_list[k];
  __shared__ bool last;
  __threadfence();
  __syncthreads();
  if (threadIdx.x == 0) last = atomicAdd(&c->fixup_done, 1u) == gridDim.x - 1;
  __syncthreads();
  if (!last || threadIdx.x != 0) return;
  __threadfence();
  c->stack_size[0] = base + rc;
  c->pop_count[0] = 0;
  c->ret_count = 0;
  if (c->bump[0] > t.cap[0]) c->bump[0] = t.cap[0];
  if (hot_out) publish(c, hot_out, epoch);
  c->fixup_done = 0;
}

__global__ void k_hot_publish(const DevCtl* c, u32* hot_out, u32 epoch) {
  publish(c, hot_out, epoch);
}

cudaError_t launch_fixup_alloc(const Tables& t, u32* hot_out, u32 epoch, cudaStream_t s) {
  const bool uniform = t.cap[1] == 0;
  if (uniform) {
    k_fixup<<<148, 256, 0, s>>>(t, hot_out, epoch);
    note_kernel(1);
    return cudaGetLastError();
  }
  k_fixup_alloc<<<1, 256, 0, s>>>(t, false); note_kernel(1);
  if (hot_out) {
    k_hot_publish<<<1, 1, 0, s>>>(t.ctl, hot_out, epoch);
    note_kernel(1);
  }
  return cudaGetLastError();
}

}  // namespace dg
