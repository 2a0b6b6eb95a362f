// dg_common.cuh — device-side layout and primitives shared by the kernels.
//
// Data layout in HBM:
//   directory  : DirEntry[local_rows], 8 B per row {base bucket, #base buckets} and
//   degree     : the exact neighbour count (the paper's vertex dictionary holds it,
//                P:L316-322, L399-407, L426-428): u32[local_rows] (L2-resident),
//                or, with DG_HOME_DEG=1, the last word of the row's HOME bucket
//   pool       : bucket array; bucket b occupies words [b*W, (b+1)*W), W = bucket_bytes/4.
//                words 2i, 2i+1 = (key, value) of pair i, i < BC = W/2 - 1
//                (set variant: word i = key i, i < BC = W - 2; see Lay below)
//                word W-2 = next bucket index of the chain (NIL = 0xFFFFFFFF)
//                word W-1 = owner row of the bucket (for the streaming purge sweep)
//                Base buckets of a row are consecutive (Fig. 1 caption P:L357-363);
//                chained buckets come from the allocator.
//   free stack : u32[pool capacity] of reclaimed bucket indices + bump cursor
//   ctl        : DevCtl (allocator cursors, counters, validation epochs)
//
// Home buckets (uniform layouts): chain 0 of row r is bucket r of a
// separate HOME pool indexed by row, mapped exactly 2^31 buckets after the bucket
// pool's base (so `pool + id * W` addresses both; home ids = kHomeBit | row).  Home
// buckets are ordinary buckets (same slots, next) whose owner is implied by their
// index; with DG_HOME_DEG=1 their last word holds the row's DEGREE, so the degree
// update of an op on chain 0 lands on the line its probe and CAS already hold (the
// gather ceiling favours it: 15.7 G ops/s with a separate counter array, 18.4 G with
// the counter in the gathered line, tools/gather_ceiling.cu; the insert kernel does
// not: see DG_HOME_DEG below).  A probe reads the
// row's chain count from a 1-byte-per-row array (`nbs`, min(nb, 255): L2-resident,
// 4.8 MB on cfg2): a key that hashes to chain 0 goes straight to the home bucket
// without the directory; the others read the directory {xbase, nb} for chain j >= 1,
// which starts at pool bucket xbase + j - 1.
//
// Bucket ids: bits 31..30 = size class (index of the pool the bucket lives in),
// bits 29..0 = index in that pool.  Uniform layouts use class 0 only (one pool of
// `bucket_bytes` buckets) plus home ids.  The degree-adaptive layout (DG_FLAG_ADAPTIVE, SURVEY
// §8(f) row 4, "hash tables with varying slab sizes") keeps three pools:
// class c holds 32 << c byte buckets (32 / 64 / 128 B), and every bucket of a row
// (base and chained) has the row's class, so a bucket id alone fixes its geometry.
#pragma once
#include <cstdint>
#include <cuda_runtime.h>

namespace dg {

typedef uint32_t u32;
typedef uint64_t u64;

constexpr u32 kEmpty = 0xFFFFFFFFu;       // empty key slot (Q18)
constexpr u32 kTomb = 0xFFFFFFFEu;        // tombstone (deleted key)
constexpr u32 kNil = 0xFFFFFFFFu;         // end of chain / no bucket
constexpr u64 kEmptyPair = 0xFFFFFFFFFFFFFFFFull;
constexpr u32 kClassShift = 30;           // bucket id = class << 30 | index
constexpr u32 kIdxMask = (1u << kClassShift) - 1u;
constexpr int kClasses = 3;               // adaptive size classes: 32, 64, 128 B
constexpr u64 kNbMask = (1ull << 40) - 1; // packed (#buckets | class << 40) entries
constexpr u32 kHomeBit = 1u << 31;        // uniform layouts: home bucket id = kHomeBit | row
constexpr u64 kMaxHomeRows = 1ull << 30;  // rows per rank of a uniform layout

struct __align__(8) DirEntry {
  u32 base;    // first base bucket
  u32 nb;      // number of base buckets
};

struct DevCtl {
  // allocator, per size class (uniform layouts use class 0)
  u32 pop_count[kClasses];   // pops taken from the free stack during the current insert phase
  u32 stack_size[kClasses];  // reclaimed buckets on the free stack
  u32 bump[kClasses];        // next never-used bucket index
  u32 ret_count;     // unused spare buckets handed back during the current insert phase
  u32 retry_count;   // ops that found no free bucket (pool exhausted) this launch
  u32 fail_epoch;    // highest batch epoch rejected by validation (0 = none)
  u32 queue;         // work-queue cursor (vertex purge, Alg2:L3-6)
  u32 dedup_count;   // distinct vertices in the current vertex-deletion batch
  u64 count;         // n_added / n_removed / TC accumulator of the current batch
  u32 hot_count;     // rows flagged for re-sizing (long chains), see k_edges / rehash
  u32 hot_pairs;     // sum of their degrees when flagged (saturating): work to re-size
  u32 route_timeout; // a fused-exchange wait gave up on a peer (router.cu)
  u32 unsorted_epoch; // highest validated batch epoch whose sources were not sorted
  u32 fixup_done;     // blocks of k_fixup finished (last-block pattern; reset by the last)
  u32 bar_count;      // grid barrier of a small k_edges launch with fused validation:
  u32 bar_gen;        //   arrivals, generation (kernels_edges.cu grid_barrier)
};

struct Tables {
  DirEntry* dir;     // uniform layouts: {xbase, nb}; adaptive: {first base bucket, nb}
  u32* home;         // uniform layouts: home bucket of every row (chain 0), W words each
  uint8_t* nbs;      // uniform layouts: min(nb, 255) per row
  u32* deg;          // adaptive layout: exact degree per local row; uniform layouts: a
                     // snapshot written by launch_degrees for the TC orientation
  u32 hw;            // uniform layouts: words per home bucket (the degree is word hw-1)
  u32* pool[kClasses];   // bucket pool per size class
  u32* stack[kClasses];  // free stack per size class (bucket ids)
  DevCtl* ctl;
  u32* ret_list;     // spare buckets returned (<= number of groups launched)
  u64 rows;          // local rows
  u32 cap[kClasses]; // buckets mapped in each pool
  u32 nranks;        // row = global id / nranks at nranks > 1
  u32* hot_flags;    // bit per local row: flagged for re-sizing (nullable = off)
  u32* hot_list;     // flagged rows
  u32 hot_cap;       // capacity of hot_list
  u32 hot_steps;     // chain buckets an insert may walk before flagging its row
};

// The degree counter of a local row: the last word of its home bucket (uniform
// layouts) or deg[row] (adaptive layout; uniform layouts too with DG_HOME_DEG=0).
// (measured on B200, cfg2 2^24 batches, profiles/r02/ab/homedeg_*: the degree word
// dirties a second sector of the home line, DRAM writes per insert launch 0.75 ->
// 1.00 GB, insert 1.207 -> 1.413 ms, delete 0.810 -> 0.926 ms: off)
#ifndef DG_HOME_DEG
#define DG_HOME_DEG 0
#endif
__device__ __forceinline__ u32* deg_at(const Tables& t, u64 row) {
  return t.hw ? t.home + row * t.hw + (t.hw - 1) : t.deg + row;
}
template <int G, bool A>
__device__ __forceinline__ u32* deg_ptr(const Tables& t, u64 row) {
  if constexpr (A || !DG_HOME_DEG) return t.deg + row;
  else return t.home + row * (4 * G) + (4 * G - 1);
}

// ------------------------------------------------------------------ hashing ----
// Q16: murmur3 fmix32, then multiply-shift onto [0, nb).  The paper defers the
// hash to Slab Hash [6]; results are hash-independent.
__device__ __forceinline__ u32 fmix32(u32 h) {
  h ^= h >> 16; h *= 0x85ebca6bu;
  h ^= h >> 13; h *= 0xc2b2ae35u;
  h ^= h >> 16;
  return h;
}
__device__ __forceinline__ u32 bucket_of(u32 key, u32 nb) {
  return (u32)(((u64)fmix32(key) * (u64)nb) >> 32);
}

// ------------------------------------------------------------------ memory ----
// 16-B loads are issued as v2.u64 so ptxas keeps ONE 128-bit load even when only
// the key words are consumed (a v4.u32 with dead lanes is split into 32-bit loads).
__device__ __forceinline__ uint4 ld_relaxed_v4(const u32* p) {
  unsigned long long a, b;
  asm volatile("ld.relaxed.gpu.global.v2.u64 {%0,%1}, [%2];" : "=l"(a), "=l"(b) : "l"(p) : "memory");
  return make_uint4((u32)a, (u32)(a >> 32), (u32)b, (u32)(b >> 32));
}
__device__ __forceinline__ uint4 ld_nc_v4(const u32* p) {
  unsigned long long a, b;
  asm volatile("ld.global.nc.v2.u64 {%0,%1}, [%2];" : "=l"(a), "=l"(b) : "l"(p));
  return make_uint4((u32)a, (u32)(a >> 32), (u32)b, (u32)(b >> 32));
}
__device__ __forceinline__ uint2 ld_nc_dir(const DirEntry* p) {
  uint2 r;
  asm volatile("ld.global.nc.v2.u32 {%0,%1}, [%2];" : "=r"(r.x), "=r"(r.y) : "l"(p));
  return r;
}
__device__ __forceinline__ uint2 ld_dir(const DirEntry* p) {
  uint2 r;
  asm volatile("ld.global.v2.u32 {%0,%1}, [%2];" : "=r"(r.x), "=r"(r.y) : "l"(p));
  return r;
}
__device__ __forceinline__ u32 ld_relaxed_u32(const u32* p) {
  u32 r;
  asm volatile("ld.relaxed.gpu.global.u32 %0, [%1];" : "=r"(r) : "l"(p) : "memory");
  return r;
}
__device__ __forceinline__ void st_relaxed_u32(u32* p, u32 v) {
  asm volatile("st.relaxed.gpu.global.u32 [%0], %1;" ::"l"(p), "r"(v) : "memory");
}
__device__ __forceinline__ void st_v4(u32* p, uint4 v) {
  asm volatile("st.global.v4.u32 [%0], {%1,%2,%3,%4};" ::"l"(p), "r"(v.x), "r"(v.y), "r"(v.z),
               "r"(v.w) : "memory");
}
__device__ __forceinline__ void prefetch_l1(const void* p) {
  asm volatile("prefetch.global.L1 [%0];" ::"l"(p));
}
__device__ __forceinline__ void prefetch_l2(const void* p) {
  asm volatile("prefetch.global.L2 [%0];" ::"l"(p));
}

// ------------------------------------------ bulk async copies (TMA engine) ----
// 1-D cp.async.bulk global -> shared with an mbarrier that counts the landed bytes:
// the staged data holds no registers while it is in flight.
__device__ __forceinline__ u32 smem_addr(const void* p) {
  return (u32)__cvta_generic_to_shared(p);
}
__device__ __forceinline__ void mbar_init(unsigned long long* b, u32 count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_addr(b)), "r"(count) : "memory");
  asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}
// order this thread's generic-proxy shared accesses before later async-proxy ones
__device__ __forceinline__ void fence_proxy_async_smem() {
  asm volatile("fence.proxy.async.shared::cta;" ::: "memory");
}
__device__ __forceinline__ void mbar_expect_tx(unsigned long long* b, u32 bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_addr(b)),
               "r"(bytes) : "memory");
}
// bytes: a multiple of 16; src and dst 16-B aligned
__device__ __forceinline__ void bulk_g2s(void* dst, const void* src, u32 bytes,
                                         unsigned long long* b) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
          smem_addr(dst)),
      "l"(src), "r"(bytes), "r"(smem_addr(b)) : "memory");
}
__device__ __forceinline__ void mbar_wait(unsigned long long* b, u32 parity) {
  const u32 a = smem_addr(b);
  u32 ok = 0;
  do {
    asm volatile(
        "{\n .reg .pred p;\n mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n"
        " selp.u32 %0, 1, 0, p;\n}" : "=r"(ok) : "r"(a), "r"(parity) : "memory");
  } while (!ok);
}

// --------------------------------------------------------------- groups -------
// A "group" is G consecutive lanes of a warp that together hold one bucket
// (16 B per lane: G = bucket_bytes/16).  Every group-collective uses the group's
// own lane mask, so groups of one warp may diverge freely.
template <int G>
struct Group {
  static constexpr int W = 4 * G;         // words per bucket
  static constexpr int BC = 2 * G - 1;    // pairs per bucket (Q15: 15 / 7 / 3)
  static constexpr int NEXT = W - 2;
  static constexpr int OWNER = W - 1;
  u32 lane;    // lane in warp
  u32 gl;      // lane in group
  u32 base;    // first warp lane of the group
  u32 mask;    // warp mask of the group
  __device__ __forceinline__ Group() {
    lane = threadIdx.x & 31u;
    gl = lane & (G - 1);
    base = lane & ~(u32)(G - 1);
    mask = (G == 32 ? 0xFFFFFFFFu : ((1u << G) - 1u)) << base;
  }
  __device__ __forceinline__ u32 ballot(bool p) const {
    return (__ballot_sync(mask, p) >> base) & (G == 32 ? 0xFFFFFFFFu : ((1u << G) - 1u));
  }
  template <typename T>
  __device__ __forceinline__ T shfl(T v, u32 src_gl) const {
    return __shfl_sync(mask, v, base + src_gl);
  }
  __device__ __forceinline__ bool last() const { return gl == (u32)(G - 1); }
};

__device__ __forceinline__ u64 pack_pair(u32 key, u32 val) { return (u64)key | ((u64)val << 32); }

__device__ __forceinline__ u32 u4c(const uint4& x, int i) {
  return i == 0 ? x.x : i == 1 ? x.y : i == 2 ? x.z : x.w;
}

// ---------------------------------------------------------- slot layouts -------
// A bucket is G 16-B units (W = 4G words); the last unit's words z, w hold the
// next link and the owner row in both variants.
//   map (S = 0): pair i = (key, value) in words 2i, 2i+1; BC = 2G-1
//        pairs (15 per 128 B);
//   set (S = 1): key i in word i, no values; BC = 4G-2 keys (30 per
//        128 B).
// Slot k of unit uu: key word 4uu + (S ? k : 2k); the last unit has half the slots.
template <int G, int S>
struct Lay {
  static constexpr int W = 4 * G;
  static constexpr int SPU = S ? 4 : 2;  // slots per 16-B unit
  static constexpr int BC = S ? W - 2 : W / 2 - 1;
  static constexpr int NEXT = W - 2;
  static constexpr int OWNER = W - 1;
  static __device__ __forceinline__ bool has(u32 uu, int k) {
    return uu != (u32)(G - 1) || k < SPU / 2;
  }
  static __device__ __forceinline__ u32 key(const uint4& x, int k) { return u4c(x, S ? k : 2 * k); }
  static __device__ __forceinline__ u32 val(const uint4& x, int k) {
    return S ? 0u : u4c(x, 2 * k + 1);
  }
  static __device__ __forceinline__ u32 word(u32 uu, int k) { return 4 * uu + (S ? k : 2 * k); }
};

// Per-class fields of a kernel-parameter Tables, selected without dynamic indexing
// (a runtime index into a parameter array makes the compiler copy the whole struct
// to local memory).
template <typename T>
__device__ __forceinline__ T by_class(const T (&a)[kClasses], u32 c) {
  return c == 0 ? a[0] : (c == 1 ? a[1] : a[2]);
}

// Geometry of one bucket: where it lives and how many 16-B units it has.  Uniform
// layouts (A = false) fold to the compile-time Lay<G, S> (pool 0, G units); the
// adaptive layout (A = true, G = 8 lanes = the largest class) reads the size class
// from the id: class c = 2 << c units in pool c.  Slot k of unit uu exists iff
// uu < units and (uu is not the last unit or k < SPU/2); the last unit's words z, w
// hold the next link and the owner row, as in Lay.
template <int G, int S, bool A>
struct Geo {
  typedef Lay<G, S> LY;
  u32* p;     // first word of the bucket
  u32 units;  // 16-B units
  bool home;  // a home bucket (uniform layouts): not on the free stack
  __device__ __forceinline__ Geo(const Tables& t, u32 id) {
    if constexpr (A) {
      const u32 c = id >> kClassShift;
      units = 2u << c;
      p = by_class(t.pool, c) + (u64)(id & kIdxMask) * (8u << c);
      home = false;
    } else {
      // home bucket r (id 2^31 | r) lies 2^31 buckets after the pool base
      // (VmmArray::reserve_pair), so one formula addresses both
      units = G;
      home = (id & kHomeBit) != 0;
      p = t.pool[0] + (u64)id * LY::W;
    }
  }
  __device__ __forceinline__ u32 words() const { return 4 * units; }
  __device__ __forceinline__ u32 next_word() const { return 4 * units - 2; }
  __device__ __forceinline__ u32 owner_word() const { return 4 * units - 1; }
  __device__ __forceinline__ bool has(u32 uu, int k) const { return has_u(units, uu, k); }
  __device__ __forceinline__ u32 bc() const { return bc_u(units); }
  // the same from a unit count alone (no pointer arithmetic)
  static __device__ __forceinline__ bool has_u(u32 units, u32 uu, int k) {
    if constexpr (A) return uu < units && (uu != units - 1 || k < LY::SPU / 2);
    else return LY::has(uu, k);
  }
  static __device__ __forceinline__ u32 bc_u(u32 units) {  // slots per bucket (Q15)
    if constexpr (A) return S ? 4 * units - 2 : 2 * units - 1;
    else return LY::BC;
  }
};

// Head of chain j of a row from its directory entry: uniform layouts start chain 0 in
// the row's home bucket and chain j >= 1 at xbase + j - 1; adaptive: base + j.
template <bool A>
__device__ __forceinline__ u32 chain_head(u32 base, u32 row, u32 j) {
  if constexpr (A) return base + j;
  else return j == 0 ? (kHomeBit | row) : base + j - 1;
}

// units of a bucket id (no pool access)
template <int G, bool A>
__device__ __forceinline__ u32 units_of(u32 id) {
  if constexpr (A) return 2u << (id >> kClassShift);
  else return (u32)G;
}

// Degree-adaptive layout (adaptive = 1): the row gets the
// smallest size class whose single bucket holds its hint at the load factor
// (32 B: hint <= lf*Bc_0, 64 B: hint <= lf*Bc_1), else 128-B buckets sized by the
// same rule.  Returns #buckets | class << 40 (kNbMask selects the count).
__device__ __forceinline__ u64 class_size(u64 hint, u32 lf_milli, u32 set) {
  for (u32 c = 0; c + 1 < (u32)kClasses; ++c) {
    const u64 bcc = set ? (8u << c) - 2 : (4u << c) - 1;
    if (hint * 1000 <= (u64)lf_milli * bcc) return 1ull | ((u64)c << 40);
  }
  const u64 den = (u64)lf_milli * (set ? 30u : 15u);
  const u64 b = (hint * 1000 + den - 1) / den;
  return (b ? b : 1ull) | ((u64)(kClasses - 1) << 40);
}

// layout code passed to the launchers: G | set << 5 | adaptive << 6
#define DG_LAY(G, S) ((G) | ((S) << 5))
#define DG_LAYA(G, S, A) ((G) | ((S) << 5) | ((A) << 6))
#define DG_ADAPTIVE_BIT 64
#define DG_FOR_LAYOUTS(X) X(2, 0) X(4, 0) X(8, 0) X(2, 1) X(4, 1) X(8, 1)
// every layout incl. the adaptive ones (G = 8 lanes, runtime class)
#define DG_FOR_LAYOUTS_A(X) \
  X(2, 0, 0) X(4, 0, 0) X(8, 0, 0) X(2, 1, 0) X(4, 1, 0) X(8, 1, 0) X(8, 0, 1) X(8, 1, 1)

}  // namespace dg
