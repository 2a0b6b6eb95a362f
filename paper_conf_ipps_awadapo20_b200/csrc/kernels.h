// kernels.h — host-callable launchers of the sm_100a kernels.
#pragma once
#include <cstdint>
#include <functional>
#include <cuda_runtime.h>

#include "dg_common.cuh"

namespace dg {

constexpr int kEdgeBlock = 256;
// rows with more base buckets than this are walked by a whole block (export, stats)
constexpr u32 kBigRowBuckets = 32;
// rows with more neighbours than this are oriented by a whole block (TC)
constexpr u32 kBigRowDegree = 1024;

// process-wide count of kernels launched by the library (dg_profile.launches)
void note_kernel(int n);
uint64_t kernel_launches();

struct EdgeBatch {
  const u32* src;
  const u32* dst;
  const u32* w;       // insert only, nullable
  u64 n;              // entries in src/dst/w
  const u64* idx;     // nullable: op ids to process (retry list)
  u64 n_ops;          // ops to process (n, 2n for undirected mirror, or |idx|)
  u64* retry_out;     // insert: op ids that found no free bucket (first retry_cap of them)
  u64 retry_cap;      // capacity of retry_out (0: the launch cannot run out of buckets)
  u32 epoch;          // batch epoch (validation)
  u64 nv;             // global vertex capacity (query range check)
  uint8_t* found;     // query
  u32* wout;          // query, nullable
  u32 reuse_tombstones;  // insert: install new keys in the first tombstone
  u32 chunk;             // insert: buckets per per-warp allocation chunk (set by the launcher)
  u32 sorted_path;       // insert: k_validate checked this epoch's sources for sortedness;
                         // a src-sorted batch runs k_insert_sorted (a3), others k_edges
  u32 excl_chains;       // k_insert_sorted: rows with at most this many chains are owned
  u32* pub;              // insert, uniform layouts: when set, the last block of k_edges
                         // does the allocator fixup and publishes to pub (small batches:
                         // one launch instead of two)
  u32 fuse_validate;     // insert / delete of a small batch (one pass of the grid): the
                         // kernel validates the batch itself (k_validate's job) before a
                         // grid barrier, instead of a separate launch
};
// largest batch (ops) whose insert / delete validates inside the probe launch
constexpr u64 kFuseValidateMaxOps = 1ull << 18;

// `lay` = DG_LAYA(G, S, A): G 16-B units per bucket, S = 1 for the set variant, A = 1
// for the degree-adaptive layout (G = 8 lanes, size class per bucket id)
// (keys only); launchers that take `G` are layout-independent.
// edge ops (kernels_edges.cu)
// locality order of a delete batch (kernels_order.cu): partitions by local row >> shift,
// at most kMaxOrderParts partitions of 2^shift rows
// (measured on cfg2 / cfg3 2^24 deletes, profiles/r02/order/partbits.txt: at most
// 256 / 128 / 64 / 32 partitions -> scatter 122 / 79 us, delete call 0.711 / 0.673 /
// 0.670 / 0.665 ms on cfg2, 0.772 / 0.714 / 0.702 ms on cfg3; 64 keeps a partition's
// rows within L2 on cfg3's 24 M rows)
#ifndef DG_ORDER_PART_BITS
#define DG_ORDER_PART_BITS 6
#endif
constexpr u32 kOrderPartBits = DG_ORDER_PART_BITS;
constexpr u32 kMaxOrderParts = 256;
u32 order_shift(u64 rows);
size_t order_scratch_bytes(int sms);
cudaError_t launch_order(const u32* src, const u32* dst, const u32* w, u64 n, bool mirror, u64 rows,
                         u32 nranks, void* scratch, u32* osrc, u32* odst, u32* ow, u64 nv,
                         u32 epoch, DevCtl* ctl, const std::function<cudaError_t()>& between,
                         int sms, cudaStream_t s);
cudaError_t launch_validate(const u32* src, const u32* dst, u64 n, u64 nv, u32 epoch, DevCtl* ctl,
                            int sms, cudaStream_t s);
cudaError_t launch_insert(int lay, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s);
cudaError_t launch_delete(int lay, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s);
cudaError_t launch_query(int lay, const Tables& t, const EdgeBatch& a, int sms, cudaStream_t s);
// after an insert launch: free stack / cursors; hot_out (mapped host, nullable)
// receives {hot_count, hot_pairs, bump[3], epoch} (kernels_edges.cu publish())
cudaError_t launch_fixup_alloc(const Tables& t, u32* hot_out, u32 epoch, cudaStream_t s);
u64 max_groups(int G, int sms);
// buckets an insert launch of n_ops ops may take beyond those it links
u64 spare_bound(u64 n_ops, int ncls, int G, int sms);

// graph structure (kernels_graph.cu)
// nb[r] for rows r in [0, count): initial bucket count from a hint,
//   packed as #buckets | class << 40 (uniform layouts: class 0; adaptive: the size
//   class rule of class_size()).
//   hint source: hints_global[(row0 + r) * nranks + rank] if hints_global, else
//   hints_local[r] if hints_local, else 0.
cudaError_t launch_initial_buckets(u64* nb, u64 count, u64 row0, const u32* hints_global,
                                   const u32* hints_local, u32 nranks, u32 rank, u32 lf_milli,
                                   u32 bc, u32 adaptive, u32 set, cudaStream_t s);
// off[r] = sum over r' < r of the class-c buckets of nbc[r'] (count + 1 entries)
// (home = 1: uniform layouts, chain 0 in the home bucket: nb - 1 pool buckets per row)
cudaError_t scan_class_offsets(const u64* nbc, u64 count, u32 c, u32 home, u64* off, void** temp,
                               size_t* temp_bytes, cudaStream_t s);
// out[i] = sum of in[0..i) for i < count (temp storage grows as needed)
cudaError_t scan_exclusive_u64(const u64* in, u64* out, u64 count, void** temp,
                               size_t* temp_bytes, cudaStream_t s);
// where the base buckets of new rows go, per size class
struct ClassBases {
  const u64* off[kClasses];  // per-row offsets within the class's new range
  u32 base0[kClasses];       // first bucket index of the class's new range
  u32 words[kClasses];       // words per bucket of the class
};
// dir[row] = {class << 30 | base0[c] + off[c][r], #buckets}, row = rows ? rows[r] :
// row0 + r; owner word of each base bucket = row (rows != NULL: re-sizing, which also
// clears the row's hot flag)
cudaError_t launch_init_rows(const Tables& t, u64 row0, u64 count, const u32* rows,
                             const u64* nbc, const ClassBases& cb, cudaStream_t s);
// new-row hints for vertex insertion (scatter, max over duplicates)
cudaError_t launch_scatter_hints(u32* hint_new, u64 row0, u64 count, const u32* ids,
                                 const u32* hints, u64 n, u32 nranks, u32 rank, cudaStream_t s);
cudaError_t launch_max_id(const u32* ids, u64 n, u32* out, cudaStream_t s);

cudaError_t launch_degrees(const Tables& t, u32* out, cudaStream_t s);
cudaError_t launch_export_offsets(const Tables& t, u64* ro, void** temp, size_t* temp_bytes,
                                  cudaStream_t s);
// big: scratch u32[2 + rows] (hub-row list)
cudaError_t launch_export_fill(int lay, const Tables& t, const u64* ro, u32* dst, u32* w, u32* big,
                               int sms, cudaStream_t s);

struct StatsOut {
  unsigned long long base_buckets, linked_buckets, live, tombs, max_chain;
  unsigned long long slots, bytes;  // key slots / bytes of the linked buckets
};
cudaError_t launch_stats(int lay, const Tables& t, StatsOut* out, u32* big, int sms, cudaStream_t s);

// structural invariants (kernels_check.cu); field order = dg_invariants (include/dg.h)
struct InvariantsOut {
  unsigned long long rows, chains, buckets, live_pairs, tombstones;
  unsigned long long empty_not_suffix, misplaced_keys, duplicate_keys, self_loops,
      keys_out_of_range, owner_mismatch, degree_mismatch, broken_chains, dup_unchecked_chains;
  unsigned long long first_bad_row;
};
cudaError_t launch_check(int lay, const Tables& t, u64 nv, u32 rank, InvariantsOut* out, int sms,
                         cudaStream_t s);

// vertex deletion (kernels_graph.cu)
// coarse filter of the deleted-vertex bitmap (bit = id >> fshift), kept in shared
// memory by the purge sweep
constexpr u32 kVdelFilterBits = 1u << 17;
cudaError_t launch_vdel_mark(const u32* ids, u64 n, u64 nv, u32 epoch, u32* bitmap, u32* filter,
                             u32 fshift, u32* dedup, DevCtl* ctl, u32 nranks, u32 rank, int sms,
                             cudaStream_t s);
cudaError_t launch_vdel_sweep(int lay, const Tables& t, const u32* bitmap, const u32* filter,
                              u32 fshift, u32 epoch, int sms, cudaStream_t s);
// nbarr[k] = base buckets of the k-th distinct deleted vertex (0 past the count), k <= n_max
cudaError_t launch_vdel_nb(const Tables& t, const u32* dedup, u64 n_max, u64* nbarr, int sms,
                           cudaStream_t s);
cudaError_t launch_vdel_neighbors(int lay, const Tables& t, const u32* dedup, const u64* boff,
                                  u32 epoch, int sms, cudaStream_t s);
cudaError_t launch_vdel_clear(int lay, const Tables& t, const u32* dedup, const u64* boff, u32 epoch,
                              int sms, cudaStream_t s);

// triangle counting consumer (kernels_tc.cu)
cudaError_t launch_tc_orient_count(const Tables& t, const u64* ro, const u32* dst, u32 part,
                                   u32 nparts, u64* ocnt, u32* big, int sms, cudaStream_t s);
cudaError_t launch_tc_orient_fill(const Tables& t, const u64* ro, const u32* dst, u32 part,
                                  u32 nparts, const u64* oro, u32* oadj, u32* oend,
                                  const u32* big, int sms, cudaStream_t s);
cudaError_t launch_tc_flat_prepare(const u32* oadj, const u32* oend, const u32* order, u64 n_units,
                                   uint2* list, u64* woff, unsigned long long* n_list_dev,
                                   u64* n_list, void** temp, size_t* temp_bytes, cudaStream_t s);
u64 tc_chunk_count(u64 wedges);
cudaError_t launch_tc_wedges_flat(int lay, const Tables& t, const u32* oadj, const uint2* list,
                                  const u64* woff, u32* chunk_k,
                                  const unsigned long long* n_list_dev,
                                  unsigned long long* count, int sms, cudaStream_t s);
cudaError_t launch_tc_probe_order(const u32* oadj, u64 n_units, u64 rows, u32* keys, u32* vals,
                                  const u32** perm, void** temp, size_t* temp_bytes,
                                  cudaStream_t s);
cudaError_t launch_tc_wedges(int lay, const Tables& t, const u32* oadj, const u32* oend,
                             const u32* perm, u64 n_units,
                             unsigned long long* count, int sms, cudaStream_t s);

// per-vertex re-sizing of long-chained tables (kernels_rehash.cu)
// flush = 0: re-size for long chains (room to double); 1: tombstone flush (the
// initial-size rule for the live keys)
cudaError_t launch_hot_sizes(const Tables& t, u32 n, u32 lf_milli, u32 bc, u32 flush, u32 adaptive,
                             u32 set, u64* nbnew, u64* nbold, u64* degs, cudaStream_t s);
// rows holding a tombstone -> hot flags / hot list (tombstone flush)
cudaError_t launch_tomb_sweep(int lay, const Tables& t, int sms, cudaStream_t s);
cudaError_t launch_hot_export(int lay, const Tables& t, u32 n, const u64* obo,
                              unsigned long long* cursor, u32* osrc, u32* odst, u32* ow, u32 rank,
                              int sms, cudaStream_t s);
cudaError_t launch_hot_release(int lay, const Tables& t, u32 n, const u64* obo, int sms,
                               cudaStream_t s);

}  // namespace dg
