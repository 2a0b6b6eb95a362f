/*
 * include/dg.h — C ABI of the B200-native dynamic graph library (libdg.so).
 *
 * The operation set is the paper's statement of the problem, §II-A
 * P:L166-196 ("Dynamic Graphs on the GPU", Awad, Ashkiani, Porumbescu, Owens,
 * IPDPS 2020):
 *   1) retrieve A_u                 -> dg_export_adjacency, dg_degrees
 *   2) insert vertex u with edges   -> dg_insert_vertices + dg_insert_edges
 *   3) delete vertex u              -> dg_delete_vertices
 *   4) insert edge <u,v,w>          -> dg_insert_edges      (Alg. 1)
 *   5) delete edge <u,v,w>          -> dg_delete_edges
 *   Search_Au(v) / edgeExist        -> dg_query_edges
 *   bulk build with known degrees   -> dg_create(hints) + one dg_insert_edges
 *   undirected graphs               -> dg_config.directed = 0
 * Each adjacency list A_u is a hash table of buckets (§IV-A); the
 * triangle-count consumer of §VI-C is dg_triangle_count.
 *
 * Conventions (all calls):
 *  - Return codes only (dg_status); nothing is thrown or aborted across the ABI.
 *  - IDs and weights are uint32.  Vertex IDs must be < 2^32-2 (0xFFFFFFFE and
 *    0xFFFFFFFF are the library's EMPTY / TOMBSTONE sentinels).  Weights are
 *    opaque 32-bit values (bit-cast floats if needed); a NULL weight array
 *    stores 0.  There is no floating point on the path.
 *  - Pointers marked "buffer" may be DEVICE memory on the handle's GPU
 *    (stream-ordered: the call enqueues work on `stream` and returns; the
 *    caller keeps the memory alive until that work completes) or HOST memory
 *    (pageable or pinned: the call stages it through library-owned device
 *    buffers and returns after every host output has been written and every
 *    host input has been copied, so host buffers may be reused on return).  A
 *    single-GPU dg_insert_edges / dg_delete_edges with host inputs and no count
 *    requested returns once its batch is uploaded and validated (the status is
 *    the call's return value) and leaves the mutation kernel running on
 *    `stream`, where later calls are ordered behind it; the upload of the next
 *    call overlaps it.  The caller owns all batch and result buffers; the
 *    library owns all table memory.
 *  - `stream` is a cudaStream_t (NULL = legacy default stream).
 *  - Phase-concurrent model: calls on one handle must be
 *    serialised by the caller (one host thread, one stream at a time); a batch
 *    holds one kind of operation; a query batch sees the state after every
 *    earlier batch enqueued on the stream.
 *  - Validation is all-or-nothing: if any src/dst/id of a mutating batch is
 *    >= the vertex capacity, the batch is rejected with no mutation
 *    (DG_ERR_VERTEX_OUT_OF_RANGE).  The check runs on the device; the status
 *    is returned by the call itself when the call has host outputs (or host
 *    buffers), otherwise by the next dg_batch_status().
 *  - A CUDA (or NCCL) failure makes the handle sticky-bad: every later call
 *    returns DG_ERR_BAD_STATE.
 *  - Multi-GPU (nranks > 1, one process per GPU): the graph is sharded by source
 *    vertex, owner(u) = u mod nranks, local row = u / nranks.  Every call that
 *    takes a batch is COLLECTIVE: all ranks call it in the same order, each with
 *    its own slice (n may differ, may be 0); the union of the slices is the
 *    batch.  Exports and degrees cover the calling rank's local rows.
 */
#ifndef DG_H_
#define DG_H_

#include <stddef.h>
#include <stdint.h>

#if defined(__GNUC__)
#define DG_API __attribute__((visibility("default")))
#else
#define DG_API
#endif

#ifdef __cplusplus
extern "C" {
#endif

typedef struct dg_graph_s* dg_graph;
/* In-process rank group (see dg_group_create). */
typedef struct dg_group_s* dg_group;

typedef enum dg_status {
  DG_OK = 0,
  DG_ERR_INVALID_ARGUMENT = 1,    /* NULL required pointer, bad config, n too large */
  DG_ERR_VERTEX_OUT_OF_RANGE = 2, /* an ID >= capacity: batch rejected, graph unchanged */
  DG_ERR_OUT_OF_MEMORY = 3,       /* table pool could not grow */
  DG_ERR_CUDA = 4,                /* CUDA runtime/driver error (handle becomes bad) */
  DG_ERR_NCCL = 5,                /* NCCL error (handle becomes bad) */
  DG_ERR_BAD_STATE = 6,           /* handle unusable after an earlier CUDA/NCCL error */
  DG_ERR_UNSUPPORTED = 7          /* configuration not supported by this build */
} dg_status;

/* Graph configuration.  Initialise with dg_config_init(). */
typedef struct dg_config {
  uint32_t struct_size;   /* sizeof(dg_config), ABI versioning */
  float load_factor;      /* target keys per bucket slot for the initial bucket count,
                             default 0.7; used as round(lf*1000)/1000 */
  uint32_t bucket_bytes;  /* 128 (default, 15 pairs = the paper's Bc),
                             64 (7 pairs) or 32 (3 pairs); ignored with DG_FLAG_ADAPTIVE */
  uint32_t directed;      /* 1 (default); 0 = every edge op is applied in both
                             directions */
  uint64_t pool_bytes;    /* initial overflow-bucket pool beyond the base buckets;
                             0 = automatic.  The pool grows on demand. */
  int32_t device;         /* CUDA device ordinal; -1 = current device */
  int32_t rank;           /* this process's rank, 0 <= rank < nranks */
  int32_t nranks;         /* number of GPUs the graph is sharded over (1 = single GPU) */
  uint32_t flags;         /* DG_FLAG_* bits, default 0 */
  const void* nccl_unique_id; /* 128-byte ncclUniqueId from dg_get_unique_id() on rank 0,
                                 broadcast by the caller; NULL when nranks == 1 or when
                                 `group` is set */
  dg_group group;         /* in-process rank group (dg_group_create) instead of NCCL:
                             the nranks ranks are host threads of this process; NULL =
                             one process per rank over NCCL */
} dg_config;

/* dg_config.flags: new keys are installed in the first tombstone of their chain by
 * default (the two-stage insert the paper offers as an option; results
 * are identical, chains stop growing under insert/delete churn).  This flag selects
 * the paper's default append-only policy: tombstones are never reused. */
#define DG_FLAG_NO_TOMBSTONE_REUSE 1u
/* Diagnostic: route a single-GPU graph (nranks == 1) through the multi-GPU batch
 * router over a 1-rank NCCL communicator (exercises partition / exchange / answer
 * return on one GPU). */
#define DG_FLAG_FORCE_ROUTER 2u
/* Set variant: the per-vertex tables hold keys only, twice as many
 * per bucket (30 per 128 B, 14 per 64 B, 6 per 32 B), for unweighted graphs and
 * triangle counting.  Weights are not stored: dg_insert_edges ignores
 * `weight`, dg_query_edges reports weight 0 for every hit, dg_export_adjacency
 * writes weight 0.  Membership results are those of the map variant. */
#define DG_FLAG_SET 4u
/* Degree-adaptive bucket sizes (the paper's future work,
 * "hash tables with varying slab sizes may better suit load balancing in
 * scale-free graphs").  Each vertex's table uses one of three bucket sizes, chosen
 * from its degree hint: the smallest bucket that holds the hint at the load factor
 * (32 B = 3 pairs for hints <= lf*3, 64 B = 7 pairs for hints <= lf*7), else 128-B
 * buckets (15 pairs) sized by the usual rule.  A vertex without a hint starts with
 * one 32-B bucket; the per-vertex re-sizing (long chains) picks the size class again
 * for twice the degree, so growing vertices move up to larger buckets.  Each size
 * class has its own bucket pool and free stack.  `bucket_bytes` is ignored.  Results
 * are those of every other layout. */
#define DG_FLAG_ADAPTIVE 8u
/* Multi-GPU batch routing through the copy exchange (partition into a local send
 * buffer, grouped send/recv, receive buffer) instead of the default fused exchange
 * (one kernel partitions the batch and stores every op straight into its owner's
 * NVLink-mapped receive window).  Results are identical; for A/B runs and tests.
 * The environment variable DG_ROUTER=nccl has the same effect. */
#define DG_FLAG_COPY_EXCHANGE 16u

/* Memory / structure statistics (Fig. 2b/c quantities). */
typedef struct dg_stats {
  uint64_t local_rows;        /* rows (vertices) held by this rank */
  uint64_t base_buckets;      /* buckets allocated at create / vertex insertion */
  uint64_t overflow_buckets;  /* chained buckets currently linked into tables */
  uint64_t free_buckets;      /* buckets on the free stack */
  uint64_t pool_buckets;      /* buckets mapped in the pool (sum over size classes) */
  uint64_t bump_buckets;      /* high-water mark: buckets ever handed out (home, base and
                                 chained; sum over size classes) */
  uint64_t live_pairs;        /* stored edges (sum of degrees) */
  uint64_t tombstones;        /* deleted-key slots not yet reclaimed */
  uint64_t max_chain;         /* longest bucket chain (in buckets) */
  uint64_t pool_bytes;        /* bytes of table memory mapped (pools + directory + free
                                 stacks): capacity, including the worst-case reservation */
  double load_factor;         /* live_pairs / key slots of the linked (base+overflow)
                                 buckets (Q14) */
  double utilization;         /* live_pairs * 8 B / table_bytes (Fig. 2c) */
  uint64_t exchange;          /* batch routing: 0 = none (single GPU), 1 = NCCL all-to-all,
                                 2 = fused partition + peer stores into NVLink-mapped windows */
  uint64_t table_bytes;       /* bytes of the linked (base+overflow) buckets */
  uint64_t bump_bytes;        /* bytes of all buckets ever handed out, home buckets included
                                 (what the streaming purge / tombstone sweeps read) */
} dg_stats;

/* Fills defaults: load_factor 0.7, bucket_bytes 128, directed 1, pool_bytes 0,
 * device -1, rank 0, nranks 1. */
DG_API void dg_config_init(dg_config* cfg);

/* Human-readable name of a status code (static string). */
DG_API const char* dg_status_string(dg_status s);

/* Multi-GPU bootstrap: writes a 128-byte ncclUniqueId to out128 (host memory).
 * Call on rank 0 only, then broadcast it (e.g. over a torch process group). */
DG_API dg_status dg_get_unique_id(void* out128);

/* In-process rank group: lets `nranks` host threads of ONE process act as the ranks
 * of a sharded graph (each thread creates its own handle with cfg.group = the group,
 * cfg.rank = its rank, cfg.nranks = nranks, and then makes every collective call
 * with its own slice, exactly as separate processes would).  Ranks may share one
 * GPU or use several (peer access is enabled where the GPUs allow it).  Each rank
 * must use its own stream, created non-blocking (cudaStreamNonBlocking, as torch
 * streams are): the fused exchange spins on the device until every rank's partition
 * kernel has stored its ops, so ranks serialised on one stream would wait out the
 * exchange timeout.  Collectives meet at a host barrier (timeout 120 s, then
 * DG_ERR_NCCL and the handle goes bad).  The group must outlive its handles.
 * Host-only object: creating it needs no GPU. */
DG_API dg_status dg_group_create(int32_t nranks, dg_group* out);
DG_API dg_status dg_group_destroy(dg_group group);

/* Create a graph of `num_vertices` vertices (global capacity; IDs
 * 0..num_vertices-1 all exist, with empty adjacency lists).
 *   degree_hints: buffer of num_vertices uint32 indexed by global vertex ID, or
 *     NULL.  Vertex u gets max(1, ceil(hint_u / (lf * Bc))) base buckets, one
 *     bucket if its hint is 0 or hints are NULL; all base
 *     buckets come from one bulk allocation.  Hints affect only
 *     performance, never results.
 *   *out receives the handle.  At nranks > 1 this call is collective. */
DG_API dg_status dg_create(const dg_config* cfg, uint64_t num_vertices, const uint32_t* degree_hints,
                    void* stream, dg_graph* out);

/* Destroy the handle and release all table memory (synchronises the device). */
DG_API dg_status dg_destroy(dg_graph g);

/* Global vertex capacity and the number of rows held by this rank. */
DG_API dg_status dg_num_vertices(dg_graph g, uint64_t* num_vertices, uint64_t* local_rows);

/* Batched edge insertion (Alg. 1).
 *   src, dst, weight: buffers of n uint32 (weight may be NULL -> 0).
 *   Self-loops are dropped (Alg1:L3).  An existing key (u,v) gets the new weight
 *   ("replace"); if (u,v) occurs more than once in the batch, the
 *   stored weight is one of the batch's weights for it (Q1).
 *   n_added (host, nullable): number of keys that did not exist before the batch;
 *   when non-NULL the call synchronises `stream` and also returns the batch's
 *   validation status. */
DG_API dg_status dg_insert_edges(dg_graph g, const uint32_t* src, const uint32_t* dst,
                          const uint32_t* weight, uint64_t n, uint64_t* n_added, void* stream);

/* Batched edge deletion by key (u,v) (weights are not matched, Q4).
 *   n_removed (host, nullable): number of keys that existed (a key deleted twice in
 *   the batch counts once); non-NULL synchronises. */
DG_API dg_status dg_delete_edges(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                          uint64_t* n_removed, void* stream);

/* Batched edge-existence query (edgeExist).
 *   found: buffer of n uint8, 1 if (src[i], dst[i]) is an edge, else 0.
 *   weight_out: buffer of n uint32 (nullable): the stored weight, 0 on a miss.
 *   An out-of-range ID answers 0 for that query and reports
 *   DG_ERR_VERTEX_OUT_OF_RANGE for the batch. */
DG_API dg_status dg_query_edges(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                         uint8_t* found, uint32_t* weight_out, void* stream);

/* Vertex insertion: grows the vertex capacity to
 * max(capacity, max(ids)+1).  New vertices get empty tables sized from
 * degree_hints (buffer of n uint32 parallel to ids, nullable).  IDs that already
 * exist are a no-op (Q12).  Their edges are then added with dg_insert_edges.
 * Synchronises `stream` (the new capacity must be known on the host). */
DG_API dg_status dg_insert_vertices(dg_graph g, const uint32_t* ids, uint64_t n,
                             const uint32_t* degree_hints, void* stream);

/* Vertex deletion (Alg. 2): for every u in ids,
 * A_u is emptied (its chained buckets return to the allocator, its degree := 0)
 * and every edge (x, u) is removed from every table before the call's stream
 * work completes.  Duplicate IDs are idempotent; IDs stay valid (Q10, Q11). */
DG_API dg_status dg_delete_vertices(dg_graph g, const uint32_t* ids, uint64_t n, void* stream);

/* Adjacency export (retrieve A_u for all local rows as CSR).
 *   row_offsets: buffer of local_rows+1 uint64 (required).
 *   dst, weight: buffers of `capacity` uint32 (nullable: size query only).
 *   *n_edges (host, required) receives the number of stored edges.  If
 *   dst != NULL and capacity < *n_edges, returns DG_ERR_INVALID_ARGUMENT and
 *   writes only row_offsets.  Rows are unsorted within themselves.
 *   Synchronises `stream`. */
DG_API dg_status dg_export_adjacency(dg_graph g, uint64_t* row_offsets, uint32_t* dst,
                              uint32_t* weight, uint64_t capacity, uint64_t* n_edges,
                              void* stream);

/* Exact out-degree of each local row: buffer of local_rows
 * uint32. */
DG_API dg_status dg_degrees(dg_graph g, uint32_t* out, void* stream);

/* Structure / memory statistics (synchronises). */
DG_API dg_status dg_get_stats(dg_graph g, dg_stats* out, void* stream);

/* Status of the most recent asynchronous batches since the last call
 * (synchronises): DG_ERR_VERTEX_OUT_OF_RANGE if any was rejected, else DG_OK. */
DG_API dg_status dg_batch_status(dg_graph g, void* stream);

/* Tombstone flush ("Tombstones can later be completely flushed out of
 * the data structure, if required"): every table holding a tombstone is rebuilt
 * compactly — its live pairs are re-inserted into a fresh base range sized by the
 * initial-bucket rule for its current degree and all of its old
 * buckets go to the free stack.  The logical graph is unchanged.  Rows are found
 * by one streaming pass over the allocated buckets per round of up to 65,536 rows.
 * *rows_rebuilt (host, nullable) receives the number of rebuilt tables.  Local to
 * this rank (not collective); synchronises `stream`. */
DG_API dg_status dg_flush_tombstones(dg_graph g, uint64_t* rows_rebuilt, void* stream);

/* Triangle count of a symmetric graph (undirected mode, directed = 0) by per-vertex
 * hash intersection (§VI-C): orient every edge from lower to higher rank,
 * rank(x) = (degree, id); for every vertex u and every pair v, w of its
 * higher-ranked neighbours, probe the hash table of v for w.  Each triangle is
 * counted once.  Work is split by u mod nparts: *count (host) receives the count
 * of part `part` (0 <= part < nparts); the sum over all parts is the total (one
 * replica per GPU, the caller sums, e.g. with an all-reduce).  Synchronises.
 * Requires nranks == 1 (each GPU holds a whole replica). */
DG_API dg_status dg_triangle_count(dg_graph g, uint32_t part, uint32_t nparts, uint64_t* count,
                                   void* stream);

/* Structural invariants of the tables (debug / test; not on the hot path).  Counts
 * violations of what the lock-free insert's correctness rests on:
 *   empty_not_suffix   chains with a key after an EMPTY slot ("empty locations can
 *                      only exist at the end of each bucket's list")
 *   misplaced_keys     live keys outside the chain their hash selects
 *   duplicate_keys     repeated live keys inside a chain (fn3)
 *   self_loops, keys_out_of_range (Alg1:L3; Q7)
 *   owner_mismatch     buckets whose owner word is not their row
 *   degree_mismatch    rows whose degree differs from their live keys
 *   broken_chains      chains longer than the pool (a cycle)
 * and reports what it walked (rows, chains, buckets, live_pairs, tombstones).
 * Chains longer than 64 buckets are not checked for duplicates (counted in
 * dup_unchecked_chains).  first_bad_row = lowest local row with a violation, or
 * UINT64_MAX.  Stream-ordered after every earlier batch; synchronises `stream`.
 * Local to the calling rank. */
typedef struct dg_invariants {
  uint64_t rows, chains, buckets, live_pairs, tombstones;
  uint64_t empty_not_suffix, misplaced_keys, duplicate_keys, self_loops, keys_out_of_range,
      owner_mismatch, degree_mismatch, broken_chains, dup_unchecked_chains;
  uint64_t first_bad_row;
} dg_invariants;
DG_API dg_status dg_check_invariants(dg_graph g, dg_invariants* out, void* stream);

/* ------------------------------------------------------------ instrumentation --
 * Off by default; used by bench.py.  While enabled, every probe-kernel launch of an
 * edge batch (and the purge kernels of a vertex-deletion batch) is bracketed by
 * CUDA events on the call's stream. */
typedef struct dg_profile {
  uint64_t launches;          /* kernels launched by libdg in this process since enable */
  uint64_t kernel_launches[5];/* timed launches: [0] insert, [1] delete, [2] query,
                                 [3] vertex purge, [4] triangle-count wedge probes */
  double kernel_ms[5];        /* their summed device durations in ms */
  uint64_t last_count;        /* n_added / n_removed of the most recent insert/delete batch */
} dg_profile;

/* enable != 0 starts (and resets) instrumentation; 0 stops it. */
DG_API dg_status dg_profile_enable(dg_graph g, int enable);
/* Reads the counters (synchronises `stream`). */
DG_API dg_status dg_profile_read(dg_graph g, dg_profile* out, void* stream);

#ifdef __cplusplus
}
#endif

#endif /* DG_H_ */
