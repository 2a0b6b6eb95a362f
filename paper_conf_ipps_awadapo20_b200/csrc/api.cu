#include <chrono>
// api.cu — the C ABI (include/dg.h) on top of the sm_100a kernels.
#include <algorithm>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <new>

#include "graph.h"
#include "kernels.h"
#include "router.h"

using dg::u32;
using dg::u64;

namespace {

constexpr u64 kMaxVertices = 0xFFFFFFFEull;  // Q18: two sentinel values reserved
constexpr u64 kMaxBatch = 0xFFFFFFFFull;

#define DG_CK(expr)                                                                   \
  do {                                                                                \
    cudaError_t e_ = (expr);                                                          \
    if (e_ != cudaSuccess) {                                                          \
      if (std::getenv("DG_DEBUG"))                                                    \
        std::fprintf(stderr, "dg: CUDA error %s at %s:%d\n", cudaGetErrorString(e_), \
                     __FILE__, __LINE__);                                             \
      g->bad = true;                                                                  \
      return DG_ERR_CUDA;                                                             \
    }                                                                                 \
  } while (0)

#define DG_TRY(expr)                  \
  do {                                \
    dg_status s_ = (expr);            \
    if (s_ != DG_OK) return s_;       \
  } while (0)

bool is_device_ptr(const void* p) {
  if (!p) return false;
  cudaPointerAttributes a;
  if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
    cudaGetLastError();
    return false;
  }
  return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged;
}

// grow-only scratch buffer
cudaError_t ensure_buf(dg_graph_s::Buf& b, size_t bytes, bool big_slack = false) {
  if (bytes <= b.bytes) return cudaSuccess;
  if (b.p) cudaFree(b.p);
  b.p = nullptr;
  b.bytes = 0;
  // geometric headroom: buffers that track a growing graph (TC scratch, export
  // staging) are not re-allocated (cudaFree synchronises the device) every call;
  // big_slack (the triangle-count scratch, re-sized as the graph grows every dynamic
  // step): 2x — a cudaFree + cudaMalloc of a multi-GB buffer measured 40-600 ms on
  // cfg5's growing graph (DG_TRACE_TC)
  size_t want = std::max<size_t>(big_slack ? 2 * bytes : bytes + bytes / 4, 1 << 20);
  cudaError_t e = cudaMalloc(&b.p, want);
  if (e == cudaSuccess) b.bytes = want;
  return e;
}

// Input buffer: device pointers pass through; host memory is copied to a staging
// buffer (the call then becomes synchronous).
// (is_dev: the caller already knows p is device memory; -1 = ask the runtime)
dg_status stage_in(dg_graph g, int slot, const void* p, size_t bytes, cudaStream_t s,
                   const void** out, bool* host, int is_dev = -1) {
  if (!p || bytes == 0 || (is_dev >= 0 ? is_dev != 0 : is_device_ptr(p))) {
    *out = p;
    return DG_OK;
  }
  *host = true;
  DG_CK(ensure_buf(g->stage[slot], bytes));
  DG_CK(cudaMemcpyAsync(g->stage[slot].p, p, bytes, cudaMemcpyHostToDevice, s));
  *out = g->stage[slot].p;
  return DG_OK;
}

// Output buffer: device pointers pass through; host outputs get a staging buffer
// that finish_out() copies back.
dg_status stage_out(dg_graph g, int slot, void* p, size_t bytes, void** out, bool* host) {
  if (!p || bytes == 0 || is_device_ptr(p)) {
    *out = p;
    return DG_OK;
  }
  *host = true;
  DG_CK(ensure_buf(g->stage[slot], bytes));
  *out = g->stage[slot].p;
  return DG_OK;
}

dg_status finish_out(dg_graph g, void* host, const void* dev, size_t bytes, cudaStream_t s) {
  if (host && dev && host != dev && bytes)
    DG_CK(cudaMemcpyAsync(host, dev, bytes, cudaMemcpyDeviceToHost, s));
  return DG_OK;
}

dg_status ensure_copy_streams(dg_graph g) {
  for (auto& cs : g->cstream)
    if (!cs) DG_CK(cudaStreamCreateWithFlags(&cs, cudaStreamNonBlocking));
  return DG_OK;
}

// Asynchronous host input (insert / delete / query with host buffers): the bytes are
// copied on the internal upload stream into staging slot `slot` (8..15) once the
// kernels that read the slot's previous contents are done; `s` waits for the copy.
// The call can then return as soon as the copy has landed, while its kernels run
// behind the next call's upload (PCIe and HBM overlap across calls).
dg_status upload_async(dg_graph g, int slot, const void* p, size_t bytes, cudaStream_t s,
                       const void** out) {
  if (!p || bytes == 0) {
    *out = p;
    return DG_OK;
  }
  DG_TRY(ensure_copy_streams(g));
  if (!g->slot_ev[slot]) DG_CK(cudaEventCreateWithFlags(&g->slot_ev[slot], cudaEventDisableTiming));
  DG_CK(ensure_buf(g->stage[slot], bytes));
  cudaStream_t up = g->cstream[0];
  DG_CK(cudaStreamWaitEvent(up, g->slot_ev[slot], 0));
  DG_CK(cudaMemcpyAsync(g->stage[slot].p, p, bytes, cudaMemcpyHostToDevice, up));
  DG_CK(cudaEventRecord(g->slot_ev[slot], up));
  DG_CK(cudaStreamWaitEvent(s, g->slot_ev[slot], 0));
  *out = g->stage[slot].p;
  return DG_OK;
}

// after the kernels reading slots [a, b) were enqueued on s
dg_status release_slots(dg_graph g, int a, int b, cudaStream_t s) {
  for (int k = a; k < b; ++k)
    if (g->slot_ev[k]) DG_CK(cudaEventRecord(g->slot_ev[k], s));
  return DG_OK;
}

// snapshot the validation verdict (Q7) after k_validate on s, before the mutation
dg_status note_validation(dg_graph g, cudaStream_t s) {
  if (!g->val_event) DG_CK(cudaEventCreateWithFlags(&g->val_event, cudaEventDisableTiming));
  if (!g->h_fail) DG_CK(cudaMallocHost(&g->h_fail, 64));
  DG_CK(cudaMemcpyAsync(g->h_fail, &g->ctl->fail_epoch, 4, cudaMemcpyDeviceToHost, s));
  DG_CK(cudaEventRecord(g->val_event, s));
  return DG_OK;
}

dg_status validation_status(dg_graph g, u32 epoch) {
  DG_CK(cudaEventSynchronize(g->val_event));
  return *g->h_fail >= epoch && *g->h_fail != 0 ? DG_ERR_VERTEX_OUT_OF_RANGE : DG_OK;
}

dg_status read_ctl(dg_graph g, cudaStream_t s) {
  DG_CK(cudaMemcpyAsync(g->hctl, g->ctl, sizeof(dg::DevCtl), cudaMemcpyDeviceToHost, s));
  DG_CK(cudaStreamSynchronize(s));
  return DG_OK;
}

dg_status status_of(dg_graph g, u32 epoch) {
  return g->hctl->fail_epoch >= epoch && g->hctl->fail_epoch != 0 ? DG_ERR_VERTEX_OUT_OF_RANGE
                                                                   : DG_OK;
}

// the |V|-bit deleted-vertex bitmap followed by its coarse filter (kVdelFilterBits)
dg_status ensure_bitmap(dg_graph g, u64 nv) {
  const u64 words = (nv + 31) / 32 + 1 + dg::kVdelFilterBits / 32;
  if (words > g->bitmap_words) {
    if (g->bitmap) cudaFree(g->bitmap);
    g->bitmap = nullptr;
    g->bitmap_words = 0;
    DG_CK(cudaMalloc(&g->bitmap, words * 4));
    g->bitmap_words = words;
  }
  return DG_OK;
}

dg_status ensure_dedup(dg_graph g, u64 n) {
  if (n > g->dedup_cap) {
    if (g->dedup) cudaFree(g->dedup);
    g->dedup = nullptr;
    g->dedup_cap = 0;
    const u64 want = std::max<u64>(n, 4096);
    DG_CK(cudaMalloc(&g->dedup, want * 4));
    g->dedup_cap = want;
  }
  return DG_OK;
}

// spare-bucket return list of an insert launch: one entry per resident thread, plus
// (adaptive layout) one per op — a lane hands back its spare when the next chain it
// extends has another size class, which happens at most once per lost link race
dg_status ensure_ret(dg_graph g, u64 n_ops) {
  // (adaptive: chunk remainders of three classes per warp)
  const u64 want = dg::max_groups(g->G, g->sms) * (g->adaptive ? 2 : 1) + (g->adaptive ? n_ops : 0) + 64;
  if (want > g->ret_cap) {
    if (g->ret_list) DG_CK(cudaFree(g->ret_list));
    g->ret_list = nullptr;
    g->ret_cap = 0;
    DG_CK(cudaMalloc(&g->ret_list, want * 4));
    g->ret_cap = want;
  }
  return DG_OK;
}

dg_status ensure_retry(dg_graph g, int k, u64 n) {
  if (n > g->retry_cap[k]) {
    if (g->retry[k]) cudaFree(g->retry[k]);
    g->retry[k] = nullptr;
    g->retry_cap[k] = 0;
    const u64 want = std::max<u64>(n, 1 << 16);
    DG_CK(cudaMalloc(&g->retry[k], want * 8));
    g->retry_cap[k] = want;
  }
  return DG_OK;
}

size_t device_free_bytes() {
  size_t f = 0, t = 0;
  if (cudaMemGetInfo(&f, &t) != cudaSuccess) {
    cudaGetLastError();
    return 0;
  }
  return f;
}

}  // namespace

namespace dg {

void prof_mark(dg_graph g, int k, cudaStream_t s) {
  if (!g->prof) return;
  if (g->prof_pool.empty()) {  // events are created in batches, outside the common path
    for (int i = 0; i < 64; ++i) {
      cudaEvent_t e;
      if (cudaEventCreate(&e) != cudaSuccess) {
        cudaGetLastError();
        return;
      }
      g->prof_pool.push_back(e);
    }
  }
  cudaEvent_t e = g->prof_pool.back();
  g->prof_pool.pop_back();
  cudaEventRecord(e, s);
  g->prof_ev[k].push_back(e);
}

// Map more memory in the pool of size class c so that at least min_buckets buckets
// exist; new buckets are all-EMPTY (0xFF bytes: EMPTY keys/values, NIL next, NIL
// owner).  Bucket indices stay below 2^30 (the id's class bits, dg_common.cuh).
dg_status grow_pool(dg_graph g, int c, u64 min_buckets, cudaStream_t s) {
  const u64 bb = g->cbytes(c);
  const u64 max_buckets = std::min<u64>(dg::kIdxMask, g->pool[c].reserved() / bb);
  if (min_buckets > max_buckets) return DG_ERR_OUT_OF_MEMORY;
  if (min_buckets <= g->cap[c]) return DG_OK;
  static const bool debug = std::getenv("DG_DEBUG") != nullptr;
  if (debug)
    std::fprintf(stderr, "dg: pool class %d grows %u -> %llu buckets\n", c, g->cap[c],
                 (unsigned long long)min_buckets);
  cudaError_t e = g->pool[c].ensure(min_buckets * bb, 0xFF, s);
  if (e == cudaErrorMemoryAllocation) {
    cudaGetLastError();
    return DG_ERR_OUT_OF_MEMORY;
  }
  DG_CK(e);
  const u64 nb = std::min<u64>(max_buckets, g->pool[c].mapped() / bb);
  e = g->stack[c].ensure(nb * 4, -1, s);
  if (e == cudaErrorMemoryAllocation) {
    cudaGetLastError();
    return DG_ERR_OUT_OF_MEMORY;
  }
  DG_CK(e);
  g->cap[c] = (u32)nb;
  return DG_OK;
}

namespace {

// Make sure an insert launch that may allocate `need` buckets cannot fail, if
// that is cheap; returns whether the launch must run in retry mode (check for
// failed ops after the launch and re-run them after growing the pool).
// (every size class must be able to absorb the worst case: all ops of the launch
// may extend chains of one class)
// The host's bound on the bump cursors, tightened from what the insert fixup kernels
// published to mapped memory (no copy, no event): launches up to the published epoch
// are done, so bump <= published bump + the worst case of the launches after it.
void refresh_bound(dg_graph g) {
  if (g->pending_need.empty()) return;
  volatile const u32* h = g->h_hot;
  const u32 pe = h[5];
  if (pe == 0 || pe < g->pub_floor) return;  // nothing newer than the last exact read
  bool dropped = false;
  while (!g->pending_need.empty() && g->pending_need.front().first <= pe) {
    g->pending_need.pop_front();
    dropped = true;
  }
  if (!dropped) return;
  u64 rest = 0;
  for (const auto& p : g->pending_need) rest += p.second;
  for (int c = 0; c < g->ncls; ++c)
    g->bump_ub[c] = std::min<u64>(g->bump_ub[c], (u64)h[2 + c] + rest);
}

// after an exact read of the cursors (read_ctl): nothing older is pending
void bound_exact(dg_graph g) {
  for (int c = 0; c < g->ncls; ++c) g->bump_ub[c] = g->hctl->bump[c];
  g->pending_need.clear();
  g->pub_floor = g->epoch;
}

dg_status plan_capacity(dg_graph g, u64 need, cudaStream_t s, bool* retry_mode) {
  *retry_mode = false;
  refresh_bound(g);
  bool ok = true;
  for (int c = 0; c < g->ncls; ++c) ok = ok && (u64)g->cap[c] >= g->bump_ub[c] + need;
  if (ok) return DG_OK;
  static const bool trace = std::getenv("DG_TRACE_PLAN") != nullptr;
  if (trace)
    std::fprintf(stderr, "dg: plan sync epoch %u need %llu cap %u bump_ub %llu pending %zu pub %u floor %u\n",
                 g->epoch, (unsigned long long)need, g->cap[0], (unsigned long long)g->bump_ub[0],
                 g->pending_need.size(), reinterpret_cast<volatile u32*>(g->h_hot)[5], g->pub_floor);
  // exact free counts
  DG_TRY(read_ctl(g, s));
  bound_exact(g);
  static const bool no_upfront = std::getenv("DG_TEST_RETRY_PATH") != nullptr;
  // Reserve the worst case (one new bucket per op) up front when it is bounded
  // (<= 4 GB and half of free device memory): steady-state batches then never
  // synchronise.  Larger batches (bulk builds) launch in retry mode and grow by what
  // actually failed.
  u64 limit = 0;  // cudaMemGetInfo is slow: query it only when a pool must grow
  for (int c = 0; c < g->ncls; ++c) {
    const u64 free_exact = (u64)g->cap[c] - g->hctl->bump[c] + g->hctl->stack_size[c];
    // pops come from the stack first; the bump cursor moves by at most need - stack.
    // Beyond the batch's own worst case, keep headroom for several more batches of this
    // size, so that back-to-back calls do not come back here (a synchronisation)
    // before the cursors published by earlier launches catch up (refresh_bound).
    if (!limit) limit = std::min<u64>(4ull << 30, device_free_bytes() / 2);
    // (64 launches of headroom: a host running ahead of the device synchronises once
    // per 64 small batches, not once per 8 — 2^16-op inserts back to back: 81 -> 29 us
    // per call, tools/call_overhead.py; the mapped headroom is capped at 2 GB)
    const u64 room = std::max<u64>(
        std::min<u64>(64 * need, std::min<u64>(limit, 2ull << 30) / g->cbytes(c)), 65536);
    if (free_exact >= need + room) continue;
    if (free_exact >= need) {  // enough for this batch: top up the headroom if cheap
      if (!no_upfront) {
        dg_status st = grow_pool(g, c, (u64)g->cap[c] + need + room - free_exact, s);
        if (st != DG_OK && st != DG_ERR_OUT_OF_MEMORY) return st;
      }
      continue;
    }
    const u64 missing = need - free_exact;
    // (adaptive layout: the worst case is reserved in every class pool — mapped
    // capacity, not table bytes; retry mode instead made every batch synchronise and
    // grow inside the step: cfg3 insert 2.4 -> 18 ms per 2^24)
    if (!no_upfront && missing * g->cbytes(c) <= limit) {
      const u64 want = (u64)g->cap[c] + missing + std::max<u64>(missing / 4, room);
      dg_status st = grow_pool(g, c, want, s);
      if (st == DG_OK) continue;
      if (st != DG_ERR_OUT_OF_MEMORY) return st;
    }
    *retry_mode = true;
  }
  return DG_OK;
}

void note_launch(dg_graph g, u64 need, u32 epoch) {
  for (int c = 0; c < g->ncls; ++c) g->bump_ub[c] = std::min<u64>(g->cap[c], g->bump_ub[c] + need);
  g->pending_need.emplace_back(epoch, need);
}

}  // namespace

// ops a retry-mode launch records before it runs the whole batch again (128 MB)
u64 retry_cap_max() {
  static const u64 v = std::getenv("DG_TEST_RETRY_CAP")
                           ? std::strtoull(std::getenv("DG_TEST_RETRY_CAP"), nullptr, 10)
                           : (1ull << 24);
  return v;
}

dg_status prepare_insert(dg_graph g, u64 n_ops, cudaStream_t s) {
  if (n_ops == 0) return DG_OK;
  bool retry_mode = false;
  DG_TRY(plan_capacity(g, n_ops + dg::spare_bound(n_ops, g->ncls, g->G, g->sms), s, &retry_mode));
  if (retry_mode) DG_TRY(ensure_retry(g, 0, std::min<u64>(n_ops, retry_cap_max())));
  DG_TRY(ensure_ret(g, n_ops));
  return DG_OK;
}

// insert n edges already resident on this GPU (their sources are local rows)
dg_status local_insert(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n, bool mirror,
                       u32 epoch, cudaStream_t s, bool fuse_validate) {
  dg::Tables t = g->tables();
  const u64 n_ops = mirror ? 2 * n : n;
  if (n_ops == 0) return DG_OK;
  const u64 need = n_ops + dg::spare_bound(n_ops, g->ncls, g->G, g->sms);
  bool retry_mode = false;
  DG_TRY(plan_capacity(g, need, s, &retry_mode));
  // Retry mode records the ops that found no bucket, up to a bounded list (128 MB);
  // when more fail, the whole batch runs again after the pool grows (an insert batch
  // is idempotent: re-applied keys are replaced by a weight of the same batch, Q1,
  // and only keys still missing count as added).
  const u64 rcap = retry_mode ? std::min<u64>(n_ops, retry_cap_max()) : 0;
  if (rcap) DG_TRY(ensure_retry(g, 0, rcap));
  DG_TRY(ensure_ret(g, n_ops));
  t = g->tables();
  dg::EdgeBatch a{};
  a.src = src;
  a.dst = dst;
  a.w = w;
  a.n = n;
  a.idx = nullptr;
  a.n_ops = n_ops;
  a.retry_out = g->retry[0];
  a.retry_cap = rcap;
  a.reuse_tombstones = g->reuse_tombstones ? 1u : 0u;
  a.epoch = epoch;
  a.nv = g->nv;
  // src-sorted batches (k_validate's verdict for this epoch) take the same-source
  // grouped path (a3)
  static const bool no_sorted = std::getenv("DG_NO_SORTED_PATH") != nullptr;
  // (large batches only: a small batch would pay a second launch for little)
  a.sorted_path = (!no_sorted && !mirror && epoch == g->validated_epoch && n >= (1u << 18)) ? 1u : 0u;
  static const u32 excl_chains = std::getenv("DG_EXCL_CHAINS")
                                     ? (u32)std::atoi(std::getenv("DG_EXCL_CHAINS")) : 256u;
  a.excl_chains = std::min<u32>(excl_chains, 256u);  // (k_insert_sorted packs chain < 256)
  // small batches: the insert kernel's last block does the allocator fixup (one launch
  // instead of two; a large batch returns more spare buckets than one block copies fast)
  const bool fused = !g->adaptive && !retry_mode && !a.sorted_path && n_ops <= (1u << 18);
  a.pub = fused ? g->d_hot : nullptr;
  a.fuse_validate = fuse_validate ? 1u : 0u;
  prof_mark(g, PROF_INSERT, s);
  DG_CK(dg::launch_insert(g->lay, t, a, g->sms, s));
  prof_mark(g, PROF_INSERT, s);
  static const bool trace_alloc = std::getenv("DG_TRACE_ALLOC") != nullptr;
  if (trace_alloc) {  // diagnostic: allocator activity of this launch (synchronises)
    const u32 b0 = g->hctl->bump[0];
    DG_TRY(read_ctl(g, s));
    std::fprintf(stderr, "dg: insert %llu ops: pops %u/%u stack, bump %u -> %u, spares back %u\n",
                 (unsigned long long)n_ops, g->hctl->pop_count[0], g->hctl->stack_size[0], b0,
                 g->hctl->bump[0], g->hctl->ret_count);
  }
  // (the fixup also publishes the chain-length metric and the cursors)
  if (!fused) DG_CK(dg::launch_fixup_alloc(t, g->d_hot, epoch, s));
  if (!retry_mode) {
    note_launch(g, need, epoch);
    return DG_OK;
  }
  // retry mode: re-run the ops that found no free bucket after growing the pool
  int cur = 0;
  for (int round = 0;; ++round) {
    DG_TRY(read_ctl(g, s));
    bound_exact(g);
    const u64 failed = g->hctl->retry_count;
    if (failed == 0) break;
    if (round > 64) return DG_ERR_OUT_OF_MEMORY;
    for (int c = 0; c < g->ncls; ++c) {  // grow the pools that ran dry
      if (g->hctl->bump[c] < g->cap[c] && g->ncls > 1) continue;
      const u64 want = (u64)g->cap[c] + failed + dg::max_groups(g->G, g->sms) + (u64)g->cap[c] / 4;
      DG_TRY(grow_pool(g, c, want, s));
    }
    const bool whole = failed > a.retry_cap;  // the list overflowed: run the batch again
    if (std::getenv("DG_DEBUG"))
      std::fprintf(stderr, "dg: retry round %d: %llu ops found no bucket%s\n", round,
                   (unsigned long long)failed, whole ? " (whole batch again)" : "");
    const u64 next_cap = std::min<u64>(whole ? n_ops : failed, rcap);
    DG_TRY(ensure_retry(g, cur ^ 1, next_cap));
    DG_CK(cudaMemsetAsync(&g->ctl->retry_count, 0, sizeof(u32), s));
    t = g->tables();
    a.idx = whole ? nullptr : g->retry[cur];
    a.n_ops = whole ? n_ops : failed;
    a.sorted_path = 0;  // re-runs go through k_edges
    a.pub = nullptr;
    a.fuse_validate = 0;  // (validated by the first launch)
    a.retry_out = g->retry[cur ^ 1];
    a.retry_cap = next_cap;
    DG_CK(dg::launch_insert(g->lay, t, a, g->sms, s));
    DG_CK(dg::launch_fixup_alloc(t, g->d_hot, epoch, s));
    cur ^= 1;
  }
  return DG_OK;
}

// Delete batches of at least this many ops are put in locality order before their
// probe (kernels_order.cu; DG_ORDER_MIN_OPS overrides, 0 = never).  Measured break-even
// on cfg2 and cfg3 (profiles/r02/order/sweep.txt): 2^20 ops lose (0.086 -> 0.100 ms),
// 2^21 break even, 2^22 / 2^23 / 2^24 gain 6 / 10 / 15%.
u64 order_min_ops() {
  static const u64 v = std::getenv("DG_ORDER_MIN_OPS")
                           ? std::strtoull(std::getenv("DG_ORDER_MIN_OPS"), nullptr, 10)
                           : (1ull << 21);
  return v;
}

// Locality order of (src, dst[, mirror]) into g->ord: the permuted arrays, or
// *ordered = false when the batch keeps its own order.  validate: the batch is
// validated here (by the order's count pass, else k_validate); note: the verdict is
// snapshot for validation_status() right after it.
// *fused: a small batch left to the probe kernel's own validation (EdgeBatch
// fuse_validate; not when the verdict must be snapshot before the probe).
// w (nullable, insert batches): the weights, permuted with their ops into *ow.
// want: the caller's decision to order (delete_order_wanted / insert_order_wanted).
dg_status order_batch(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n, bool mirror,
                      u32 epoch, bool validate, bool note, bool want, const u32** osrc,
                      const u32** odst, const u32** ow, bool* ordered, bool* fused,
                      cudaStream_t s) {
  const u64 n_ops = mirror ? 2 * n : n;
  *ordered = want;
  *fused = false;
  if (!*ordered) {
    *fused = validate && !note && n_ops < dg::kFuseValidateMaxOps;
    if (validate && !*fused) DG_CK(dg::launch_validate(src, dst, n, g->nv, epoch, g->ctl, g->sms, s));
    if (note) DG_TRY(note_validation(g, s));
    return DG_OK;
  }
  DG_CK(ensure_buf(g->ord[0], dg::order_scratch_bytes(g->sms)));
  DG_CK(ensure_buf(g->ord[1], n_ops * 4));
  DG_CK(ensure_buf(g->ord[2], n_ops * 4));
  if (w) DG_CK(ensure_buf(g->ord[3], n_ops * 4));
  dg_status nst = DG_OK;
  auto between = [&]() -> cudaError_t {
    if (note) nst = note_validation(g, s);
    return nst == DG_OK ? cudaSuccess : cudaErrorUnknown;
  };
  const cudaError_t e = dg::launch_order(src, dst, w, n, mirror, g->rows, g->nranks, g->ord[0].p,
                                         (u32*)g->ord[1].p, (u32*)g->ord[2].p,
                                         w ? (u32*)g->ord[3].p : nullptr, g->nv, epoch,
                                         validate ? g->ctl : nullptr, between, g->sms, s);
  if (nst != DG_OK) return nst;
  DG_CK(e);
  *osrc = (const u32*)g->ord[1].p;
  *odst = (const u32*)g->ord[2].p;
  if (ow) *ow = w ? (const u32*)g->ord[3].p : nullptr;
  return DG_OK;
}

bool delete_order_wanted(dg_graph g, u64 n_ops) {
  const u64 lim = order_min_ops();
  return lim != 0 && n_ops >= lim && n_ops < (1ull << 32) && g->rows > 1;
}

// Inserts are ordered only when ops of one row rarely meet in flight: at most
// DG_ORDER_INSERT_PER_ROW (default 1.0) ops per local row on average (measured with the
// reorder untimed, tools/locality_probe.py: cfg3's 2^24 batch over 24 M rows, 0.7 per
// row, 1.50 -> 0.95 ms; cfg2's over 4.85 M rows, 3.5 per row, 1.18 -> 1.15 ms: ops
// of one row then race for the same free slot).
bool insert_order_wanted(dg_graph g, u64 n_ops);

// An insert batch of this rank (not routed): validation, then the insert — a small
// batch validates inside its insert launch (one launch instead of two; no sortedness
// verdict: the src-sorted path is for batches >= 2^18); a large batch over many rows
// is put in locality order (its count pass validates; an ordered batch is not
// src-sorted); otherwise k_validate (with the sortedness verdict) and the insert.
// note: snapshot the verdict for validation_status() (host-buffer calls).
dg_status validated_insert(dg_graph g, const u32* src, const u32* dst, const u32* w, u64 n,
                           u32 epoch, bool note, cudaStream_t s) {
  const bool mirror = !g->directed;
  const u64 n_ops = mirror ? 2 * n : n;
  if (insert_order_wanted(g, n_ops)) {
    const u32 *os = nullptr, *od = nullptr, *ow = nullptr;
    bool ordered = false, fused = false;
    DG_TRY(order_batch(g, src, dst, w, n, mirror, epoch, true, note, true, &os, &od, &ow, &ordered,
                       &fused, s));
    return local_insert(g, os, od, ow, n_ops, false, epoch, s, false);
  }
  const bool fuse = !note && n > 0 && n_ops < kFuseValidateMaxOps;
  if (!fuse) {
    DG_CK(launch_validate(src, dst, n, g->nv, epoch, g->ctl, g->sms, s));
    g->validated_epoch = epoch;
  }
  if (note) DG_TRY(note_validation(g, s));
  return local_insert(g, src, dst, w, n, mirror, epoch, s, fuse);
}

bool insert_order_wanted(dg_graph g, u64 n_ops) {
  static const double per_row = std::getenv("DG_ORDER_INSERT_PER_ROW")
                                    ? std::atof(std::getenv("DG_ORDER_INSERT_PER_ROW")) : 1.0;
  return delete_order_wanted(g, n_ops) && (double)n_ops <= per_row * (double)g->rows;
}

// validate / note: see order_batch (the router validates its batches itself)
dg_status local_delete(dg_graph g, const u32* src, const u32* dst, u64 n, bool mirror, u32 epoch,
                       cudaStream_t s, bool validate, bool note) {
  u64 n_ops = mirror ? 2 * n : n;
  if (n_ops == 0) {
    if (validate) DG_CK(dg::launch_validate(src, dst, n, g->nv, epoch, g->ctl, g->sms, s));
    if (note) DG_TRY(note_validation(g, s));
    return DG_OK;
  }
  prof_mark(g, PROF_DELETE, s);
  bool ordered = false, fused = false;
  DG_TRY(order_batch(g, src, dst, nullptr, n, mirror, epoch, validate, note,
                     delete_order_wanted(g, n_ops), &src, &dst, nullptr, &ordered, &fused, s));
  if (ordered) n = n_ops;  // explicit directed ops (mirrors expanded)
  dg::EdgeBatch a{};
  a.src = src;
  a.dst = dst;
  a.n = n;
  a.n_ops = n_ops;
  a.epoch = epoch;
  a.nv = g->nv;
  a.fuse_validate = fused ? 1u : 0u;
  DG_CK(dg::launch_delete(g->lay, g->tables(), a, g->sms, s));
  prof_mark(g, PROF_DELETE, s);
  return DG_OK;
}

dg_status local_query(dg_graph g, const u32* src, const u32* dst, u64 n, uint8_t* found, u32* wout,
                      u32 epoch, cudaStream_t s) {
  if (n == 0) return DG_OK;
  dg::EdgeBatch a{};
  a.src = src;
  a.dst = dst;
  a.n = n;
  a.n_ops = n;
  a.epoch = epoch;
  a.nv = g->nv;
  a.found = found;
  a.wout = wout;
  prof_mark(g, PROF_QUERY, s);
  DG_CK(dg::launch_query(g->lay, g->tables(), a, g->sms, s));
  prof_mark(g, PROF_QUERY, s);
  return DG_OK;
}

// Re-size the rows flagged by the insert kernel for long chains:
// export their pairs, release all their buckets, give each a fresh base range sized
// for twice its degree, and insert the pairs again.  Runs before an insert batch
// (phase-concurrent: no other batch in flight on the handle).
dg_status rehash_hot(dg_graph g, cudaStream_t s) {
  DG_TRY(read_ctl(g, s));  // exact count (the published one may lag a batch)
  return rehash_rows(g, std::min<u32>(g->hctl->hot_count, g->hot_cap), false, s);
}

// Re-build the n rows of hot_list (flush = false: long chains, sized to double;
// true: tombstone flush, sized by the initial rule for their live keys).
dg_status rehash_rows(dg_graph g, u32 n, bool flush, cudaStream_t s) {
  if (n == 0) return DG_OK;
  g->in_rehash = true;
  struct Guard {
    dg_graph g;
    ~Guard() { g->in_rehash = false; }
  } guard{g};
  const u64 m = (u64)n + 1;
  DG_CK(ensure_buf(g->rh[0], (6 + dg::kClasses) * m * 8));
  u64* nbnew = reinterpret_cast<u64*>(g->rh[0].p);  // #buckets | class << 40
  u64* nbold = nbnew + m;
  u64* degs = nbold + m;
  u64* obo = degs + m;
  u64* doff = obo + m;
  u64* cursor = doff + m;
  u64* nboff = cursor + m;  // per class: kClasses arrays of m
  dg::Tables t = g->tables();
  DG_CK(dg::launch_hot_sizes(t, n, g->lf_milli, g->BC, flush ? 1u : 0u, g->adaptive ? 1u : 0u,
                             g->set ? 1u : 0u, nbnew, nbold, degs, s));
  u64 tot[2 + dg::kClasses] = {};
  for (int c = 0; c < g->ncls; ++c) {
    DG_CK(dg::scan_class_offsets(nbnew, n, (u32)c, g->adaptive ? 0u : 1u, nboff + c * m,
                                 &g->scan_temp, &g->scan_bytes, s));
    DG_CK(cudaMemcpyAsync(&tot[2 + c], nboff + c * m + n, 8, cudaMemcpyDeviceToHost, s));
  }
  DG_CK(dg::scan_exclusive_u64(nbold, obo, m, &g->scan_temp, &g->scan_bytes, s));
  DG_CK(dg::scan_exclusive_u64(degs, doff, m, &g->scan_temp, &g->scan_bytes, s));
  DG_CK(cudaMemcpyAsync(&tot[1], doff + n, 8, cudaMemcpyDeviceToHost, s));
  if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
  g->snap_pending = false;
  DG_TRY(read_ctl(g, s));
  const u64 total_deg = tot[1];
  if (std::getenv("DG_DEBUG"))
    std::fprintf(stderr, "dg: re-sizing %u rows (%llu pairs, %llu/%llu/%llu new base buckets)\n",
                 n, (unsigned long long)total_deg, (unsigned long long)tot[2],
                 (unsigned long long)tot[3], (unsigned long long)tot[4]);
  dg::ClassBases cb{};
  u32 newbump[dg::kClasses] = {0, 0, 0};
  for (int c = 0; c < g->ncls; ++c) {
    const u64 bump0 = g->hctl->bump[c];
    if (bump0 + tot[2 + c] + 1 >= dg::kIdxMask) {  // no room: forget the flags
      DG_CK(cudaMemsetAsync(g->hot_flags, 0, g->hot_words * 4, s));
      DG_CK(cudaMemsetAsync(&g->ctl->hot_count, 0, 8, s));
      return flush ? DG_ERR_OUT_OF_MEMORY : DG_OK;
    }
  }
  for (int c = 0; c < g->ncls; ++c) {
    const u64 bump0 = g->hctl->bump[c];
    if (tot[2 + c]) DG_TRY(grow_pool(g, c, bump0 + tot[2 + c] + g->cap[c] / 8 + 65536, s));
    cb.off[c] = nboff + c * m;
    cb.base0[c] = (u32)bump0;
    cb.words[c] = g->cbytes(c) / 4;
    newbump[c] = (u32)(bump0 + tot[2 + c]);
  }
  t = g->tables();
  DG_CK(ensure_buf(g->rh[1], total_deg * 4 + 4));
  DG_CK(ensure_buf(g->rh[2], total_deg * 4 + 4));
  DG_CK(ensure_buf(g->rh[3], total_deg * 4 + 4));
  u32* osrc = reinterpret_cast<u32*>(g->rh[1].p);
  u32* odst = reinterpret_cast<u32*>(g->rh[2].p);
  u32* ow = reinterpret_cast<u32*>(g->rh[3].p);
  DG_CK(cudaMemcpyAsync(cursor, doff, n * 8, cudaMemcpyDeviceToDevice, s));
  DG_CK(dg::launch_hot_export(g->lay, t, n, obo, reinterpret_cast<unsigned long long*>(cursor), osrc,
                              odst, ow, g->rank, g->sms, s));
  DG_CK(dg::launch_hot_release(g->lay, t, n, obo, g->sms, s));
  DG_CK(dg::launch_init_rows(t, 0, n, t.hot_list, nbnew, cb, s));
  DG_CK(cudaMemcpyAsync(g->ctl->bump, newbump, 4 * dg::kClasses, cudaMemcpyHostToDevice, s));
  DG_CK(cudaMemsetAsync(g->hot_flags, 0, g->hot_words * 4, s));
  DG_CK(cudaMemsetAsync(&g->ctl->hot_count, 0, 8, s));  // hot_count, hot_pairs
  g->h_hot[0] = g->h_hot[1] = 0;
  DG_CK(cudaMemsetAsync(&g->ctl->count, 0, 8, s));
  DG_CK(cudaMemsetAsync(&g->ctl->retry_count, 0, 4, s));
  for (int c = 0; c < g->ncls; ++c) g->bump_ub[c] = std::max<u64>(g->bump_ub[c], newbump[c]);
  g->pending_need.clear();  // (synchronised above: every earlier launch is done)
  g->pub_floor = g->epoch + 1;
  // the pairs go back through the ordinary insert kernel (all keys distinct)
  DG_TRY(local_insert(g, osrc, odst, ow, total_deg, false, ++g->epoch, s));
  DG_CK(cudaStreamSynchronize(s));
  return DG_OK;
}

}  // namespace dg

// ======================================================================= C ABI ==
extern "C" {

void dg_config_init(dg_config* c) {
  if (!c) return;
  std::memset(c, 0, sizeof(*c));
  c->struct_size = sizeof(dg_config);
  c->load_factor = 0.7f;
  c->bucket_bytes = 128;
  c->directed = 1;
  c->pool_bytes = 0;
  c->device = -1;
  c->rank = 0;
  c->nranks = 1;
  c->nccl_unique_id = nullptr;
}

const char* dg_status_string(dg_status s) {
  switch (s) {
    case DG_OK: return "DG_OK";
    case DG_ERR_INVALID_ARGUMENT: return "DG_ERR_INVALID_ARGUMENT";
    case DG_ERR_VERTEX_OUT_OF_RANGE: return "DG_ERR_VERTEX_OUT_OF_RANGE";
    case DG_ERR_OUT_OF_MEMORY: return "DG_ERR_OUT_OF_MEMORY";
    case DG_ERR_CUDA: return "DG_ERR_CUDA";
    case DG_ERR_NCCL: return "DG_ERR_NCCL";
    case DG_ERR_BAD_STATE: return "DG_ERR_BAD_STATE";
    case DG_ERR_UNSUPPORTED: return "DG_ERR_UNSUPPORTED";
  }
  return "DG_ERR_UNKNOWN";
}

dg_status dg_get_unique_id(void* out128) {
  if (!out128) return DG_ERR_INVALID_ARGUMENT;
  return dg::router_unique_id(out128);
}

static void prof_clear(dg_graph g) {
  for (auto& v : g->prof_ev) {
    for (cudaEvent_t e : v) g->prof_pool.push_back(e);
    v.clear();
  }
}

static void destroy_graph(dg_graph g) {
  if (!g) return;
  cudaSetDevice(g->device);
  cudaDeviceSynchronize();
  cudaGetLastError();
  prof_clear(g);
  for (cudaEvent_t e : g->prof_pool) cudaEventDestroy(e);
  g->prof_pool.clear();
  if (g->router) dg::router_destroy(g->router);
  g->dir.release();
  g->degv.release();
  g->home.release();  // (a view into pool[0]'s reservation: before the pools)
  g->nbsv.release();
  for (auto& p : g->pool) p.release();
  for (auto& p : g->stack) p.release();
  if (g->ctl) cudaFree(g->ctl);
  if (g->hctl) cudaFreeHost(g->hctl);
  if (g->snap_event) cudaEventDestroy(g->snap_event);
  if (g->ret_list) cudaFree(g->ret_list);
  for (auto* p : g->retry)
    if (p) cudaFree(p);
  if (g->bitmap) cudaFree(g->bitmap);
  if (g->dedup) cudaFree(g->dedup);
  if (g->scan_temp) cudaFree(g->scan_temp);
  if (g->stats_dev) cudaFree(g->stats_dev);
  if (g->small_dev) cudaFree(g->small_dev);
  for (auto& b : g->stage)
    if (b.p) cudaFree(b.p);
  for (auto& a : g->tcv) a.release();
  for (auto& b : g->rh)
    if (b.p) cudaFree(b.p);
  if (g->big.p) cudaFree(g->big.p);
  if (g->hot_flags) cudaFree(g->hot_flags);
  if (g->hot_list) cudaFree(g->hot_list);
  if (g->h_hot) cudaFreeHost(g->h_hot);
  for (auto& cs : g->cstream)
    if (cs) cudaStreamDestroy(cs);
  for (cudaEvent_t e : g->slot_ev)
    if (e) cudaEventDestroy(e);
  if (g->val_event) cudaEventDestroy(g->val_event);
  if (g->h_fail) cudaFreeHost(g->h_fail);
  for (cudaEvent_t e : g->pipe_ev) cudaEventDestroy(e);
  cudaGetLastError();
  delete g;
}

// Allocate base buckets for rows [row0, row0+count) from the bump region and
// initialise their directory entries (one bulk allocation).
static dg_status add_rows(dg_graph g, u64 row0, u64 count, const u32* hints_global,
                          const u32* hints_local, u64 slack_buckets, cudaStream_t s) {
  if (count == 0) return DG_OK;
  // uniform layouts address home buckets by row in 30 bits (2^30 rows of 128 B are
  // 128 GiB: more than the tables could hold anyway)
  if (!g->adaptive && row0 + count > dg::kMaxHomeRows) return DG_ERR_UNSUPPORTED;
  u64* nb = nullptr;   // #buckets | class << 40
  u64* off = nullptr;  // per class: count + 1 offsets
  DG_CK(cudaMallocAsync(&nb, (count + 1) * 8, s));
  DG_CK(cudaMallocAsync(&off, (count + 1) * 8 * g->ncls, s));
  DG_CK(dg::launch_initial_buckets(nb, count, row0, hints_global, hints_local, g->nranks, g->rank,
                                   g->lf_milli, g->BC, g->adaptive ? 1u : 0u, g->set ? 1u : 0u, s));
  u64 total[dg::kClasses] = {0, 0, 0};
  for (int c = 0; c < g->ncls; ++c) {
    DG_CK(dg::scan_class_offsets(nb, count, (u32)c, g->adaptive ? 0u : 1u, off + c * (count + 1),
                                 &g->scan_temp,
                                 &g->scan_bytes, s));
    DG_CK(cudaMemcpyAsync(&total[c], off + c * (count + 1) + count, 8, cudaMemcpyDeviceToHost, s));
  }
  DG_TRY(read_ctl(g, s));  // also synchronises
  dg::ClassBases cb{};
  u32 newbump[dg::kClasses] = {0, 0, 0};
  for (int c = 0; c < g->ncls; ++c) {
    const u64 base0 = g->hctl->bump[c];
    dg_status st = DG_OK;
    if (base0 + total[c] + 1 >= dg::kIdxMask) st = DG_ERR_OUT_OF_MEMORY;
    if (st == DG_OK) st = dg::grow_pool(g, c, base0 + total[c] + slack_buckets, s);
    if (st != DG_OK) {
      cudaFreeAsync(nb, s);
      cudaFreeAsync(off, s);
      return st;
    }
    cb.off[c] = off + c * (count + 1);
    cb.base0[c] = (u32)base0;
    cb.words[c] = g->cbytes(c) / 4;
    newbump[c] = (u32)(base0 + total[c]);
  }
  cudaError_t e = g->dir.ensure((row0 + count) * sizeof(dg::DirEntry), 0, s);
  if (e == cudaErrorMemoryAllocation) return DG_ERR_OUT_OF_MEMORY;
  DG_CK(e);
  e = g->degv.ensure((row0 + count) * sizeof(u32), 0, s);
  if (e == cudaErrorMemoryAllocation) return DG_ERR_OUT_OF_MEMORY;
  DG_CK(e);
  if (!g->adaptive) {  // (k_init_rows writes every new home bucket and chain-count byte)
    e = g->home.ensure((row0 + count) * g->bucket_bytes, -1, s);
    if (e == cudaErrorMemoryAllocation) return DG_ERR_OUT_OF_MEMORY;
    DG_CK(e);
    e = g->nbsv.ensure(row0 + count, -1, s);
    if (e == cudaErrorMemoryAllocation) return DG_ERR_OUT_OF_MEMORY;
    DG_CK(e);
  }
  g->rows = row0 + count;
  {  // re-sizing flags: one bit per row (transient: a growth simply clears them)
    const u64 words = (g->rows + 31) / 32 + 1;
    if (words > g->hot_words) {
      if (g->hot_flags) cudaFree(g->hot_flags);
      g->hot_flags = nullptr;
      g->hot_words = 0;
      DG_CK(cudaMalloc(&g->hot_flags, words * 4));
      g->hot_words = words;
      DG_CK(cudaMemsetAsync(g->hot_flags, 0, words * 4, s));
      DG_CK(cudaMemsetAsync(&g->ctl->hot_count, 0, 8, s));
    }
  }
  DG_CK(dg::launch_init_rows(g->tables(), row0, count, nullptr, nb, cb, s));
  DG_CK(cudaMemcpyAsync(g->ctl->bump, newbump, 4 * dg::kClasses, cudaMemcpyHostToDevice, s));
  DG_CK(cudaFreeAsync(nb, s));
  DG_CK(cudaFreeAsync(off, s));
  DG_CK(cudaStreamSynchronize(s));
  for (int c = 0; c < g->ncls; ++c) g->bump_ub[c] = std::max<u64>(g->bump_ub[c], newbump[c]);
  g->pending_need.clear();  // (synchronised: every earlier launch is done)
  g->pub_floor = g->epoch + 1;
  return DG_OK;
}

dg_status dg_create(const dg_config* cfg, uint64_t num_vertices, const uint32_t* degree_hints,
                    void* stream, dg_graph* out) {
  if (!cfg || !out) return DG_ERR_INVALID_ARGUMENT;
  *out = nullptr;
  if (cfg->struct_size != sizeof(dg_config)) return DG_ERR_INVALID_ARGUMENT;
  if (num_vertices > kMaxVertices) return DG_ERR_INVALID_ARGUMENT;
  if (cfg->bucket_bytes != 32 && cfg->bucket_bytes != 64 && cfg->bucket_bytes != 128)
    return DG_ERR_INVALID_ARGUMENT;
  if (!(cfg->load_factor > 0.0f) || !(cfg->load_factor < 1000.0f)) return DG_ERR_INVALID_ARGUMENT;
  if (cfg->nranks < 1 || cfg->rank < 0 || cfg->rank >= cfg->nranks) return DG_ERR_INVALID_ARGUMENT;
  if (cfg->nranks > 1 && !cfg->nccl_unique_id && !cfg->group) return DG_ERR_INVALID_ARGUMENT;
  if (cfg->flags & ~(DG_FLAG_NO_TOMBSTONE_REUSE | DG_FLAG_FORCE_ROUTER | DG_FLAG_SET |
                     DG_FLAG_ADAPTIVE | DG_FLAG_COPY_EXCHANGE))
    return DG_ERR_INVALID_ARGUMENT;

  dg_graph g = new (std::nothrow) dg_graph_s();
  if (!g) return DG_ERR_OUT_OF_MEMORY;
  g->cfg = *cfg;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  auto fail = [&](dg_status st) {
    destroy_graph(g);
    return st;
  };
  if (cfg->device >= 0) {
    if (cudaSetDevice(cfg->device) != cudaSuccess) return fail(DG_ERR_CUDA);
    g->device = cfg->device;
  } else if (cudaGetDevice(&g->device) != cudaSuccess) {
    return fail(DG_ERR_CUDA);
  }
  cudaDeviceProp prop;
  if (cudaGetDeviceProperties(&prop, g->device) != cudaSuccess) return fail(DG_ERR_CUDA);
  g->sms = prop.multiProcessorCount;
  g->adaptive = (cfg->flags & DG_FLAG_ADAPTIVE) != 0;
  g->ncls = g->adaptive ? dg::kClasses : 1;
  g->bucket_bytes = g->adaptive ? 128u : cfg->bucket_bytes;  // adaptive: largest class
  g->G = (int)(g->bucket_bytes / 16);
  g->W = g->bucket_bytes / 4;
  g->set = (cfg->flags & DG_FLAG_SET) != 0;
  g->BC = g->set ? g->bucket_bytes / 4 - 2 : g->bucket_bytes / 8 - 1;  // Q15
  g->lay = DG_LAYA(g->G, g->set ? 1 : 0, g->adaptive ? 1 : 0);
  g->lf_milli = std::max<u32>(1, (u32)std::lround((double)cfg->load_factor * 1000.0));
  g->nranks = (u32)cfg->nranks;
  g->rank = (u32)cfg->rank;
  g->directed = cfg->directed != 0;
  g->reuse_tombstones = (cfg->flags & DG_FLAG_NO_TOMBSTONE_REUSE) == 0;
  g->nv = num_vertices;

  const size_t total_mem = prop.totalGlobalMem;
  const u64 max_rows = (kMaxVertices + g->nranks - 1) / g->nranks + 1;
  for (int c = 0; c < g->ncls; ++c) {
    if (!g->adaptive) {
      // the pool (bucket ids < 2^30) and, 2^31 buckets after its base, the home buckets
      const u64 bb = g->bucket_bytes;
      if (g->pool[c].reserve_pair(g->device, std::min<u64>(total_mem, bb << 30), bb << 31,
                                  std::min<u64>(max_rows, dg::kMaxHomeRows) * bb,
                                  g->home) != cudaSuccess)
        return fail(DG_ERR_CUDA);
    } else if (g->pool[c].reserve(g->device, total_mem) != cudaSuccess) {
      return fail(DG_ERR_CUDA);
    }
    if (g->stack[c].reserve(g->device, total_mem / g->cbytes(c) * 4 + (2u << 20)) != cudaSuccess)
      return fail(DG_ERR_CUDA);
  }
  if (g->dir.reserve(g->device, max_rows * sizeof(dg::DirEntry)) != cudaSuccess ||
      g->degv.reserve(g->device, max_rows * sizeof(u32)) != cudaSuccess ||
      (!g->adaptive && g->nbsv.reserve(g->device, std::min<u64>(max_rows, dg::kMaxHomeRows)) !=
                           cudaSuccess))
    return fail(DG_ERR_CUDA);

  if (cudaMalloc(&g->ctl, sizeof(dg::DevCtl)) != cudaSuccess) return fail(DG_ERR_CUDA);
  if (cudaMemsetAsync(g->ctl, 0, sizeof(dg::DevCtl), s) != cudaSuccess) return fail(DG_ERR_CUDA);
  if (cudaMallocHost(&g->hctl, sizeof(dg::DevCtl)) != cudaSuccess) return fail(DG_ERR_CUDA);
  std::memset(g->hctl, 0, sizeof(dg::DevCtl));
  if (cudaEventCreateWithFlags(&g->snap_event, cudaEventDisableTiming) != cudaSuccess)
    return fail(DG_ERR_CUDA);
  if (ensure_ret(g, 0) != DG_OK) return fail(DG_ERR_CUDA);
  if (cudaMalloc(&g->small_dev, 64) != cudaSuccess) return fail(DG_ERR_CUDA);
  if (const char* hs = std::getenv("DG_HOT_STEPS")) g->hot_steps = (u32)std::atoi(hs);
  if (cudaMalloc(&g->hot_list, (size_t)g->hot_cap * 4) != cudaSuccess) return fail(DG_ERR_CUDA);
  if (cudaHostAlloc(reinterpret_cast<void**>(&g->h_hot), 64, cudaHostAllocMapped) != cudaSuccess ||
      cudaHostGetDevicePointer(reinterpret_cast<void**>(&g->d_hot), g->h_hot, 0) != cudaSuccess)
    return fail(DG_ERR_CUDA);
  g->h_hot[0] = g->h_hot[1] = 0;
  if (cudaMalloc(&g->stats_dev, sizeof(dg::StatsOut)) != cudaSuccess) return fail(DG_ERR_CUDA);

  if (g->nranks > 1 || (cfg->group && (cfg->flags & DG_FLAG_FORCE_ROUTER))) {
    dg_status st = dg::router_create(g, cfg->nccl_unique_id, &g->router);
    if (st != DG_OK) return fail(st);
  } else if (cfg->flags & DG_FLAG_FORCE_ROUTER) {
    // diagnostic: route a single-GPU graph through the router (1-rank NCCL communicator)
    char id[128];
    dg_status st = dg::router_unique_id(id);
    if (st == DG_OK) st = dg::router_create(g, id, &g->router);
    if (st != DG_OK) return fail(st);
  }
  if (g->router) {  // peer receive windows for the fused exchange (collective)
    dg_status st = dg::router_setup_fused(g, s);
    if (st != DG_OK) return fail(st);
  }

  // hints: indexed by global vertex id
  const void* hints = nullptr;
  bool host = false;
  dg_status st = stage_in(g, 0, degree_hints, degree_hints ? num_vertices * 4 : 0, s, &hints, &host);
  if (st != DG_OK) return fail(st);
  const u64 rows = dg::rows_for(num_vertices, g->nranks, g->rank);
  // overflow slack beyond the base buckets
  u64 slack = cfg->pool_bytes ? cfg->pool_bytes / g->bucket_bytes : 0;
  if (!cfg->pool_bytes) slack = std::max<u64>(rows / 4, 1u << 16);
  if (rows) {
    st = add_rows(g, 0, rows, reinterpret_cast<const u32*>(hints), nullptr, slack, s);
  } else {
    for (int c = 0; c < g->ncls && st == DG_OK; ++c) st = dg::grow_pool(g, c, slack, s);
  }
  if (st != DG_OK) return fail(st);
  if (cudaStreamSynchronize(s) != cudaSuccess) return fail(DG_ERR_CUDA);
  *out = g;
  return DG_OK;
}

dg_status dg_destroy(dg_graph g) {
  if (!g) return DG_ERR_INVALID_ARGUMENT;
  destroy_graph(g);
  return DG_OK;
}

dg_status dg_num_vertices(dg_graph g, uint64_t* num_vertices, uint64_t* local_rows) {
  if (!g) return DG_ERR_INVALID_ARGUMENT;
  if (num_vertices) *num_vertices = g->nv;
  if (local_rows) *local_rows = g->rows;
  return DG_OK;
}

static dg_status check_handle(dg_graph g) {
  if (!g) return DG_ERR_INVALID_ARGUMENT;
  if (g->bad) return DG_ERR_BAD_STATE;
  int cur = -1;
  if (cudaGetDevice(&cur) == cudaSuccess && cur == g->device) return DG_OK;
  if (cudaSetDevice(g->device) != cudaSuccess) {
    g->bad = true;
    return DG_ERR_CUDA;
  }
  return DG_OK;
}

dg_status dg_insert_edges(dg_graph g, const uint32_t* src, const uint32_t* dst,
                          const uint32_t* weight, uint64_t n, uint64_t* n_added, void* stream) {
  DG_TRY(check_handle(g));
  if (n > kMaxBatch) return DG_ERR_INVALID_ARGUMENT;
  if (n && (!src || !dst)) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  if (n_added) *n_added = 0;
  // re-size tables whose chains grew too long in earlier batches
  if (g->hot_steps) {
    // worth a re-sizing pass (it synchronises): flagged pairs reach 1/1024 of the
    // table slots (at least 2,048), or the flag list is filling up.  The counters are
    // the ones the last finished insert published (mapped memory, no copy, no event).
    const u32 hot_rows = reinterpret_cast<volatile u32*>(g->h_hot)[0];
    const u32 hot_pairs = reinterpret_cast<volatile u32*>(g->h_hot)[1];
    if (hot_rows) {
      u64 slots = 0;
      for (int c = 0; c < g->ncls; ++c) slots += g->bump_ub[c] * (g->adaptive ? (4u << c) - 1 : g->BC);
      const u64 thr = std::max<u64>(2048, slots / 1024);
      if (hot_pairs >= thr || hot_rows >= g->hot_cap / 2) DG_TRY(dg::rehash_hot(g, s));
    }
  }
  const u32 epoch = ++g->epoch;
  bool host = false;
  const void *ds = nullptr, *dd = nullptr, *dw = nullptr;
  const bool dev_src = is_device_ptr(src), dev_dst = is_device_ptr(dst);
  const bool dev_w = weight && is_device_ptr(weight);
  if (!g->router && !n_added && n && !dev_src && !dev_dst && (!weight || !dev_w)) {
    // host inputs, no count requested: return once the batch is uploaded and
    // validated; the insert kernel runs behind the caller's next upload
    DG_TRY(upload_async(g, 8, src, n * 4, s, &ds));
    DG_TRY(upload_async(g, 9, dst, n * 4, s, &dd));
    DG_TRY(upload_async(g, 10, weight, weight ? n * 4 : 0, s, &dw));
    DG_TRY(dg::validated_insert(g, (const u32*)ds, (const u32*)dd, (const u32*)dw, n, epoch, true,
                                s));
    DG_TRY(release_slots(g, 8, 11, s));
    return validation_status(g, epoch);
  }
  DG_TRY(stage_in(g, 0, src, n * 4, s, &ds, &host, dev_src));
  DG_TRY(stage_in(g, 1, dst, n * 4, s, &dd, &host, dev_dst));
  DG_TRY(stage_in(g, 2, weight, weight ? n * 4 : 0, s, &dw, &host, dev_w));
  if (g->router) {
    DG_TRY(dg::router_insert(g, (const u32*)ds, (const u32*)dd, (const u32*)dw, n, epoch, s));
  } else {
    DG_TRY(dg::validated_insert(g, (const u32*)ds, (const u32*)dd, (const u32*)dw, n, epoch, false,
                                s));
  }
  if (n_added || host) {
    DG_TRY(read_ctl(g, s));
    u64 cnt = g->hctl->count;
    if (g->router) DG_TRY(dg::router_sum_u64(g, &cnt, s));
    if (n_added) *n_added = cnt;
    g->snap_pending = false;
    dg::bound_exact(g);
    return status_of(g, epoch);
  }
  return DG_OK;
}

dg_status dg_delete_edges(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                          uint64_t* n_removed, void* stream) {
  DG_TRY(check_handle(g));
  if (n > kMaxBatch) return DG_ERR_INVALID_ARGUMENT;
  if (n && (!src || !dst)) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  if (n_removed) *n_removed = 0;
  const u32 epoch = ++g->epoch;
  bool host = false;
  const void *ds = nullptr, *dd = nullptr;
  const bool dev_src = is_device_ptr(src), dev_dst = is_device_ptr(dst);
  if (!g->router && !n_removed && n && !dev_src && !dev_dst) {
    // host inputs, no count requested: as in dg_insert_edges
    DG_TRY(upload_async(g, 11, src, n * 4, s, &ds));
    DG_TRY(upload_async(g, 12, dst, n * 4, s, &dd));
    DG_TRY(dg::local_delete(g, (const u32*)ds, (const u32*)dd, n, !g->directed, epoch, s, true, true));
    DG_TRY(release_slots(g, 11, 13, s));
    return validation_status(g, epoch);
  }
  DG_TRY(stage_in(g, 0, src, n * 4, s, &ds, &host, dev_src));
  DG_TRY(stage_in(g, 1, dst, n * 4, s, &dd, &host, dev_dst));
  if (g->router) {
    DG_TRY(dg::router_delete(g, (const u32*)ds, (const u32*)dd, n, epoch, s));
  } else {
    DG_TRY(dg::local_delete(g, (const u32*)ds, (const u32*)dd, n, !g->directed, epoch, s, true, false));
  }
  if (n_removed || host) {
    if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
    g->snap_pending = false;
    DG_TRY(read_ctl(g, s));
    u64 cnt = g->hctl->count;
    if (g->router) DG_TRY(dg::router_sum_u64(g, &cnt, s));
    if (n_removed) *n_removed = cnt;
    return status_of(g, epoch);
  }
  return DG_OK;
}

// Host-buffer queries are pipelined in chunks over two internal copy streams: the
// upload of chunk k+1 and the download of the answers of chunk k-1 overlap the probe
// kernel of chunk k (PCIe is full duplex).  Queries never mutate, so unlike
// inserts/deletes they need no batch-wide validation before the first kernel.
static dg_status query_host_pipelined(dg_graph g, const u32* src, const u32* dst, u64 n,
                                      uint8_t* found, u32* wout, u32 epoch, cudaStream_t s) {
  constexpr u64 kChunk = 1ull << 22;
  const u64 nch = (n + kChunk - 1) / kChunk;
  DG_CK(ensure_buf(g->stage[13], n * 4));
  DG_CK(ensure_buf(g->stage[14], n * 4));
  DG_CK(ensure_buf(g->stage[3], n));
  if (wout) DG_CK(ensure_buf(g->stage[4], n * 4));
  DG_TRY(ensure_copy_streams(g));
  while (g->pipe_ev.size() < 2 * nch + 1) {
    cudaEvent_t e;
    DG_CK(cudaEventCreateWithFlags(&e, cudaEventDisableTiming));
    g->pipe_ev.push_back(e);
  }
  u32* ds = reinterpret_cast<u32*>(g->stage[13].p);
  u32* dd = reinterpret_cast<u32*>(g->stage[14].p);
  uint8_t* df = reinterpret_cast<uint8_t*>(g->stage[3].p);
  u32* dw = wout ? reinterpret_cast<u32*>(g->stage[4].p) : nullptr;
  cudaStream_t up = g->cstream[0], down = g->cstream[1];
  // slots 13/14 belong to this pipeline alone (it completes before returning), so the
  // uploads need not wait for earlier kernels on s: they overlap them
  for (u64 k = 0; k < nch; ++k) {
    const u64 off = k * kChunk, cnt = std::min(kChunk, n - off);
    DG_CK(cudaMemcpyAsync(ds + off, src + off, cnt * 4, cudaMemcpyHostToDevice, up));
    DG_CK(cudaMemcpyAsync(dd + off, dst + off, cnt * 4, cudaMemcpyHostToDevice, up));
    DG_CK(cudaEventRecord(g->pipe_ev[1 + 2 * k], up));
    DG_CK(cudaStreamWaitEvent(s, g->pipe_ev[1 + 2 * k], 0));
    DG_TRY(dg::local_query(g, ds + off, dd + off, cnt, df + off, dw ? dw + off : nullptr, epoch, s));
    DG_CK(cudaEventRecord(g->pipe_ev[2 + 2 * k], s));
    DG_CK(cudaStreamWaitEvent(down, g->pipe_ev[2 + 2 * k], 0));
    DG_CK(cudaMemcpyAsync(found + off, df + off, cnt, cudaMemcpyDeviceToHost, down));
    if (wout)
      DG_CK(cudaMemcpyAsync(wout + off, dw + off, cnt * 4, cudaMemcpyDeviceToHost, down));
  }
  DG_CK(cudaStreamSynchronize(down));
  DG_CK(cudaStreamSynchronize(s));
  return DG_OK;
}

dg_status dg_query_edges(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                         uint8_t* found, uint32_t* weight_out, void* stream) {
  DG_TRY(check_handle(g));
  if (n > kMaxBatch) return DG_ERR_INVALID_ARGUMENT;
  if (n && (!src || !dst || !found)) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  const u32 epoch = ++g->epoch;
  if (!g->router && n >= (1ull << 23) && !is_device_ptr(src) && !is_device_ptr(dst) &&
      !is_device_ptr(found) && (!weight_out || !is_device_ptr(weight_out))) {
    DG_TRY(query_host_pipelined(g, src, dst, n, found, weight_out, epoch, s));
    if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
    g->snap_pending = false;
    DG_TRY(read_ctl(g, s));
    return status_of(g, epoch);
  }
  bool host = false;
  const void *ds = nullptr, *dd = nullptr;
  void *df = nullptr, *dw = nullptr;
  DG_TRY(stage_in(g, 0, src, n * 4, s, &ds, &host));
  DG_TRY(stage_in(g, 1, dst, n * 4, s, &dd, &host));
  DG_TRY(stage_out(g, 3, found, n, &df, &host));
  DG_TRY(stage_out(g, 4, weight_out, weight_out ? n * 4 : 0, &dw, &host));
  if (g->router) {
    DG_TRY(dg::router_query(g, (const u32*)ds, (const u32*)dd, n, (uint8_t*)df, (u32*)dw, epoch, s));
  } else {
    DG_TRY(dg::local_query(g, (const u32*)ds, (const u32*)dd, n, (uint8_t*)df, (u32*)dw, epoch, s));
  }
  if (host) {
    DG_TRY(finish_out(g, found, df, n, s));
    DG_TRY(finish_out(g, weight_out, dw, weight_out ? n * 4 : 0, s));
    if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
    g->snap_pending = false;
    DG_TRY(read_ctl(g, s));
    return status_of(g, epoch);
  }
  return DG_OK;
}

dg_status dg_insert_vertices(dg_graph g, const uint32_t* ids, uint64_t n,
                             const uint32_t* degree_hints, void* stream) {
  DG_TRY(check_handle(g));
  if (n > kMaxBatch) return DG_ERR_INVALID_ARGUMENT;
  if (n && !ids) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  bool host = false;
  const void *di = nullptr, *dh = nullptr;
  DG_TRY(stage_in(g, 5, ids, n * 4, s, &di, &host));
  DG_TRY(stage_in(g, 6, degree_hints, degree_hints ? n * 4 : 0, s, &dh, &host));
  if (g->router) {
    // every rank needs every (id, hint): the rows of an ID live on its owner
    const u32* all_ids = nullptr;
    const u32* all_h = nullptr;
    u64 all_n = 0, hn = 0;
    DG_TRY(dg::router_allgather_u32(g, (const u32*)di, n, 0, &all_ids, &all_n, s));
    if (!dh && n) {  // a rank without hints contributes zeros (= unknown degree)
      DG_CK(ensure_buf(g->stage[6], n * 4));
      DG_CK(cudaMemsetAsync(g->stage[6].p, 0, n * 4, s));
      dh = g->stage[6].p;
    }
    DG_TRY(dg::router_allgather_u32(g, (const u32*)dh, n, 1, &all_h, &hn, s));
    di = all_ids;
    dh = all_h;
    n = all_n;
  }
  u64 maxid = 0;
  bool any = n > 0;
  if (any) {
    DG_CK(dg::launch_max_id((const u32*)di, n, g->small_dev, s));
    u32 m = 0;
    DG_CK(cudaMemcpyAsync(&m, g->small_dev, 4, cudaMemcpyDeviceToHost, s));
    DG_CK(cudaStreamSynchronize(s));
    maxid = m;
    if (maxid >= kMaxVertices) return DG_ERR_VERTEX_OUT_OF_RANGE;
  }
  u64 new_nv = g->nv;
  if (any) new_nv = std::max<u64>(new_nv, maxid + 1);
  if (g->router) DG_TRY(dg::router_max_u64(g, &new_nv, s));
  if (new_nv <= g->nv) return DG_OK;  // Q12: existing IDs are a no-op
  if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
  g->snap_pending = false;
  const u64 new_rows = dg::rows_for(new_nv, g->nranks, g->rank);
  const u64 row0 = g->rows;
  const u64 count = new_rows - row0;
  if (count) {
    u32* hint_new = nullptr;
    DG_CK(cudaMallocAsync(&hint_new, count * 4, s));
    DG_CK(cudaMemsetAsync(hint_new, 0, count * 4, s));
    DG_CK(dg::launch_scatter_hints(hint_new, row0, count, (const u32*)di, (const u32*)dh, n,
                                   g->nranks, g->rank, s));
    dg_status st = add_rows(g, row0, count, nullptr, hint_new, std::max<u64>(count / 4, 4096), s);
    cudaFreeAsync(hint_new, s);
    if (st != DG_OK) return st;
  }
  g->nv = new_nv;
  DG_CK(cudaStreamSynchronize(s));
  return DG_OK;
}

dg_status dg_delete_vertices(dg_graph g, const uint32_t* ids, uint64_t n, void* stream) {
  DG_TRY(check_handle(g));
  if (n > kMaxBatch) return DG_ERR_INVALID_ARGUMENT;
  if (n && !ids) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  const u32 epoch = ++g->epoch;
  bool host = false;
  const void* di = nullptr;
  DG_TRY(stage_in(g, 5, ids, n * 4, s, &di, &host));
  const u32* all_ids = (const u32*)di;
  u64 all_n = n;
  if (g->router) DG_TRY(dg::router_allgather_u32(g, all_ids, n, 0, &all_ids, &all_n, s));
  if (all_n == 0) return DG_OK;
  DG_TRY(ensure_bitmap(g, g->nv));
  DG_TRY(ensure_dedup(g, all_n));
  const u64 bwords = (g->nv + 31) / 32 + 1;
  u32* filter = g->bitmap + bwords;
  u32 fshift = 0;
  while (((g->nv - 1) >> fshift) >= dg::kVdelFilterBits) ++fshift;
  DG_CK(cudaMemsetAsync(g->bitmap, 0, (bwords + dg::kVdelFilterBits / 32) * 4, s));
  DG_CK(cudaMemsetAsync(&g->ctl->queue, 0, 2 * sizeof(u32), s));  // queue, dedup_count
  const dg::Tables t = g->tables();
  DG_CK(dg::launch_vdel_mark(all_ids, all_n, g->nv, epoch, g->bitmap, filter, fshift, g->dedup,
                             g->ctl, g->nranks, g->rank, g->sms, s));
  static const bool force_sweep = std::getenv("DG_FORCE_SWEEP") != nullptr;
  // base-bucket offsets of the distinct deleted vertices (flattened purge work)
  DG_CK(ensure_buf(g->stage[7], (all_n + 1) * 8 * 2));
  u64* nbarr = reinterpret_cast<u64*>(g->stage[7].p);
  u64* boff = nbarr + (all_n + 1);
  DG_CK(dg::launch_vdel_nb(t, g->dedup, all_n, nbarr, g->sms, s));
  DG_CK(dg::scan_exclusive_u64(nbarr, boff, all_n + 1, &g->scan_temp, &g->scan_bytes, s));
  dg::prof_mark(g, dg::PROF_VDEL, s);
  if (!g->directed && g->nranks == 1 && !force_sweep) {
    // undirected: Alg. 2 — delete u from the tables of its neighbours
    DG_CK(dg::launch_vdel_neighbors(g->lay, t, g->dedup, boff, epoch, g->sms, s));
  } else {
    // directed: follow-up sweep over all tables
    DG_CK(dg::launch_vdel_sweep(g->lay, t, g->bitmap, filter, fshift, epoch, g->sms, s));
  }
  DG_CK(dg::launch_vdel_clear(g->lay, t, g->dedup, boff, epoch, g->sms, s));
  dg::prof_mark(g, dg::PROF_VDEL, s);
  if (host) {
    if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
    g->snap_pending = false;
    DG_TRY(read_ctl(g, s));
    return status_of(g, epoch);
  }
  return DG_OK;
}

dg_status dg_export_adjacency(dg_graph g, uint64_t* row_offsets, uint32_t* dst, uint32_t* weight,
                              uint64_t capacity, uint64_t* n_edges, void* stream) {
  DG_TRY(check_handle(g));
  if (!row_offsets || !n_edges) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  bool host = false;
  void* dro = nullptr;
  DG_TRY(stage_out(g, 3, row_offsets, (g->rows + 1) * 8, &dro, &host));
  const dg::Tables t = g->tables();
  DG_CK(dg::launch_export_offsets(t, (u64*)dro, &g->scan_temp, &g->scan_bytes, s));
  u64 m = 0;
  DG_CK(cudaMemcpyAsync(&m, (u64*)dro + g->rows, 8, cudaMemcpyDeviceToHost, s));
  DG_CK(cudaStreamSynchronize(s));
  *n_edges = m;
  if (dst) {
    if (capacity < m) {
      DG_TRY(finish_out(g, row_offsets, dro, (g->rows + 1) * 8, s));
      DG_CK(cudaStreamSynchronize(s));
      return DG_ERR_INVALID_ARGUMENT;
    }
    void *dd = nullptr, *dw = nullptr;
    DG_TRY(stage_out(g, 4, dst, m * 4, &dd, &host));
    DG_TRY(stage_out(g, 7, weight, weight ? m * 4 : 0, &dw, &host));
    DG_CK(ensure_buf(g->big, (g->rows + 2) * 4));
    DG_CK(dg::launch_export_fill(g->lay, t, (const u64*)dro, (u32*)dd, (u32*)dw, (u32*)g->big.p,
                                 g->sms, s));
    DG_TRY(finish_out(g, dst, dd, m * 4, s));
    DG_TRY(finish_out(g, weight, dw, weight ? m * 4 : 0, s));
  }
  DG_TRY(finish_out(g, row_offsets, dro, (g->rows + 1) * 8, s));
  DG_CK(cudaStreamSynchronize(s));
  return DG_OK;
}

dg_status dg_degrees(dg_graph g, uint32_t* out, void* stream) {
  DG_TRY(check_handle(g));
  if (!out) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  bool host = false;
  void* d = nullptr;
  DG_TRY(stage_out(g, 3, out, g->rows * 4, &d, &host));
  DG_CK(dg::launch_degrees(g->tables(), (u32*)d, s));
  if (host) {
    DG_TRY(finish_out(g, out, d, g->rows * 4, s));
    DG_CK(cudaStreamSynchronize(s));
  }
  return DG_OK;
}

dg_status dg_get_stats(dg_graph g, dg_stats* out, void* stream) {
  DG_TRY(check_handle(g));
  if (!out) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  dg::StatsOut h{};
  auto* d = reinterpret_cast<dg::StatsOut*>(g->stats_dev);
  DG_CK(ensure_buf(g->big, (g->rows + 2) * 4));
  DG_CK(dg::launch_stats(g->lay, g->tables(), d, (u32*)g->big.p, g->sms, s));
  DG_CK(cudaMemcpyAsync(&h, d, sizeof(h), cudaMemcpyDeviceToHost, s));
  if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
  g->snap_pending = false;
  DG_TRY(read_ctl(g, s));
  std::memset(out, 0, sizeof(*out));
  out->local_rows = g->rows;
  out->exchange = !g->router ? 0 : dg::router_fused(g->router) ? 2 : 1;
  out->base_buckets = h.base_buckets;
  out->overflow_buckets = h.linked_buckets - h.base_buckets;
  out->pool_bytes = g->dir.mapped() + g->degv.mapped() + g->home.mapped() + g->nbsv.mapped();
  for (int c = 0; c < g->ncls; ++c) {
    out->free_buckets += g->hctl->stack_size[c];
    out->pool_buckets += g->cap[c];
    out->bump_buckets += g->hctl->bump[c];
    out->bump_bytes += (u64)g->hctl->bump[c] * g->cbytes(c);
    out->pool_bytes += g->pool[c].mapped() + g->stack[c].mapped();
  }
  if (!g->adaptive) {  // the home buckets (one per row) are handed out and swept too
    out->bump_buckets += g->rows;
    out->bump_bytes += g->rows * g->bucket_bytes;
  }
  out->live_pairs = h.live;
  out->tombstones = h.tombs;
  out->max_chain = h.max_chain;
  // realised load factor = keys / key slots of the linked buckets (Q14)
  out->load_factor = h.slots ? (double)h.live / (double)h.slots : 0.0;
  out->utilization = h.bytes ? (double)h.live * 8.0 / (double)h.bytes : 0.0;
  out->table_bytes = h.bytes;
  return DG_OK;
}

dg_status dg_batch_status(dg_graph g, void* stream) {
  DG_TRY(check_handle(g));
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
  g->snap_pending = false;
  DG_TRY(read_ctl(g, s));
  dg_status st = DG_OK;
  if (g->hctl->fail_epoch > g->checked_epoch) st = DG_ERR_VERTEX_OUT_OF_RANGE;
  g->checked_epoch = g->epoch;
  return st;
}

dg_status dg_flush_tombstones(dg_graph g, uint64_t* rows_rebuilt, void* stream) {
  DG_TRY(check_handle(g));
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  if (rows_rebuilt) *rows_rebuilt = 0;
  // (rows flagged by earlier inserts are rebuilt below too)
  u64 total = 0;
  for (int pass = 0; pass < 100000; ++pass) {
    dg::Tables t = g->tables();
    t.hot_flags = g->hot_flags;
    DG_CK(dg::launch_tomb_sweep(g->lay, t, g->sms, s));
    if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
    g->snap_pending = false;
    DG_TRY(read_ctl(g, s));
    const u32 found = g->hctl->hot_count;
    if (found == 0) break;
    const u32 n = std::min<u32>(found, g->hot_cap);
    DG_TRY(dg::rehash_rows(g, n, true, s));
    total += n;
  }
  if (rows_rebuilt) *rows_rebuilt = total;
  return DG_OK;
}

// Triangle-count scratch k: a growable VMM array (a large virtual range reserved once,
// physical memory mapped at its end as the graph grows: no free, no copy, no
// re-allocation of the whole buffer — cudaFree + cudaMalloc of multi-GB scratch cost
// 40-600 ms on single cfg5 steps).  The contents need not survive growth.
static dg_status tc_buf(dg_graph g, int k, size_t bytes, cudaStream_t s) {
  dg::VmmArray& a = g->tcv[k];
  if (!a.ptr()) {
    // first use: map twice the need, so a graph that keeps growing between triangle
    // counts (cfg5 more than doubles over its 10 steps) maps new memory rarely
    DG_CK(a.reserve(g->device, 64ull << 30));
    DG_CK(a.ensure(std::min<size_t>(2 * bytes, a.reserved()), -1, s));
  }
  DG_CK(a.ensure(bytes, -1, s));
  return DG_OK;
}

dg_status dg_triangle_count(dg_graph g, uint32_t part, uint32_t nparts, uint64_t* count,
                            void* stream) {
  DG_TRY(check_handle(g));
  if (!count || nparts == 0 || part >= nparts) return DG_ERR_INVALID_ARGUMENT;
  if (g->nranks != 1) return DG_ERR_UNSUPPORTED;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  *count = 0;
  // DG_TRACE_TC=1: wall time of each phase (synchronising after each) on stderr
  static const bool trace = std::getenv("DG_TRACE_TC") != nullptr;
  auto tprev = std::chrono::steady_clock::now();
  auto tmark = [&](const char* what) {
    if (!trace) return;
    cudaStreamSynchronize(s);
    const auto now = std::chrono::steady_clock::now();
    std::fprintf(stderr, "dg tc: %-12s %8.3f ms\n", what,
                 std::chrono::duration<double, std::milli>(now - tprev).count());
    tprev = now;
  };
  const dg::Tables t = g->tables();
  const u64 rows = g->rows;
  // (1) adjacency export (a12): CSR of every A_u
  DG_TRY(tc_buf(g, 0, (rows + 1) * 8, s));
  u64* ro = reinterpret_cast<u64*>(g->tcv[0].ptr());
  DG_CK(dg::launch_export_offsets(t, ro, &g->scan_temp, &g->scan_bytes, s));
  u64 m = 0;
  DG_CK(cudaMemcpyAsync(&m, ro + rows, 8, cudaMemcpyDeviceToHost, s));
  DG_CK(cudaStreamSynchronize(s));
  if (m >= 0xFFFFFFFFull) return DG_ERR_UNSUPPORTED;
  DG_TRY(tc_buf(g, 1, m * 4 + 4, s));
  u32* dst = reinterpret_cast<u32*>(g->tcv[1].ptr());
  DG_CK(ensure_buf(g->big, (rows + 2) * 4, true));
  u32* big = reinterpret_cast<u32*>(g->big.p);
  DG_CK(dg::launch_export_fill(g->lay, t, ro, dst, nullptr, big, g->sms, s));
  tmark("export");
  // (2) orientation by rank = (degree, id)
  DG_TRY(tc_buf(g, 2, (rows + 1) * 8, s));
  DG_TRY(tc_buf(g, 3, (rows + 1) * 8, s));
  u64* ocnt = reinterpret_cast<u64*>(g->tcv[2].ptr());
  u64* oro = reinterpret_cast<u64*>(g->tcv[3].ptr());
  DG_CK(dg::launch_tc_orient_count(t, ro, dst, part, nparts, ocnt, big, g->sms, s));
  DG_CK(dg::scan_exclusive_u64(ocnt, oro, rows + 1, &g->scan_temp, &g->scan_bytes, s));
  u64 mo = 0;
  DG_CK(cudaMemcpyAsync(&mo, oro + rows, 8, cudaMemcpyDeviceToHost, s));
  DG_CK(cudaStreamSynchronize(s));
  DG_TRY(tc_buf(g, 4, mo * 4 + 4, s));
  DG_TRY(tc_buf(g, 5, mo * 4 + 4, s));
  u32* oadj = reinterpret_cast<u32*>(g->tcv[4].ptr());
  u32* oend = reinterpret_cast<u32*>(g->tcv[5].ptr());
  DG_CK(dg::launch_tc_orient_fill(t, ro, dst, part, nparts, oro, oadj, oend, big, g->sms, s));
  tmark("orient");
  // (3) probe order: entries sorted by the probed vertex (kernels_tc.cu; off unless
  // DG_TC_ORDER=1: measured on cfg5 it cuts the wedge kernel's DRAM reads 380 -> 52 GB
  // but mixes entries of very different candidate counts in a warp, 64 -> 150 G
  // instructions, 111 -> 237 ms)
  const u32* perm = nullptr;
  static const bool tc_order = std::getenv("DG_TC_ORDER") != nullptr &&
                               std::atoi(std::getenv("DG_TC_ORDER")) != 0;
  if (tc_order) {
    DG_TRY(tc_buf(g, 6, mo * 8 + 8, s));
    DG_TRY(tc_buf(g, 7, mo * 8 + 8, s));
    DG_CK(dg::launch_tc_probe_order(oadj, mo, rows, (u32*)g->tcv[6].ptr(), (u32*)g->tcv[7].ptr(), &perm,
                                    &g->scan_temp, &g->scan_bytes, s));
  }
  // (4) one edgeExist per wedge: uniform layouts number the wedges and give every lane
  // one (k_tc_wedges_flat, DG_TC_FLAT=0: the per-entry kernel); the adaptive layout
  // keeps the per-entry kernel
  static const bool tc_flat = std::getenv("DG_TC_FLAT") == nullptr ||
                              std::atoi(std::getenv("DG_TC_FLAT")) != 0;
  const bool flat = tc_flat && !g->adaptive && mo < (1ull << 31);
  uint2* list = nullptr;
  u64* woff = nullptr;
  u32* chunk_k = nullptr;
  unsigned long long* nlist_dev = nullptr;
  if (flat) {
    DG_TRY(tc_buf(g, 8, mo * 8 + 8, s));
    DG_TRY(tc_buf(g, 9, mo * 8 + 24, s));
    list = (uint2*)g->tcv[8].ptr();
    woff = (u64*)g->tcv[9].ptr();
    nlist_dev = (unsigned long long*)((char*)g->tcv[9].ptr() + mo * 8 + 8);  // (after woff[mo])
    u64 nl = 0;
    DG_CK(dg::launch_tc_flat_prepare(oadj, oend, perm, mo, list, woff, nlist_dev, &nl, &g->scan_temp,
                                     &g->scan_bytes, s));
    u64 wedges = 0;  // (sizes the chunk table)
    DG_CK(cudaMemcpyAsync(&wedges, woff + nl, 8, cudaMemcpyDeviceToHost, s));
    DG_CK(cudaStreamSynchronize(s));
    DG_TRY(tc_buf(g, 10, dg::tc_chunk_count(wedges) * 4 + 4, s));
    chunk_k = (u32*)g->tcv[10].ptr();
  tmark("flat_prep");
  }
  DG_CK(cudaMemsetAsync(&g->ctl->count, 0, 8, s));
  dg::prof_mark(g, dg::PROF_TC, s);
  if (flat)
    DG_CK(dg::launch_tc_wedges_flat(g->lay, t, oadj, list, woff, chunk_k, nlist_dev,
                                    reinterpret_cast<unsigned long long*>(&g->ctl->count), g->sms, s));
  else
    DG_CK(dg::launch_tc_wedges(g->lay, t, oadj, oend, perm, mo,
                               reinterpret_cast<unsigned long long*>(&g->ctl->count), g->sms, s));
  dg::prof_mark(g, dg::PROF_TC, s);
  tmark("wedges");
  DG_TRY(read_ctl(g, s));
  *count = g->hctl->count;
  return DG_OK;
}

dg_status dg_check_invariants(dg_graph g, dg_invariants* out, void* stream) {
  DG_TRY(check_handle(g));
  if (!out) return DG_ERR_INVALID_ARGUMENT;
  static_assert(sizeof(dg_invariants) == sizeof(dg::InvariantsOut), "dg_invariants layout");
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  dg::InvariantsOut* d = nullptr;
  DG_CK(cudaMallocAsync(&d, sizeof(*d), s));
  DG_CK(dg::launch_check(g->lay, g->tables(), g->nv, g->rank, d, g->sms, s));
  DG_CK(cudaMemcpyAsync(out, d, sizeof(*d), cudaMemcpyDeviceToHost, s));
  DG_CK(cudaFreeAsync(d, s));
  DG_CK(cudaStreamSynchronize(s));
  return DG_OK;
}

dg_status dg_profile_enable(dg_graph g, int enable) {
  DG_TRY(check_handle(g));
  cudaDeviceSynchronize();
  prof_clear(g);
  g->prof = enable != 0;
  g->prof_launch0 = dg::kernel_launches();
  return DG_OK;
}

dg_status dg_profile_read(dg_graph g, dg_profile* out, void* stream) {
  DG_TRY(check_handle(g));
  if (!out) return DG_ERR_INVALID_ARGUMENT;
  cudaStream_t s = reinterpret_cast<cudaStream_t>(stream);
  std::memset(out, 0, sizeof(*out));
  if (g->snap_pending) DG_CK(cudaEventSynchronize(g->snap_event));
  g->snap_pending = false;
  DG_TRY(read_ctl(g, s));
  for (int k = 0; k < 5; ++k) {
    auto& v = g->prof_ev[k];
    for (size_t i = 0; i + 1 < v.size(); i += 2) {
      float ms = 0.f;
      DG_CK(cudaEventSynchronize(v[i + 1]));
      DG_CK(cudaEventElapsedTime(&ms, v[i], v[i + 1]));
      out->kernel_ms[k] += ms;
      out->kernel_launches[k] += 1;
    }
  }
  out->launches = dg::kernel_launches() - g->prof_launch0;
  out->last_count = g->hctl->count;
  return DG_OK;
}

}  // extern "C"
