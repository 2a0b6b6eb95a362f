// graph.h — host-side state behind a dg_graph handle.
#pragma once
#include <cstddef>
#include <cstdint>
#include <deque>
#include <utility>
#include <vector>

#include <cuda_runtime.h>

#include "../../include/dg.h"
#include "dg_common.cuh"
#include "vmm.h"

namespace dg {
struct Router;  // multi-GPU batch router (router.cu)
}

struct dg_graph_s {
  dg_config cfg{};
  int device = 0;
  int sms = 148;
  int G = 8;              // lanes per bucket (bucket_bytes / 16; adaptive: 8)
  bool set = false;       // set variant: keys only (DG_FLAG_SET)
  bool adaptive = false;  // degree-adaptive bucket sizes (DG_FLAG_ADAPTIVE)
  int ncls = 1;           // size classes in use (uniform 1, adaptive 3)
  int lay = DG_LAY(8, 0); // layout code for the launchers
  uint32_t W = 32;        // words per bucket (uniform layouts)
  uint32_t BC = 15;       // pairs (keys, set variant) per bucket (uniform layouts)
  uint32_t bucket_bytes = 128;  // uniform layouts; adaptive: the largest class
  uint32_t lf_milli = 700;
  uint32_t nranks = 1, rank = 0;
  bool directed = true;
  bool reuse_tombstones = true;

  uint64_t nv = 0;        // global vertex capacity
  uint64_t rows = 0;      // local rows

  dg::VmmArray dir, degv;
  dg::VmmArray home;  // uniform layouts: one home bucket per row (chain 0)
  dg::VmmArray nbsv;  // uniform layouts: min(nb, 255) per row (the probe's chain count)
  dg::VmmArray pool[dg::kClasses], stack[dg::kClasses];  // per size class
  uint32_t cap[dg::kClasses] = {0, 0, 0};      // buckets mapped in each pool
  uint64_t bump_ub[dg::kClasses] = {0, 0, 0};  // host upper bounds of the device bump cursors
  // insert launches whose cursors the fixup kernel has not published yet: (epoch,
  // worst-case buckets); the bound is published bump + their sum (api.cu refresh_bound)
  std::deque<std::pair<uint32_t, uint64_t>> pending_need;
  uint32_t pub_floor = 0;  // publications older than this epoch predate an exact read
  // bytes of one bucket of class c
  uint32_t cbytes(int c) const { return adaptive ? (32u << c) : bucket_bytes; }

  dg::DevCtl* ctl = nullptr;       // device
  dg::DevCtl* hctl = nullptr;      // pinned host mirror (snapshots)
  cudaEvent_t snap_event = nullptr;
  bool snap_pending = false;
  uint32_t* ret_list = nullptr;
  uint64_t ret_cap = 0;
  uint64_t* retry[2] = {nullptr, nullptr};
  uint64_t retry_cap[2] = {0, 0};
  uint32_t* bitmap = nullptr;
  uint64_t bitmap_words = 0;
  uint32_t* dedup = nullptr;
  uint64_t dedup_cap = 0;
  void* scan_temp = nullptr;
  size_t scan_bytes = 0;
  void* stats_dev = nullptr;
  uint32_t* small_dev = nullptr;   // scratch words

  uint32_t epoch = 0;
  uint32_t checked_epoch = 0;
  uint32_t validated_epoch = 0;  // batch whose sources k_validate checked (sortedness, a3)
  bool bad = false;

  struct Buf {
    void* p = nullptr;
    size_t bytes = 0;
  } stage[16];
  // asynchronous host inputs (slots 8..15): event recorded after the last kernel
  // that read each slot; the next upload into the slot waits for it
  cudaEvent_t slot_ev[16] = {};
  cudaEvent_t val_event = nullptr;  // batch validated (status readable)
  uint32_t* h_fail = nullptr;       // pinned copy of ctl->fail_epoch
  dg::VmmArray tcv[11];  // triangle counting scratch (CSR, orientation, probe order, flat wedge list)
  Buf ord[4];  // locality order of large batches: per-block partition counts / offsets,
               // permuted src, dst, weights (kernels_order.cu)
  Buf rh[4];  // re-sizing scratch
  Buf big;    // hub-row list (export, stats, TC orientation)
  // per-vertex re-sizing of long chains
  uint32_t* hot_flags = nullptr;
  uint64_t hot_words = 0;
  uint32_t* hot_list = nullptr;
  uint32_t hot_cap = 65536;
  uint32_t hot_steps = 4;      // 0 = off
  // mapped pinned {hot_count, hot_pairs, bump[3], epoch}, written by the insert's fixup
  // kernel (read by the host without a copy; it may lag behind the stream, which only
  // delays re-sizing and keeps the cursor bound conservative)
  uint32_t* h_hot = nullptr;
  uint32_t* d_hot = nullptr;   // its device alias
  bool in_rehash = false;
  cudaStream_t cstream[2] = {nullptr, nullptr};  // host-buffer pipeline: upload, download
  std::vector<cudaEvent_t> pipe_ev;

  dg::Router* router = nullptr;

  // instrumentation (dg_profile_*)
  bool prof = false;
  uint64_t prof_launch0 = 0;
  std::vector<cudaEvent_t> prof_ev[5];  // start/stop pairs per kernel kind
  std::vector<cudaEvent_t> prof_pool;   // recycled events (none created on the hot path)

  dg::Tables tables() const {
    dg::Tables t;
    t.dir = reinterpret_cast<dg::DirEntry*>(dir.ptr());
    t.home = adaptive ? nullptr : reinterpret_cast<uint32_t*>(home.ptr());
    t.nbs = adaptive ? nullptr : reinterpret_cast<uint8_t*>(nbsv.ptr());
    t.deg = reinterpret_cast<uint32_t*>(degv.ptr());
    t.hw = (adaptive || !DG_HOME_DEG) ? 0u : (uint32_t)(bucket_bytes / 4);
    for (int c = 0; c < dg::kClasses; ++c) {
      t.pool[c] = c < ncls ? reinterpret_cast<uint32_t*>(pool[c].ptr()) : nullptr;
      t.stack[c] = c < ncls ? reinterpret_cast<uint32_t*>(stack[c].ptr()) : nullptr;
      t.cap[c] = c < ncls ? cap[c] : 0;
    }
    t.ctl = ctl;
    t.ret_list = ret_list;
    t.rows = rows;
    t.nranks = nranks;
    t.hot_flags = hot_steps ? hot_flags : nullptr;
    t.hot_list = hot_list;
    t.hot_cap = hot_cap;
    t.hot_steps = hot_steps;
    return t;
  }
};

namespace dg {

inline uint64_t rows_for(uint64_t nv, uint32_t nranks, uint32_t rank) {
  return nv > rank ? (nv - rank + nranks - 1) / nranks : 0;
}

enum ProfKind { PROF_INSERT = 0, PROF_DELETE = 1, PROF_QUERY = 2, PROF_VDEL = 3, PROF_TC = 4 };
// record an event of kind k on s if instrumentation is enabled
void prof_mark(dg_graph g, int k, cudaStream_t s);

// internal entry points shared by api.cu and router.cu
dg_status grow_pool(dg_graph g, int c, uint64_t min_buckets, cudaStream_t s);
dg_status rehash_hot(dg_graph g, cudaStream_t s);
dg_status rehash_rows(dg_graph g, uint32_t n, bool flush, cudaStream_t s);
// fuse_validate: the insert launch validates the batch itself (small batches, EdgeBatch)
dg_status local_insert(dg_graph g, const uint32_t* src, const uint32_t* dst, const uint32_t* w,
                       uint64_t n, bool mirror, uint32_t epoch, cudaStream_t s, bool fuse_validate = false);
// the allocation part of local_insert for n_ops ops, done ahead (the router calls it
// before the exchange so nothing device-synchronising runs after its scatter)
dg_status prepare_insert(dg_graph g, uint64_t n_ops, cudaStream_t s);
// validate: run the batch validation (Q7) first; note: snapshot its verdict for
// validation_status() (api.cu order_batch)
// validation + insert of a local (not routed) batch, in locality order when it pays
dg_status validated_insert(dg_graph g, const uint32_t* src, const uint32_t* dst, const uint32_t* w,
                           uint64_t n, uint32_t epoch, bool note, cudaStream_t s);
dg_status local_delete(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                       bool mirror, uint32_t epoch, cudaStream_t s, bool validate, bool note);
dg_status local_query(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                      uint8_t* found, uint32_t* wout, uint32_t epoch, cudaStream_t s);

}  // namespace dg
