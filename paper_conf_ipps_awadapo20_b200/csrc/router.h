// router.h — multi-GPU batch router: shards edge ops by source vertex
// (owner(u) = u mod P, local row = u / P) with an NCCL all-to-all over NVLink.
// The paper has a single GPU; this is the B200-node extension named
// by BASELINE.json's north_star.
#pragma once
#include <cstdint>

#include <cuda_runtime.h>

#include "../../include/dg.h"

namespace dg {

struct Router;

dg_status router_unique_id(void* out128);
dg_status router_create(dg_graph g, const void* unique_id, Router** out);
void router_destroy(Router* r);
// collective, after g->router is set: map every peer's receive window (CUDA IPC over
// NVLink) for the fused exchange; falls back to the NCCL exchange if any rank cannot
// (or DG_ROUTER=nccl).  router_fused() tells which path is active.
dg_status router_setup_fused(dg_graph g, cudaStream_t s);
bool router_fused(const Router* r);

// collective edge ops: each rank passes its slice; validation is agreed on by all
dg_status router_insert(dg_graph g, const uint32_t* src, const uint32_t* dst, const uint32_t* w,
                        uint64_t n, uint32_t epoch, cudaStream_t s);
dg_status router_delete(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                        uint32_t epoch, cudaStream_t s);
dg_status router_query(dg_graph g, const uint32_t* src, const uint32_t* dst, uint64_t n,
                       uint8_t* found, uint32_t* wout, uint32_t epoch, cudaStream_t s);
// concatenation of every rank's array (rank order); slot selects one of two
// router-owned output buffers (0: ids, 1: a parallel array such as hints)
dg_status router_allgather_u32(dg_graph g, const uint32_t* data, uint64_t n, int slot,
                               const uint32_t** all, uint64_t* all_n, cudaStream_t s);
dg_status router_sum_u64(dg_graph g, uint64_t* v, cudaStream_t s);
dg_status router_max_u64(dg_graph g, uint64_t* v, cudaStream_t s);

}  // namespace dg
