// router.cu — multi-GPU batch router (placeholder: single-GPU build).
#include "graph.h"
#include "router.h"

namespace dg {

struct Router {};

dg_status router_unique_id(void*) { return DG_ERR_UNSUPPORTED; }
dg_status router_create(dg_graph, const void*, Router**) { return DG_ERR_UNSUPPORTED; }
void router_destroy(Router* r) { delete r; }
dg_status router_insert(dg_graph, const uint32_t*, const uint32_t*, const uint32_t*, uint64_t,
                        uint32_t, cudaStream_t) {
  return DG_ERR_UNSUPPORTED;
}
dg_status router_delete(dg_graph, const uint32_t*, const uint32_t*, uint64_t, uint32_t,
                        cudaStream_t) {
  return DG_ERR_UNSUPPORTED;
}
dg_status router_query(dg_graph, const uint32_t*, const uint32_t*, uint64_t, uint8_t*, uint32_t*,
                       uint32_t, cudaStream_t) {
  return DG_ERR_UNSUPPORTED;
}
dg_status router_allgather_ids(dg_graph, const uint32_t*, uint64_t, const uint32_t**, uint64_t*,
                               cudaStream_t) {
  return DG_ERR_UNSUPPORTED;
}
dg_status router_sum_u64(dg_graph, uint64_t*, cudaStream_t) { return DG_ERR_UNSUPPORTED; }
dg_status router_max_u64(dg_graph, uint64_t*, cudaStream_t) { return DG_ERR_UNSUPPORTED; }

}  // namespace dg
