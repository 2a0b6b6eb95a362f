// comm.h — the collectives the batch router needs (router.cu), behind one interface
// with two transports:
//   * NcclComm   — one process per GPU (the production layout): NCCL over NVLink /
//                  NVSwitch; receive windows are exported with CUDA IPC.
//   * GroupComm  — an in-process rank group (dg_group, include/dg.h): the P ranks are
//                  host threads of ONE process, each with its own handle and stream,
//                  on one or several GPUs.  Collectives meet at a host barrier and move
//                  bytes with device copies; receive windows are shared by pointer.
//                  This is how the P >= 2 router (partition, fused window scatter, copy
//                  exchange, answer return, unpermute) runs on a single B200.
// The paper has a single GPU; the router is the north_star extension.
#pragma once
#include <cstddef>
#include <cstdint>

#include <cuda_runtime.h>

#include "../../include/dg.h"

namespace dg {

struct Comm {
  virtual ~Comm() = default;
  virtual uint32_t size() const = 0;
  virtual uint32_t rank() const = 0;
  // every rank contributes `bytes` from device buffer `send`; `recv` (device, P*bytes)
  // receives them in rank order.  Stream-ordered on s (GroupComm: completes on return).
  virtual dg_status allgather(const void* send, void* recv, size_t bytes, cudaStream_t s) = 0;
  // grouped point-to-point: between group_start and group_end, the k-th send from q to
  // p matches the k-th recv at p from q (byte counts must agree)
  virtual dg_status group_start() = 0;
  virtual dg_status send(const void* buf, size_t bytes, uint32_t peer, cudaStream_t s) = 0;
  virtual dg_status recv(void* buf, size_t bytes, uint32_t peer, cudaStream_t s) = 0;
  virtual dg_status group_end(cudaStream_t s) = 0;
  // in-place all-reduce of one u64 in device memory (sum or max)
  virtual dg_status allreduce_u64(uint64_t* dev, bool max, cudaStream_t s) = 0;
  // collective: map every rank's receive window so this rank can store into it;
  // peers[q] = rank q's window in this rank's address space (peers[rank] = mine).
  // *fail (same on every rank) = some rank could not map a peer.
  virtual dg_status map_windows(char* mine, char** peers, bool* fail, cudaStream_t s) = 0;
  virtual void unmap_windows(char** peers) = 0;
  // In-process groups only (no-op for NCCL): a host barrier every rank passes after
  // its device-synchronising work (allocation) for a batch and before it enqueues
  // the fused scatter.  Ranks sharing one device would otherwise deadlock: a rank
  // blocked in a device-wide synchronisation waits for a peer's spin-wait kernel,
  // which waits for this rank's not-yet-launched scatter.
  virtual dg_status quiesce() { return DG_OK; }
  // How the fused exchange waits for the peers' stores into this rank's window.
  // false: a one-thread device kernel spins on the window's arrival counter (separate
  // processes / contexts).  true: in-process groups order the streams with CUDA events
  // instead (streams of one context can share a hardware queue, where a spinning
  // kernel would block the very peer kernel it waits for): wait_peers records `ev`
  // on s after this rank's stores, and makes s wait for every peer's event.
  virtual bool host_ordered() const { return false; }
  virtual dg_status wait_peers(cudaEvent_t ev, cudaStream_t s) { return DG_ERR_UNSUPPORTED; }
};

// NCCL transport (dlopen'ed NCCL; unique_id = 128-byte ncclUniqueId)
bool nccl_available();
dg_status nccl_unique_id(void* out128);
dg_status nccl_comm_create(const void* unique_id, uint32_t P, uint32_t rank, Comm** out);

// in-process group transport
dg_status group_comm_create(dg_group grp, uint32_t P, uint32_t rank, int device, Comm** out);

}  // namespace dg
