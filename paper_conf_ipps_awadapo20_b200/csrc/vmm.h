// vmm.h — growable device arrays on CUDA virtual memory management.
//
// A large virtual range is reserved once; physical memory is created and mapped
// in chunks at the end as the array grows.  Growth therefore never copies and
// never moves data, so bucket indices and directory pointers stay valid (the
// paper instead copies the vertex dictionary on growth; the result
// is the same, the cost is not).  Driver entry points are resolved at run time
// through cudaGetDriverEntryPoint, so libdg.so has no link-time dependency on
// libcuda (it still loads on a machine without a GPU).
#pragma once
#include <cstddef>
#include <cstdint>
#include <vector>

#include <cuda.h>
#include <cuda_runtime.h>

namespace dg {

class VmmArray {
 public:
  VmmArray() = default;
  ~VmmArray() { release(); }
  VmmArray(const VmmArray&) = delete;
  VmmArray& operator=(const VmmArray&) = delete;

  // Reserve `max_bytes` of virtual address space on `device`.
  cudaError_t reserve(int device, size_t max_bytes);
  // One reservation for two arrays: this one at its start (`max_bytes`) and `hi` at
  // byte offset `hi_offset` (`hi_bytes`), so that hi.ptr() - ptr() == hi_offset
  // exactly (the home buckets sit 2^31 buckets after the pool: one address formula
  // serves both, dg_common.cuh Geo).  Release `hi` before this array.
  cudaError_t reserve_pair(int device, size_t max_bytes, size_t hi_offset, size_t hi_bytes,
                           VmmArray& hi);
  // Ensure at least `bytes` are mapped; new memory is filled with `fill` (a byte
  // value, or -1 for no fill) on `stream`.
  cudaError_t ensure(size_t bytes, int fill, cudaStream_t stream);
  void release();

  void* ptr() const { return reinterpret_cast<void*>(base_); }
  size_t mapped() const { return mapped_; }
  size_t reserved() const { return reserved_; }
  size_t granularity() const { return gran_; }

 private:
  CUdeviceptr base_ = 0;
  size_t reserved_ = 0;
  size_t va_bytes_ = 0;  // bytes of the reservation this array frees (0: a view into another's)
  size_t mapped_ = 0;
  size_t gran_ = 0;
  int device_ = 0;
  std::vector<CUmemGenericAllocationHandle> handles_;
  std::vector<size_t> sizes_;
};

}  // namespace dg
