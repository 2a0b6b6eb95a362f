// vmm.cu — see vmm.h.
#include "vmm.h"

#include <algorithm>
#include <mutex>

namespace dg {
namespace {

struct Driver {
  decltype(&cuMemAddressReserve) AddressReserve = nullptr;
  decltype(&cuMemAddressFree) AddressFree = nullptr;
  decltype(&cuMemCreate) Create = nullptr;
  decltype(&cuMemRelease) Release = nullptr;
  decltype(&cuMemMap) Map = nullptr;
  decltype(&cuMemUnmap) Unmap = nullptr;
  decltype(&cuMemSetAccess) SetAccess = nullptr;
  decltype(&cuMemGetAllocationGranularity) GetGranularity = nullptr;
  bool ok = false;
};

template <typename F>
bool resolve(const char* name, F& fn) {
  void* p = nullptr;
  cudaDriverEntryPointQueryResult q;
  if (cudaGetDriverEntryPoint(name, &p, cudaEnableDefault, &q) != cudaSuccess ||
      q != cudaDriverEntryPointSuccess || !p)
    return false;
  fn = reinterpret_cast<F>(p);
  return true;
}

const Driver& driver() {
  static Driver d;
  static std::once_flag once;
  std::call_once(once, [] {
    d.ok = resolve("cuMemAddressReserve", d.AddressReserve) &&
           resolve("cuMemAddressFree", d.AddressFree) && resolve("cuMemCreate", d.Create) &&
           resolve("cuMemRelease", d.Release) && resolve("cuMemMap", d.Map) &&
           resolve("cuMemUnmap", d.Unmap) && resolve("cuMemSetAccess", d.SetAccess) &&
           resolve("cuMemGetAllocationGranularity", d.GetGranularity);
  });
  return d;
}

CUmemAllocationProp prop_for(int device) {
  CUmemAllocationProp p = {};
  p.type = CU_MEM_ALLOCATION_TYPE_PINNED;
  p.location.type = CU_MEM_LOCATION_TYPE_DEVICE;
  p.location.id = device;
  return p;
}

}  // namespace

cudaError_t VmmArray::reserve(int device, size_t max_bytes) {
  const Driver& d = driver();
  if (!d.ok) return cudaErrorNotSupported;
  device_ = device;
  CUmemAllocationProp p = prop_for(device);
  size_t g = 0;
  if (d.GetGranularity(&g, &p, CU_MEM_ALLOC_GRANULARITY_RECOMMENDED) != CUDA_SUCCESS || !g)
    return cudaErrorMemoryAllocation;
  gran_ = g;
  reserved_ = (std::max<size_t>(max_bytes, g) + g - 1) / g * g;
  if (d.AddressReserve(&base_, reserved_, g, 0, 0) != CUDA_SUCCESS) {
    base_ = 0;
    reserved_ = 0;
    return cudaErrorMemoryAllocation;
  }
  va_bytes_ = reserved_;
  return cudaSuccess;
}

cudaError_t VmmArray::reserve_pair(int device, size_t max_bytes, size_t hi_offset,
                                   size_t hi_bytes, VmmArray& hi) {
  const Driver& d = driver();
  if (!d.ok) return cudaErrorNotSupported;
  device_ = hi.device_ = device;
  CUmemAllocationProp p = prop_for(device);
  size_t g = 0;
  if (d.GetGranularity(&g, &p, CU_MEM_ALLOC_GRANULARITY_RECOMMENDED) != CUDA_SUCCESS || !g)
    return cudaErrorMemoryAllocation;
  gran_ = hi.gran_ = g;
  reserved_ = (std::max<size_t>(max_bytes, g) + g - 1) / g * g;
  hi.reserved_ = (std::max<size_t>(hi_bytes, g) + g - 1) / g * g;
  if (hi_offset % g || reserved_ > hi_offset) return cudaErrorInvalidValue;
  const size_t total = hi_offset + hi.reserved_;
  if (d.AddressReserve(&base_, total, g, 0, 0) != CUDA_SUCCESS) {
    base_ = 0;
    reserved_ = hi.reserved_ = 0;
    return cudaErrorMemoryAllocation;
  }
  va_bytes_ = total;
  hi.base_ = base_ + hi_offset;
  hi.va_bytes_ = 0;
  return cudaSuccess;
}

cudaError_t VmmArray::ensure(size_t bytes, int fill, cudaStream_t stream) {
  if (bytes <= mapped_) return cudaSuccess;
  const Driver& d = driver();
  if (!base_) return cudaErrorInvalidValue;
  if (bytes > reserved_) return cudaErrorMemoryAllocation;
  // grow by at least 1/4 of what is mapped, in granularity multiples
  size_t want = std::max(bytes, mapped_ + mapped_ / 4);
  want = std::min(reserved_, (want + gran_ - 1) / gran_ * gran_);
  const size_t chunk = want - mapped_;
  CUmemAllocationProp p = prop_for(device_);
  CUmemGenericAllocationHandle h;
  if (d.Create(&h, chunk, &p, 0) != CUDA_SUCCESS) return cudaErrorMemoryAllocation;
  if (d.Map(base_ + mapped_, chunk, 0, h, 0) != CUDA_SUCCESS) {
    d.Release(h);
    return cudaErrorMemoryAllocation;
  }
  CUmemAccessDesc a = {};
  a.location.type = CU_MEM_LOCATION_TYPE_DEVICE;
  a.location.id = device_;
  a.flags = CU_MEM_ACCESS_FLAGS_PROT_READWRITE;
  if (d.SetAccess(base_ + mapped_, chunk, &a, 1) != CUDA_SUCCESS) {
    d.Unmap(base_ + mapped_, chunk);
    d.Release(h);
    return cudaErrorMemoryAllocation;
  }
  handles_.push_back(h);
  sizes_.push_back(chunk);
  if (fill >= 0) {
    cudaError_t e = cudaMemsetAsync(reinterpret_cast<void*>(base_ + mapped_), fill, chunk, stream);
    if (e != cudaSuccess) return e;
  }
  mapped_ = want;
  return cudaSuccess;
}

void VmmArray::release() {
  if (!base_) return;
  const Driver& d = driver();
  size_t off = 0;
  for (size_t i = 0; i < handles_.size(); ++i) {
    d.Unmap(base_ + off, sizes_[i]);
    d.Release(handles_[i]);
    off += sizes_[i];
  }
  if (va_bytes_) d.AddressFree(base_, va_bytes_);
  handles_.clear();
  sizes_.clear();
  base_ = 0;
  reserved_ = mapped_ = va_bytes_ = 0;
}

}  // namespace dg
