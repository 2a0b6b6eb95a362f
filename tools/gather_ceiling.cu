// gather_ceiling.cu — measured random-gather ceiling on this GPU:
// random S-byte reads (S = 32/64/128, one S-byte block per group of S/16 lanes
// with 16-B lane loads) over a buffer >= 4x L2, enough loads in flight to
// saturate.  This is the achievable bandwidth for hash probes, reported beside the
// STREAM-copy peak of MEASURED_PEAKS.json.  Build/run:
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/gc tools/gather_ceiling.cu && /tmp/gc
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ uint64_t mix(uint64_t x) {
  x ^= x >> 33; x *= 0xff51afd7ed558ccdULL; x ^= x >> 33; x *= 0xc4ceb9fe1a85ec53ULL;
  return x ^ (x >> 33);
}

template <int G, int U>
__global__ void gather(const uint4* __restrict__ buf, uint64_t nblocks, uint64_t iters,
                       unsigned long long* sink) {
  const uint32_t lane = threadIdx.x & 31, gl = lane & (G - 1);
  const uint64_t gid = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) / G;
  uint32_t acc = 0;
  for (uint64_t it = 0; it < iters; ++it) {
    uint4 q[U];
#pragma unroll
    for (int k = 0; k < U; ++k) {
      const uint64_t b = ((mix(gid * 1315423911ULL + it * U + k) & 0xFFFFFFFFull) * nblocks) >> 32;
      q[k] = __ldg(buf + b * G + gl);
    }
#pragma unroll
    for (int k = 0; k < U; ++k) acc += q[k].x ^ q[k].w;
  }
  if (acc == 0x12345678u) atomicAdd(sink, 1ull);
}

template <int G, int U>
double run(const uint4* buf, uint64_t bytes, int sms) {
  const uint64_t nblocks = bytes / (16 * G);
  const int blocks = sms * 8, threads = 256;
  const uint64_t groups = (uint64_t)blocks * threads / G;
  const uint64_t iters = 64;
  unsigned long long* sink;
  cudaMalloc(&sink, 8);
  gather<G, U><<<blocks, threads>>>(buf, nblocks, 4, sink);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  cudaEventRecord(a);
  gather<G, U><<<blocks, threads>>>(buf, nblocks, iters, sink);
  cudaEventRecord(b);
  cudaEventSynchronize(b);
  float ms = 0;
  cudaEventElapsedTime(&ms, a, b);
  cudaFree(sink);
  const double moved = (double)groups * iters * U * 16 * G;
  return moved / (ms * 1e-3) / 1e9;
}

int main() {
  int dev = 0;
  cudaDeviceProp p;
  cudaGetDeviceProperties(&p, dev);
  const uint64_t bytes = (uint64_t)p.l2CacheSize * 32;  // >= 4x L2
  uint4* buf;
  if (cudaMalloc(&buf, bytes) != cudaSuccess) return 1;
  cudaMemset(buf, 1, bytes);
  printf("{\"gpu\": \"%s\", \"l2_bytes\": %d, \"buffer_bytes\": %llu, \"sms\": %d, \"GBs\": {",
         p.name, p.l2CacheSize, (unsigned long long)bytes, p.multiProcessorCount);
  printf("\"S32_U4\": %.1f, ", run<2, 4>(buf, bytes, p.multiProcessorCount));
  printf("\"S64_U4\": %.1f, ", run<4, 4>(buf, bytes, p.multiProcessorCount));
  printf("\"S128_U2\": %.1f, ", run<8, 2>(buf, bytes, p.multiProcessorCount));
  printf("\"S128_U4\": %.1f, ", run<8, 4>(buf, bytes, p.multiProcessorCount));
  printf("\"S128_U8\": %.1f}}\n", run<8, 8>(buf, bytes, p.multiProcessorCount));
  cudaFree(buf);
  return 0;
}
