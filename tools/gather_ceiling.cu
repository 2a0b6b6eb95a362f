// gather_ceiling.cu — measured random-gather ceiling on this GPU:
// random S-byte reads (S = 32/64/128, one S-byte block per group of S/16 lanes
// with 16-B lane loads) over a buffer >= 4x L2, enough loads in flight to
// saturate.  This is the achievable bandwidth for hash probes, reported beside the
// STREAM-copy peak of MEASURED_PEAKS.json.  The read-modify-write modes add, per
// gathered block, what an insert / delete adds per op: an 8-B store into the block
// (M = 1: dirties one sector that is written back) or a 64-bit CAS on it (M = 2),
// plus a fire-and-forget atomic on an L2-resident counter array (M = 3, the degree
// update) — the achievable op rate for the mutating probe kernels; M = 4 puts that
// counter in the last word of the gathered block (a degree kept in the home bucket).  Build/run:
//   nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/gc tools/gather_ceiling.cu && /tmp/gc
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ uint64_t mix(uint64_t x) {
  x ^= x >> 33; x *= 0xff51afd7ed558ccdULL; x ^= x >> 33; x *= 0xc4ceb9fe1a85ec53ULL;
  return x ^ (x >> 33);
}

template <int G, int U, int M>
__global__ void gather(uint4* __restrict__ buf, uint64_t nblocks, uint64_t iters,
                       unsigned long long* sink, uint32_t* cnt, uint32_t ncnt) {
  const uint32_t lane = threadIdx.x & 31, gl = lane & (G - 1);
  const uint64_t gid = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) / G;
  uint32_t acc = 0;
  for (uint64_t it = 0; it < iters; ++it) {
    uint4 q[U];
#pragma unroll
    for (int k = 0; k < U; ++k) {
      const uint64_t b = ((mix(gid * 1315423911ULL + it * U + k) & 0xFFFFFFFFull) * nblocks) >> 32;
      q[k] = M == 0 ? __ldg(buf + b * G + gl) : buf[b * G + gl];
    }
#pragma unroll
    for (int k = 0; k < U; ++k) acc += q[k].x ^ q[k].w;
    if (M > 0) {
      // the lane that owns op k (k-th lane of the group) mutates its block
#pragma unroll
      for (int k = 0; k < U; ++k) {
        if (gl != (uint32_t)(k % G)) continue;
        const uint64_t h = mix(gid * 1315423911ULL + it * U + k);
        const uint64_t b = ((h & 0xFFFFFFFFull) * nblocks) >> 32;
        unsigned long long* p = reinterpret_cast<unsigned long long*>(buf + b * G) + ((h >> 40) & (2 * G - 1));
        if (M == 1) {
          *p = (unsigned long long)(acc + k);
        } else {
          acc += (uint32_t)atomicCAS(p, (unsigned long long)q[k].x, (unsigned long long)(acc + k));
          if (M == 3) atomicAdd(cnt + ((h >> 8) % ncnt), 1u);
          // M = 4: the counter lives in the gathered block itself (last word)
          if (M == 4) atomicAdd(reinterpret_cast<uint32_t*>(buf + b * G) + 4 * G - 1, 1u);
        }
      }
    }
  }
  if (acc == 0x12345678u) atomicAdd(sink, 1ull);
}

// ---------------------------------------------------- cp.async.bulk mode ----
// Blackwell data movement instead of register loads: each warp keeps 2 x D random
// 128-B buckets in flight as 1-D bulk copies (cp.async.bulk, SASS UBLKCP) into a
// shared-memory ring, completion tracked by one mbarrier per stage (expect_tx),
// double-buffered: while stage s is consumed the other stage's copies are in
// flight.  In-flight requests per SM = warps x 2D, bounded by shared memory rather
// than registers x occupancy.
__device__ __forceinline__ uint32_t smem_u32(const void* p) {
  return (uint32_t)__cvta_generic_to_shared(p);
}

template <int D>
__global__ void gather_bulk(const uint4* __restrict__ buf, uint64_t nblocks, uint64_t iters,
                            unsigned long long* sink) {
  extern __shared__ __align__(128) unsigned char smem[];
  __shared__ __align__(8) unsigned long long bars[32][2];
  const uint32_t w = threadIdx.x >> 5, lane = threadIdx.x & 31;
  uint4* ring = reinterpret_cast<uint4*>(smem) + (size_t)w * 2 * D * 8;  // [stage][D][8]
  const uint64_t gw = ((uint64_t)blockIdx.x * blockDim.x + threadIdx.x) >> 5;
  const uint32_t b0 = smem_u32(&bars[w][0]), b1 = smem_u32(&bars[w][1]);
  if (lane == 0) {
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(b0));
    asm volatile("mbarrier.init.shared::cta.b64 [%0], 1;" ::"r"(b1));
    asm volatile("fence.mbarrier_init.release.cluster;");
  }
  __syncwarp();
  auto issue = [&](int st, uint64_t it) {
    const uint32_t bar = st ? b1 : b0;
    if (lane == 0)
      asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(bar),
                   "r"(D * 128) : "memory");
    __syncwarp();
    for (int k = lane; k < D; k += 32) {
      const uint64_t b = ((mix(gw * 2654435761ULL + it * D + k) & 0xFFFFFFFFull) * nblocks) >> 32;
      const uint32_t dst = smem_u32(ring + ((size_t)st * D + k) * 8);
      asm volatile(
          "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], 128, [%2];"
          ::"r"(dst), "l"(buf + b * 8), "r"(bar) : "memory");
    }
  };
  auto wait = [&](int st, uint32_t parity) {
    const uint32_t bar = st ? b1 : b0;
    asm volatile(
        "{\n .reg .pred p;\n WAIT_%=:\n"
        " mbarrier.try_wait.parity.shared::cta.b64 p, [%0], %1;\n"
        " @!p bra WAIT_%=;\n}" ::"r"(bar), "r"(parity) : "memory");
  };
  uint32_t acc = 0;
  issue(0, 0);
  issue(1, 1);
  for (uint64_t it = 0; it < iters; ++it) {
    const int st = (int)(it & 1);
    wait(st, (uint32_t)((it >> 1) & 1));
    for (int k = lane; k < D; k += 32) {
      const uint4 x = ring[((size_t)st * D + k) * 8 + (it & 7)];
      acc += x.x ^ x.w;
    }
    __syncwarp();
    if (it + 2 < iters + 2) issue(st, it + 2);
  }
  wait(0, (uint32_t)(((iters) >> 1) & 1));
  wait(1, (uint32_t)(((iters + 1) >> 1) & 1));
  if (acc == 0x12345678u) atomicAdd(sink, 1ull);
}

// G ops/s of the bulk-copy gather: D buckets per stage, `warps` warps per block
template <int D>
double run_bulk(const uint4* buf, uint64_t bytes, int sms, int bps, int warps) {
  const uint64_t nblocks = bytes / 128;
  const int threads = 32 * warps;
  const size_t smem = (size_t)warps * 2 * D * 128;
  if (cudaFuncSetAttribute(gather_bulk<D>, cudaFuncAttributeMaxDynamicSharedMemorySize,
                           (int)smem) != cudaSuccess)
    return 0.0;
  unsigned long long* sink;
  cudaMalloc(&sink, 8);
  const uint64_t iters = 64;
  gather_bulk<D><<<sms * bps, threads, smem>>>(buf, nblocks, 4, sink);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  cudaEventRecord(a);
  gather_bulk<D><<<sms * bps, threads, smem>>>(buf, nblocks, iters, sink);
  const cudaError_t le = cudaGetLastError();  // e.g. more shared memory than an SM has
  cudaEventRecord(b);
  if (le != cudaSuccess || cudaEventSynchronize(b) != cudaSuccess) {
    cudaGetLastError();
    cudaFree(sink);
    return 0.0;
  }
  float ms = 0;
  cudaEventElapsedTime(&ms, a, b);
  cudaFree(sink);
  // every iteration consumes one stage of D buckets (the two issued past the end are
  // waited for but not counted)
  return (double)sms * bps * warps * iters * D / (ms * 1e-3) / 1e9;
}

template <int G, int U, int M = 0>
double run(uint4* buf, uint64_t bytes, int sms, uint32_t* cnt = nullptr, uint32_t ncnt = 1,
           double* gops = nullptr, int bps = 8) {
  const uint64_t nblocks = bytes / (16 * G);
  const int blocks = sms * bps, threads = 256;
  const uint64_t groups = (uint64_t)blocks * threads / G;
  const uint64_t iters = 64;
  unsigned long long* sink;
  cudaMalloc(&sink, 8);
  gather<G, U, M><<<blocks, threads>>>(buf, nblocks, 4, sink, cnt, ncnt);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  cudaEventRecord(a);
  gather<G, U, M><<<blocks, threads>>>(buf, nblocks, iters, sink, cnt, ncnt);
  cudaEventRecord(b);
  cudaEventSynchronize(b);
  float ms = 0;
  cudaEventElapsedTime(&ms, a, b);
  cudaFree(sink);
  const double moved = (double)groups * iters * U * 16 * G;
  if (gops) *gops = (double)groups * iters * U / (ms * 1e-3) / 1e9;
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
  printf("\"S128_U8\": %.1f}, ", run<8, 8>(buf, bytes, p.multiProcessorCount));
  // read-modify-write modes (128-B blocks): G ops/s
  uint32_t* cnt;
  const uint32_t ncnt = 4847571;  // one counter per cfg2 row (19 MB, L2-resident)
  cudaMalloc(&cnt, 4ull * ncnt);
  cudaMemset(cnt, 0, 4ull * ncnt);
  // best over in-flight depth U and resident blocks per SM
  const int sm = p.multiProcessorCount;
  double best[5] = {0, 0, 0, 0, 0};
  for (int bps : {4, 8, 16}) {
    double g;
#define DG_TRY(U_)                                                       \
    run<8, U_, 0>(buf, bytes, sm, cnt, ncnt, &g, bps); best[0] = g > best[0] ? g : best[0]; \
    run<8, U_, 1>(buf, bytes, sm, cnt, ncnt, &g, bps); best[1] = g > best[1] ? g : best[1]; \
    run<8, U_, 2>(buf, bytes, sm, cnt, ncnt, &g, bps); best[2] = g > best[2] ? g : best[2]; \
    run<8, U_, 3>(buf, bytes, sm, cnt, ncnt, &g, bps); best[3] = g > best[3] ? g : best[3]; \
    run<8, U_, 4>(buf, bytes, sm, cnt, ncnt, &g, bps); best[4] = g > best[4] ? g : best[4];
    DG_TRY(2) DG_TRY(4) DG_TRY(8)
#undef DG_TRY
  }
  printf("\"G_ops_s_S128\": {\"read\": %.2f, \"read_store8\": %.2f, \"read_cas8\": %.2f, "
         "\"read_cas8_counter\": %.2f, \"read_cas8_counter_in_block\": %.2f}, ", best[0], best[1], best[2],
         best[3], best[4]);
  // cp.async.bulk + mbarrier gather (128-B buckets into shared memory): best over
  // buckets per stage D, warps per block and blocks per SM
  double bb = 0;
  char cfgs[64] = "";
  for (int bps : {1, 2, 4}) {
    for (int warps : {4, 8}) {
      double g;
#define DG_TRYB(D_)                                                                    \
      g = run_bulk<D_>(buf, bytes, sm, bps, warps);                                    \
      if (g > bb) { bb = g; snprintf(cfgs, sizeof cfgs, "D%d_w%d_b%d", D_, warps, bps); }
      DG_TRYB(8) DG_TRYB(16) DG_TRYB(32) DG_TRYB(64)
#undef DG_TRYB
    }
  }
  printf("\"G_ops_s_S128_bulk\": {\"read\": %.2f, \"best\": \"%s\"}}\n", bb, cfgs);
  cudaFree(cnt);
  cudaFree(buf);
  return 0;
}
