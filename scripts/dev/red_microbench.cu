// L2 fp64 RED throughput micro-benchmark (DESIGN.md §13 "second roofline line").
// Every lane issues fire-and-forget fp64 atomicAdd (RED.E.ADD.F64) to scattered addresses of
// a tally-sized array, the access pattern of the history kernel's per-facet flush: the 32
// lanes of a warp hit 32 unrelated cells.  Reports REDs per second for several footprints
// (L2-resident and HBM-sized).  Build: nvcc -O3 -gencode arch=compute_100a,code=sm_100a
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>

__device__ __forceinline__ uint32_t mix(uint32_t x) {
  x ^= x >> 16; x *= 0x7feb352dU; x ^= x >> 15; x *= 0x846ca68bU; x ^= x >> 16; return x;
}

// walk: each lane moves like a particle, +1 or +nx cells per RED, from a scattered start
__global__ void red_kernel(double* t, uint32_t mask, uint32_t nx, int iters, int walk) {
  const uint32_t tid = blockIdx.x * blockDim.x + threadIdx.x;
  uint32_t c = mix(tid * 2654435761u + 12345u) & mask;
  for (int k = 0; k < iters; ++k) {
    uint32_t a = walk ? c : (mix(c + k) & mask);
    asm volatile("red.global.add.f64 [%0], %1;" :: "l"(t + a), "d"(1.0) : "memory");
    if (walk) c = (c + ((mix(tid + k) & 1) ? 1u : nx)) & mask;
  }
}

int main() {
  int sms = 0; cudaDeviceGetAttribute(&sms, cudaDevAttrMultiProcessorCount, 0);
  const size_t max_cells = 1u << 24;   // 16.8M doubles = 134 MB (the 4000^2 tally is 128 MB)
  double* t; cudaMalloc(&t, max_cells * sizeof(double));
  cudaMemset(t, 0, max_cells * sizeof(double));
  cudaEvent_t e0, e1; cudaEventCreate(&e0); cudaEventCreate(&e1);
  const int threads = 256, blocks = sms * 8, iters = 2048;
  printf("{\"sms\": %d, \"results\": [", sms);
  bool first = true;
  for (int walk = 0; walk < 2; ++walk)
    for (int lg = 16; lg <= 24; lg += 2) {
      const uint32_t mask = (1u << lg) - 1;
      red_kernel<<<blocks, threads>>>(t, mask, 4000, iters, walk);   // warm-up
      cudaEventRecord(e0);
      for (int r = 0; r < 5; ++r) red_kernel<<<blocks, threads>>>(t, mask, 4000, iters, walk);
      cudaEventRecord(e1); cudaEventSynchronize(e1);
      float ms; cudaEventElapsedTime(&ms, e0, e1);
      const double reds = 5.0 * blocks * threads * (double)iters;
      printf("%s{\"pattern\": \"%s\", \"footprint_MB\": %.1f, \"reds_per_s\": %.4e}",
             first ? "" : ", ", walk ? "walk" : "random", (double)(1u << lg) * 8 / 1e6,
             reds / (ms * 1e-3));
      first = false;
    }
  printf("], \"err\": \"%s\"}\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}
