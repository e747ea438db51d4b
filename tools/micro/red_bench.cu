// Random-RED throughput microbenchmark (tools only; not part of the library).
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>
__device__ __forceinline__ uint64_t mix(uint64_t z) {
  z += 0x9E3779B97F4A7C15ull; z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull; return z ^ (z >> 31);
}
template <typename T>
__global__ void k_red(T *y, uint64_t n_ops, uint64_t mask) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n_ops; i += (uint64_t)gridDim.x * blockDim.x)
    atomicAdd(&y[mix(i) & mask], (T)1);
}
template <typename T>
static float run(uint64_t elems, uint64_t ops) {
  T *y; cudaMalloc(&y, elems * sizeof(T)); cudaMemset(y, 0, elems * sizeof(T));
  cudaEvent_t a, b; cudaEventCreate(&a); cudaEventCreate(&b);
  k_red<T><<<148 * 8, 256>>>(y, ops, elems - 1);
  cudaEventRecord(a);
  k_red<T><<<148 * 8, 256>>>(y, ops, elems - 1);
  cudaEventRecord(b); cudaEventSynchronize(b);
  float ms; cudaEventElapsedTime(&ms, a, b); cudaFree(y); return ms;
}
int main() {
  const uint64_t ops = 134217728;
  for (uint64_t mb : {4ull, 32ull, 64ull, 128ull, 256ull}) {
    uint64_t e8 = mb * 1024 * 1024 / 8, e4 = mb * 1024 * 1024 / 4;
    printf("%4llu MB: u64 %.3f ms (%.1f G/s)  f64 %.3f ms  u32 %.3f ms  f32 %.3f ms\n", (unsigned long long)mb,
           run<unsigned long long>(e8, ops), ops / 1e6 / run<unsigned long long>(e8, ops), run<double>(e8, ops),
           run<unsigned int>(e4, ops), run<float>(e4, ops));
  }
  return 0;
}
