// Host round-trip latency (tools only): kernel + cudaStreamSynchronize, with the kernel storing
// to device memory / to pinned host memory, or a 4-B cudaMemcpyAsync D2H -- with and without
// a large D2H copy in flight on another stream.
#include <cuda_runtime.h>
#include <stdio.h>
#include <chrono>
__global__ void k_store(unsigned *p, unsigned v) { if (threadIdx.x == 0) *p = v; }
__global__ void k_copy(unsigned *dst, const unsigned *src) { if (threadIdx.x == 0) *dst = *src; }
int main() {
  size_t big = 256ull << 20;
  void *d_big, *h_big;
  cudaMalloc(&d_big, big);
  cudaMallocHost(&h_big, big);
  unsigned *d_w, *h_w;
  cudaMalloc(&d_w, 64);
  cudaMallocHost(&h_w, 64);
  cudaStream_t a, b;
  cudaStreamCreateWithFlags(&a, cudaStreamNonBlocking);
  cudaStreamCreateWithFlags(&b, cudaStreamNonBlocking);
  for (int busy = 0; busy < 2; ++busy) {
    for (int mode = 0; mode < 3; ++mode) {
      cudaDeviceSynchronize();
      if (busy)
        for (int i = 0; i < 6; ++i) cudaMemcpyAsync(h_big, d_big, big, cudaMemcpyDeviceToHost, a);
      const int n = 50;
      auto t0 = std::chrono::steady_clock::now();
      for (int i = 0; i < n; ++i) {
        if (mode == 0) k_store<<<1, 32, 0, b>>>(d_w, i);
        else if (mode == 1) k_copy<<<1, 32, 0, b>>>(h_w, d_w);
        else cudaMemcpyAsync(h_w, d_w, 4, cudaMemcpyDeviceToHost, b);
        cudaStreamSynchronize(b);
      }
      auto t1 = std::chrono::steady_clock::now();
      printf("%s %-22s %8.1f us/roundtrip\n", busy ? "busy" : "idle",
             mode == 0 ? "kernel->device mem" : mode == 1 ? "kernel->pinned host" : "memcpyAsync 4B D2H",
             std::chrono::duration<double, std::micro>(t1 - t0).count() / n);
      cudaDeviceSynchronize();
    }
  }
  return 0;
}
