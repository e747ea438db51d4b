// Stream-ordered pool reuse probe (tools only): does a freed big block serve smaller requests
// without new mappings?  nvcc -gencode arch=compute_100a,code=sm_100a tools/micro/pool_probe.cu
#include <chrono>
#include <cstdio>
#include <cstdint>
#include <cuda_runtime.h>
static double ms(std::chrono::steady_clock::time_point a) {
  return std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - a).count();
}
int main() {
  cudaMemPool_t pool;
  cudaMemPoolProps pp{};
  pp.allocType = cudaMemAllocationTypePinned;
  pp.location.type = cudaMemLocationTypeDevice;
  pp.location.id = 0;
  cudaMemPoolCreate(&pool, &pp);
  uint64_t thr = ~0ull;
  cudaMemPoolSetAttribute(pool, cudaMemPoolAttrReleaseThreshold, &thr);
  cudaStream_t s;
  cudaStreamCreate(&s);
  auto alloc = [&](size_t mb, const char *what) {
    void *p;
    auto t = std::chrono::steady_clock::now();
    cudaMallocFromPoolAsync(&p, mb << 20, pool, s);
    printf("%-28s %6zu MiB: %.3f ms\n", what, mb, ms(t));
    return p;
  };
  void *a = alloc(4096, "fresh");
  cudaFreeAsync(a, s);
  cudaStreamSynchronize(s);
  void *b = alloc(512, "after free 4G");
  void *c = alloc(1024, "after free 4G");
  void *d = alloc(2048, "after free 4G");
  void *e = alloc(512, "after free 4G (over)");
  cudaFreeAsync(b, s); cudaFreeAsync(c, s); cudaFreeAsync(d, s); cudaFreeAsync(e, s);
  cudaStreamSynchronize(s);
  void *f = alloc(3072, "after frees of 4 blocks");
  void *h = alloc(1024, "after frees of 4 blocks");
  cudaFreeAsync(f, s); cudaFreeAsync(h, s);
  cudaStreamSynchronize(s);
  void *x = alloc(4096, "whole again");
  cudaFreeAsync(x, s);
  cudaStreamSynchronize(s);
  cudaStream_t s2;
  cudaStreamCreate(&s2);
  {
    void *p;
    auto t = std::chrono::steady_clock::now();
    cudaMallocFromPoolAsync(&p, 1024ull << 20, pool, s2);
    printf("%-28s %6d MiB: %.3f ms\n", "other stream", 1024, ms(t));
  }
  printf("err=%s\n", cudaGetErrorString(cudaGetLastError()));
  return 0;
}
