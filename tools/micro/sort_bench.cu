// CTA bitonic sort timing (tools only): nvcc -gencode arch=compute_100a,code=sm_100a -O3 -I include
//   -I paper_journals_pvldb_shalht17_b200/csrc tools/micro/sort_bench.cu -o /tmp/sort_bench
#include <cstdio>
#include <cstdint>
#include <vector>
#include <algorithm>
#include "gpma_internal.cuh"

using namespace gp;

template <int MODE>
__global__ void __launch_bounds__(1024) k_sort(uint64_t *in, uint64_t *out, uint32_t n, unsigned long long *cyc) {
  __shared__ uint64_t sk[2048];
  __shared__ uint32_t si[2048];
  uint32_t np2 = 2;
  while (np2 < n) np2 <<= 1;
  const uint32_t np2a = MODE == 2 && np2 < 64 ? 64 : np2;
  for (uint32_t i = threadIdx.x; i < np2a; i += blockDim.x) {
    sk[i] = i < n ? in[i] : ~0ull;
    si[i] = i;
  }
  __syncthreads();
  unsigned long long t0 = clock64();
  if (MODE == 0) cta_bitonic_sort_u64(sk, np2);
  else if (MODE == 1) cta_bitonic_sort(sk, si, np2);
  else cta_merge_sort_u64(sk, np2 < 64 ? 64 : np2);
  unsigned long long t1 = clock64();
  if (threadIdx.x == 0) *cyc = t1 - t0;
  for (uint32_t i = threadIdx.x; i < n; i += blockDim.x) out[i] = sk[i];
}

int main() {
  for (uint32_t n : {1u, 5u, 33u, 64u, 100u, 1000u, 2000u, 2048u}) {
    std::vector<uint64_t> h(n);
    uint64_t x = 88172645463325252ull;
    for (auto &v : h) { x ^= x << 13; x ^= x >> 7; x ^= x << 17; v = x >> 8; }
    uint64_t *d, *o; unsigned long long *c;
    cudaMalloc(&d, n * 8); cudaMalloc(&o, n * 8); cudaMalloc(&c, 8);
    cudaMemcpy(d, h.data(), n * 8, cudaMemcpyHostToDevice);
    for (int mode = 0; mode < 3; ++mode) {
      unsigned long long cy = 0;
      for (int rep = 0; rep < 3; ++rep) {
        if (mode == 0) k_sort<0><<<1, 1024>>>(d, o, n, c); else if (mode == 1) k_sort<1><<<1, 1024>>>(d, o, n, c); else k_sort<2><<<1, 1024>>>(d, o, n, c);
        cudaMemcpy(&cy, c, 8, cudaMemcpyDeviceToHost);
      }
      std::vector<uint64_t> r(n);
      cudaMemcpy(r.data(), o, n * 8, cudaMemcpyDeviceToHost);
      auto s = h; std::sort(s.begin(), s.end());
      printf("n=%u mode=%d cycles=%llu ok=%d err=%s\n", n, mode, cy, (int)(r == s), cudaGetErrorString(cudaGetLastError()));
    }
  }
  return 0;
}
