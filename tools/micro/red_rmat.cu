// Random-RED throughput with RMAT-skewed vs uniform destinations (tools only; not part of the
// library).  V = 2^24 u64 targets (128 MB) or the lower half (64 MB); 134M REDs.
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>
__device__ __forceinline__ uint64_t mix(uint64_t z) {
  z += 0x9E3779B97F4A7C15ull; z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull; return z ^ (z >> 31);
}
__device__ __forceinline__ uint32_t rmat_dst(uint64_t i, int scale) {
  uint32_t d = 0;
  for (int l = 0; l < scale; l += 4) {
    uint64_t w = mix(i * 8 + l);
    for (int k = 0; k < 4 && l + k < scale; ++k) {
      uint32_t r = (uint32_t)(w >> (16 * k)) & 0xFFFF;
      d = (d << 1) | (r >= 49807u);          // P(bit = 1) = 0.24 (b + d quadrants)
    }
  }
  return (d * 0x9E3779B1u) & ((1u << scale) - 1);   // odd multiplier: a bijection (scramble)
}
// mode 0 uniform, 1 rmat; half: keep only dst < V/2 (others skipped)
__global__ void k_red(unsigned long long *y, uint64_t n_ops, int scale, int mode, int half, int agg) {
  const uint32_t V = 1u << scale;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n_ops; i += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t d = mode ? rmat_dst(i, scale) : (uint32_t)(mix(i) & (V - 1));
    if (half && d >= V / 2) continue;
    if (agg) {
      unsigned m = __match_any_sync(__activemask(), d);
      unsigned long long s = __popc(m);
      if ((__ffs(m) - 1) == (int)(threadIdx.x & 31)) atomicAdd(&y[d], s);
    } else atomicAdd(&y[d], 1ull);
  }
}
__global__ void k_gen(uint32_t *dst, uint64_t n_ops, int scale, int mode) {
  const uint32_t V = 1u << scale;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n_ops; i += (uint64_t)gridDim.x * blockDim.x)
    dst[i] = mode ? rmat_dst(i, scale) : (uint32_t)(mix(i) & (V - 1));
}
__global__ void k_red_buf(unsigned long long *y, const uint32_t *dst, uint64_t n_ops, uint32_t lim) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n_ops; i += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t d = __ldcs(dst + i);
    if (d < lim) atomicAdd(&y[d], 1ull);
  }
}
__global__ void k_gen_only(unsigned long long *y, uint64_t n_ops, int scale, int mode) {
  const uint32_t V = 1u << scale;
  uint32_t acc = 0;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n_ops; i += (uint64_t)gridDim.x * blockDim.x)
    acc ^= mode ? rmat_dst(i, scale) : (uint32_t)(mix(i) & (V - 1));
  if (acc == 0x12345678) y[0] = acc;
}
// REDs with the destinations in a hot bitmap skipped (what a shared-memory aggregation of the
// hot destinations would leave to L2): measures the same-address serialisation on hot lines
__global__ void k_red_buf_skip(unsigned long long *y, const uint32_t *dst, uint64_t n_ops, const uint32_t *hot) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n_ops; i += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t d = __ldcs(dst + i);
    if ((__ldg(hot + (d >> 5)) >> (d & 31)) & 1u) continue;
    atomicAdd(&y[d], 1ull);
  }
}
__global__ void k_mark_hot(const unsigned long long *cnt, uint32_t V, unsigned long long thr, uint32_t *hot) {
  for (uint32_t v = blockIdx.x * blockDim.x + threadIdx.x; v < V; v += gridDim.x * blockDim.x)
    if (cnt[v] >= thr) atomicOr(hot + (v >> 5), 1u << (v & 31));
}
int main() {
  const uint64_t ops = 134217728;
  const int scale = 24;
  unsigned long long *y;
  cudaMalloc(&y, (8ull << scale));
  cudaMemset(y, 0, 8ull << scale);
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  for (int mode = 0; mode < 2; ++mode) {
    float ms;
    k_gen_only<<<148 * 8, 256>>>(y, ops, scale, mode);
    cudaEventRecord(a);
    k_gen_only<<<148 * 8, 256>>>(y, ops, scale, mode);
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    cudaEventElapsedTime(&ms, a, b);
    printf("%s gen only: %.3f ms\n", mode ? "rmat" : "unif", ms);
    for (int half = 0; half < 2; ++half)
      for (int agg = 0; agg < 2; ++agg) {
        k_red<<<148 * 8, 256>>>(y, ops, scale, mode, half, agg);
        cudaEventRecord(a);
        k_red<<<148 * 8, 256>>>(y, ops, scale, mode, half, agg);
        cudaEventRecord(b);
        cudaEventSynchronize(b);
        cudaEventElapsedTime(&ms, a, b);
        printf("%s half=%d agg=%d: %.3f ms\n", mode ? "rmat" : "unif", half, agg, ms);
      }
  }
  uint32_t *dst;
  cudaMalloc(&dst, ops * 4);
  for (int mode = 0; mode < 2; ++mode) {
    k_gen<<<148 * 8, 256>>>(dst, ops, scale, mode);
    for (uint32_t lim : {1u << 24, 1u << 23, 1u << 22, 0u}) {
      float ms;
      k_red_buf<<<148 * 8, 256>>>(y, dst, ops, lim);
      cudaEventRecord(a);
      k_red_buf<<<148 * 8, 256>>>(y, dst, ops, lim);
      cudaEventRecord(b);
      cudaEventSynchronize(b);
      cudaEventElapsedTime(&ms, a, b);
      printf("buf %s dst<%u: %.3f ms\n", mode ? "rmat" : "unif", lim, ms);
    }
  }
  // share of RMAT REDs to the most frequent destinations
  {
    unsigned long long *h = (unsigned long long *)malloc(8ull << scale);
    cudaMemset(y, 0, 8ull << scale);
    k_red_buf<<<148 * 8, 256>>>(y, dst, ops, 1u << 24);
    cudaMemcpy(h, y, 8ull << scale, cudaMemcpyDeviceToHost);
    // counting sort of counts
    static unsigned long long hist[1 << 22];
    unsigned long long mx = 0;
    for (uint32_t v = 0; v < (1u << scale); ++v) { unsigned long long c = h[v]; if (c >= (1u << 22)) c = (1u << 22) - 1; hist[c]++; if (h[v] > mx) mx = h[v]; }
    unsigned long long top = 0, acc = 0;
    printf("max count %llu\n", mx);
    unsigned long long marks[] = {1, 16, 256, 1024, 4096, 16384, 65536, 262144, 1048576};
    int mi = 0;
    for (int64_t c = (1 << 22) - 1; c >= 0 && mi < 9; --c) {
      for (unsigned long long k = 0; k < hist[c] && mi < 9; ++k) {
        ++top; acc += c;
        if (top == marks[mi]) { printf("top %llu vertices: %.1f%% of REDs (min count %lld)\n", top, 100.0 * acc / ops, (long long)c); ++mi; }
      }
    }
  }
  {
    unsigned long long *cnt;
    cudaMalloc(&cnt, 8ull << scale);
    cudaMemset(cnt, 0, 8ull << scale);
    k_red_buf<<<148 * 8, 256>>>(cnt, dst, ops, 1u << 24);   // rmat dst (last generated mode)
    uint32_t *hot;
    cudaMalloc(&hot, (1u << scale) / 8);
    for (unsigned long long thr : {~0ull, 58449ull, 18328ull, 5853ull, 1882ull, 615ull}) {
      cudaMemset(hot, 0, (1u << scale) / 8);
      k_mark_hot<<<148 * 8, 256>>>(cnt, 1u << scale, thr, hot);
      float ms;
      k_red_buf_skip<<<148 * 8, 256>>>(y, dst, ops, hot);
      cudaEventRecord(a);
      k_red_buf_skip<<<148 * 8, 256>>>(y, dst, ops, hot);
      cudaEventRecord(b);
      cudaEventSynchronize(b);
      cudaEventElapsedTime(&ms, a, b);
      printf("rmat REDs, destinations with count >= %llu skipped: %.3f ms\n", thr, ms);
    }
  }
  return 0;
}
