// Random-access DRAM microbenchmark (tools only; not part of the library): the roofline of the
// update kernels, which touch per key a handful of independent random lines (leaf keys / values,
// live count, tombstone mask, head line, out-degree) in arrays far larger than L2.
//   read G:  one aligned G-byte access per op (G/16 x 16-B loads by one thread), 4 ops in flight
//   rmw  :   one atomicAdd (returning) u32 at a random index
//   red  :   one atomicAdd (no return) u32 at a random index
// over an array of S bytes (>> 126 MB L2 unless stated), ops = 2^24 .. 2^26.  Prints ops/s and
// the bytes moved at the access granularity (G, or 32 B for atomics).
// nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o rand_bw rand_bw.cu
#include <cuda_runtime.h>
#include <stdint.h>
#include <stdio.h>
#include <stdlib.h>

__device__ __forceinline__ uint64_t mix(uint64_t z) {
  z += 0x9E3779B97F4A7C15ull;
  z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
  z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
  return z ^ (z >> 31);
}

template <int M>
__device__ __forceinline__ uint4 ld16(const uint4 *p) {
  if (M == 0) return __ldg(p);                 // ld.global.nc (read-only / texture path)
  if (M == 1) return __ldcg(p);                // ld.global.cg (L2 only)
  if (M == 2) return __ldcs(p);                // ld.global.cs (streaming)
  uint4 v;                                     // ld.global (weak, L1-cached)
  asm volatile("ld.global.v4.u32 {%0,%1,%2,%3}, [%4];" : "=r"(v.x), "=r"(v.y), "=r"(v.z), "=r"(v.w) : "l"(p));
  return v;
}

template <int G, int R, int M = 0>
__global__ void __launch_bounds__(256) k_read(const uint4 *__restrict__ a, uint64_t nlines, uint64_t nops,
                                              uint64_t seed, uint4 *sink) {
  constexpr int W = G / 16;
  uint4 acc = make_uint4(0, 0, 0, 0);
  const uint64_t nthr = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i0 < nops; i0 += nthr * R) {
    uint4 v[R][W];
#pragma unroll
    for (int q = 0; q < R; ++q) {
      const uint64_t i = i0 + q * nthr;
      const uint64_t line = mix(i ^ seed) & (nlines - 1);   // (sizes are powers of two)
#pragma unroll
      for (int w = 0; w < W; ++w) v[q][w] = i < nops ? ld16<M>(a + line * W + w) : make_uint4(0, 0, 0, 0);
    }
#pragma unroll
    for (int q = 0; q < R; ++q)
#pragma unroll
      for (int w = 0; w < W; ++w) {
        acc.x ^= v[q][w].x; acc.y ^= v[q][w].y; acc.z ^= v[q][w].z; acc.w ^= v[q][w].w;
      }
  }
  if ((acc.x ^ acc.y ^ acc.z ^ acc.w) == 0x12345678u) sink[0] = acc;
}

template <bool RET>
__global__ void __launch_bounds__(256) k_atomic(uint32_t *a, uint64_t n, uint64_t nops, uint64_t seed, uint32_t *sink) {
  uint32_t acc = 0;
  const uint64_t nthr = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < nops; i += nthr) {
    const uint64_t j = mix(i ^ seed) & (n - 1);
    if (RET) acc += atomicAdd(a + j, 1u);
    else atomicAdd(a + j, 1u);
  }
  if (RET && acc == 0x12345678u) sink[0] = acc;
}

// read-modify-write of a random aligned G-byte line (the leaf rewrite of the insert kernel)
template <int G, int R>
__global__ void __launch_bounds__(256) k_line_rmw(uint4 *a, uint64_t nlines, uint64_t nops, uint64_t seed) {
  constexpr int W = G / 16;
  const uint64_t nthr = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i0 < nops; i0 += nthr * R) {
    uint64_t line[R];
    uint4 v[R][W];
#pragma unroll
    for (int q = 0; q < R; ++q) {
      line[q] = mix((i0 + q * nthr) ^ seed) & (nlines - 1);
#pragma unroll
      for (int w = 0; w < W; ++w) v[q][w] = i0 + q * nthr < nops ? a[line[q] * W + w] : make_uint4(0, 0, 0, 0);
    }
#pragma unroll
    for (int q = 0; q < R; ++q)
      if (i0 + q * nthr < nops)
#pragma unroll
        for (int w = 0; w < W; ++w) { v[q][w].x += 1; a[line[q] * W + w] = v[q][w]; }
  }
}

__global__ void k_copy(const uint4 *__restrict__ a, uint4 *__restrict__ b, uint64_t n) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n; i += (uint64_t)gridDim.x * blockDim.x)
    b[i] = a[i];
}

static int nsm() {
  int d, s;
  cudaGetDevice(&d);
  cudaDeviceGetAttribute(&s, cudaDevAttrMultiProcessorCount, d);
  return s;
}

template <class F>
static float timeit(F f) {
  cudaEvent_t a, b;
  cudaEventCreate(&a);
  cudaEventCreate(&b);
  f();                                    // warm-up
  float best = 1e30f;
  for (int r = 0; r < 5; ++r) {
    cudaEventRecord(a);
    f();
    cudaEventRecord(b);
    cudaEventSynchronize(b);
    float ms;
    cudaEventElapsedTime(&ms, a, b);
    best = ms < best ? ms : best;
  }
  return best;
}

template <int G, int R = 4, int M = 0>
static void read_case(const uint4 *a, uint64_t bytes, uint64_t nops, uint4 *sink, int blocks) {
  const uint64_t nl = bytes / G;
  const float ms = timeit([&] { k_read<G, R, M><<<blocks, 256>>>(a, nl, nops, 7, sink); });
  printf("{\"kind\": \"read\", \"ldmode\": %d, \"ilp\": %d, \"granule_B\": %d, \"array_MB\": %llu, \"ops\": %llu, \"ms\": %.4f, \"Gops_s\": %.3f, "
         "\"GB_s_at_granule\": %.1f}\n",
         M, R, G, (unsigned long long)(bytes >> 20), (unsigned long long)nops, ms, nops / ms / 1e6, nops * (double)G / ms / 1e6);
}

template <bool RET>
static void atomic_case(uint32_t *a, uint64_t bytes, uint64_t nops, uint32_t *sink, int blocks) {
  const float ms = timeit([&] { k_atomic<RET><<<blocks, 256>>>(a, bytes / 4, nops, 11, sink); });
  printf("{\"kind\": \"%s\", \"granule_B\": 32, \"array_MB\": %llu, \"ops\": %llu, \"ms\": %.4f, \"Gops_s\": %.3f, "
         "\"GB_s_at_granule\": %.1f}\n",
         RET ? "atomic_rmw" : "red", (unsigned long long)(bytes >> 20), (unsigned long long)nops, ms, nops / ms / 1e6,
         nops * 32.0 / ms / 1e6);
}

int main() {
  const uint64_t big = 4ull << 30;                       // 4 GiB >> L2
  uint4 *a, *b, *sink;
  cudaMalloc(&a, big);
  cudaMalloc(&b, big);
  cudaMalloc(&sink, 64);
  cudaMemset(a, 1, big);
  const int blocks = nsm() * 8;
  const float cms = timeit([&] { k_copy<<<blocks, 256>>>(a, b, big / 16); });
  printf("{\"kind\": \"copy\", \"array_MB\": %llu, \"ms\": %.4f, \"GB_s\": %.1f}\n", (unsigned long long)(big >> 20), cms,
         2.0 * big / cms / 1e6);
  const uint64_t nops = 1ull << 25;
  if (getenv("RB_LDMODES")) {                  // load-instruction variants of random 32/64-B reads
    read_case<32, 4, 0>(a, big, nops, sink, blocks);
    read_case<32, 4, 1>(a, big, nops, sink, blocks);
    read_case<32, 4, 2>(a, big, nops, sink, blocks);
    read_case<32, 4, 3>(a, big, nops, sink, blocks);
    read_case<64, 4, 0>(a, big, nops, sink, blocks);
    read_case<64, 4, 1>(a, big, nops, sink, blocks);
    read_case<16, 4, 0>(a, big, nops, sink, blocks);
    read_case<16, 4, 1>(a, big, nops, sink, blocks);
    cudaError_t e = cudaDeviceSynchronize();
    return e ? 1 : 0;
  }
  for (uint64_t mb : {64ull, 128ull, 256ull, 2048ull, 4096ull}) {
    read_case<16>(a, mb << 20, nops, sink, blocks);
    read_case<32>(a, mb << 20, nops, sink, blocks);
    read_case<64>(a, mb << 20, nops, sink, blocks);
    read_case<128>(a, mb << 20, nops, sink, blocks);
  }
  read_case<32, 8>(a, big, nops, sink, blocks);
  read_case<64, 8>(a, big, nops, sink, blocks);
  read_case<128, 8>(a, big, nops, sink, blocks);
  // the L2 fetch granularity limit (a hint): does a random sector miss fetch 32, 64 or 128 B?
  for (int gr : {32, 64, 128}) {
    size_t before = 0, after = 0;
    cudaDeviceGetLimit(&before, cudaLimitMaxL2FetchGranularity);
    cudaDeviceSetLimit(cudaLimitMaxL2FetchGranularity, gr);
    cudaDeviceGetLimit(&after, cudaLimitMaxL2FetchGranularity);
    printf("{\"kind\": \"l2_fetch_granularity\", \"before\": %zu, \"set\": %d, \"after\": %zu}\n", before, gr, after);
    read_case<32>(a, big, nops, sink, blocks);
    read_case<64>(a, big, nops, sink, blocks);
    read_case<16>(a, 128ull << 20, nops, sink, blocks);
    atomic_case<true>((uint32_t *)a, 1024ull << 20, nops, (uint32_t *)sink, blocks);
  }
  cudaDeviceSetLimit(cudaLimitMaxL2FetchGranularity, 128);
  for (uint64_t mb : {1024ull, 2048ull}) {
    const float m64 = timeit([&] { k_line_rmw<64, 4><<<blocks, 256>>>(a, (mb << 20) / 64, nops, 3); });
    const float m128 = timeit([&] { k_line_rmw<128, 4><<<blocks, 256>>>(a, (mb << 20) / 128, nops, 3); });
    printf("{\"kind\": \"line_rmw\", \"granule_B\": 64, \"array_MB\": %llu, \"ops\": %llu, \"ms\": %.4f, \"Gops_s\": %.3f}\n",
           (unsigned long long)mb, (unsigned long long)nops, m64, nops / m64 / 1e6);
    printf("{\"kind\": \"line_rmw\", \"granule_B\": 128, \"array_MB\": %llu, \"ops\": %llu, \"ms\": %.4f, \"Gops_s\": %.3f}\n",
           (unsigned long long)mb, (unsigned long long)nops, m128, nops / m128 / 1e6);
  }
  for (uint64_t mb : {64ull, 128ull, 256ull, 1024ull, 4096ull}) {
    atomic_case<true>((uint32_t *)a, mb << 20, nops, (uint32_t *)sink, blocks);
    atomic_case<false>((uint32_t *)a, mb << 20, nops, (uint32_t *)sink, blocks);
  }
  cudaError_t e = cudaDeviceSynchronize();
  if (e) printf("{\"error\": \"%s\"}\n", cudaGetErrorString(e));
  return e ? 1 : 0;
}
