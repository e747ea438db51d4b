// sweep.cuh -- TMA-fed sweeps over the gapped slot array (sm_100a).
//
// The analytics that read "CSR on GPMA" in place stream the whole key array and
// the per-leaf tombstone masks once per pass, and do random work per live edge (REDs into
// y for PageRank, parent-array probes for CC).  A warp that both loads and issues the random
// traffic serialises the two: while its RED/atomic queue is full it cannot issue its next
// loads.  Here the stream is decoupled from the per-edge work:
//
//   * one producer warp per CTA: one elected lane issues 1-D bulk copies (cp.async.bulk,
//     TMA engine) of a tile of T slots -- keys (8 B/slot) + the tile's tombstone-mask words
//     + an operation-specific side slice (e.g. the tile's PageRank contributions) -- into a
//     ring of S shared-memory stages, each completed by an mbarrier transaction count;
//   * NC consumer warps wait on a stage's "full" barrier, visit their T/NC slots from shared
//     memory and release the stage on its "empty" barrier (one arrive per warp).
//
// The CTA is persistent (one per SM) and owns a contiguous run of tiles, so the side slices
// of consecutive tiles are adjacent.  T is a multiple of L (tiles are leaf aligned).
#pragma once

#include <cuda_runtime.h>
#include <stdint.h>

namespace gp {
namespace tma {

__device__ __forceinline__ uint32_t smem_u32(const void *p) {
  return (uint32_t)__cvta_generic_to_shared(p);
}

__device__ __forceinline__ void mbar_init(uint64_t *bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}

__device__ __forceinline__ void mbar_fence_init() {
  asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
}

// arrive (count 1) and add `bytes` to the transaction count of the current phase
__device__ __forceinline__ void mbar_arrive_tx(uint64_t *bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes)
               : "memory");
}

__device__ __forceinline__ void mbar_arrive(uint64_t *bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}

// block until the phase with the given parity has completed
__device__ __forceinline__ void mbar_wait(uint64_t *bar, uint32_t parity) {
  const uint32_t a = smem_u32(bar);
  uint32_t done;
  do {
    asm volatile(
        "{\n\t.reg .pred p;\n\t"
        "mbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\t"
        "selp.u32 %0, 1, 0, p;\n\t}"
        : "=r"(done)
        : "r"(a), "r"(parity)
        : "memory");
  } while (!done);
}

// 1-D bulk copy global -> shared, completing `bytes` on `bar` (16-B aligned, bytes % 16 == 0)
__device__ __forceinline__ void bulk_g2s(void *dst, const void *src, uint32_t bytes, uint64_t *bar,
                                         uint64_t pol) {
  asm volatile(
      "cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes.L2::cache_hint [%0], [%1], %2, [%3], %4;" ::"r"(
          smem_u32(dst)),
      "l"(src), "r"(bytes), "r"(smem_u32(bar)), "l"(pol)
      : "memory");
}

__device__ __forceinline__ uint64_t policy_evict_first() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_first.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}

__device__ __forceinline__ uint64_t policy_evict_last() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}

}  // namespace tma

// Shared-memory layout of one stage: keys[T], tmask[T/4] (enough for L >= 4), side bytes.
template <int T, int SIDE>
struct SweepStage {
  uint64_t key[T];
  uint32_t tm[T / 4];
  alignas(16) unsigned char side[SIDE];
};

// Per-tile bounds of the rows met in the tile, from the locate heads (R9): every key of the
// tile lies in [head[s0/L], head[(s0+T)/L]) and every vertex owns a guard slot, so at most
// T+2 consecutive rows meet a tile.  ulo/uhi are local rows (minus rb), clamped to [0, nr).
struct TileRows {
  uint32_t ulo, uhi;   // inclusive
};

__device__ __forceinline__ TileRows tile_rows(uint64_t h_lo, uint64_t h_hi, uint32_t rb, uint32_t nr) {
  TileRows r;
  if (h_lo == ~0ull || nr == 0) {
    r.ulo = r.uhi = 0;
    return r;
  }
  uint32_t lo = (uint32_t)(h_lo >> 32) - rb;
  uint32_t hi = (h_hi == ~0ull) ? nr - 1 : (uint32_t)(h_hi >> 32) - rb;
  if (lo >= nr) lo = nr - 1;
  if (hi >= nr) hi = nr - 1;
  if (hi < lo) hi = lo;
  r.ulo = lo;
  r.uhi = hi;
  return r;
}

// The generic persistent sweep.  Op must provide
//   static constexpr int SIDE;                       side bytes per stage (multiple of 16)
//   __device__ uint32_t side_bytes(uint64_t s0, uint64_t h_lo, uint64_t h_hi, uint32_t *meta) const;
//       producer lane: bytes of the tile's side slice (0 = none) and a word for the consumers
//   __device__ void side_copy(uint64_t s0, uint32_t meta, void *dst, uint32_t bytes, uint64_t *bar) const;
//       producer lane: issue the side copies (completing on bar)
//   template <int G> __device__ void visit_warp(const uint64_t *key, const uint32_t *tm,
//                         const void *side, uint32_t meta, uint64_t s0, uint32_t i0, uint32_t L,
//                         uint32_t lgL, void *ex) const;
//       consumer lane: slots i0 + 32 j (j < G) of the tile starting at slot s0 (batch the
//       shared-memory loads of all G slots before using them: LDS latency is the limit)
//   static constexpr int EXTRA;                      CTA-private shared bytes (ex), may be 0
//   __device__ void init(void *ex) const;  __device__ void finish(void *ex) const;
//       all threads of the CTA, before the first tile / after the last one
// Launch: grid = #SMs (persistent), block = 32 * (NC + 1), dynamic smem = sweep_smem<T,S,Op>().
// Requires a store whose every row has its guard (rows_indexed) for the T+2 row bound.
template <int T, int S, class Op>
constexpr size_t sweep_smem() {
  return sizeof(SweepStage<T, Op::SIDE>) * S + 2 * S * sizeof(uint64_t) + S * sizeof(uint32_t) + 128 +
         ((Op::EXTRA + 15) & ~15);
}

// Body of a sweep kernel; each operation wraps it in its own __global__ (named in profiles)
// with __launch_bounds__(32 * (NC + 1), 1).
template <int T, int S, int NC, class Op>
__device__ __forceinline__ void sweep_run(const uint64_t *__restrict__ key, const uint32_t *__restrict__ tmask,
                                          const uint64_t *__restrict__ head, uint64_t cap, uint32_t L,
                                          uint32_t lgL, const Op &op) {
  static_assert(T % (32 * NC) == 0, "consumer warps split a tile in 32-slot groups");
  using Stage = SweepStage<T, Op::SIDE>;
  extern __shared__ __align__(128) unsigned char smem_raw[];
  // align by pointer arithmetic (an integer round trip would hide the shared address space)
  unsigned char *base = smem_raw + ((128u - (tma::smem_u32(smem_raw) & 127u)) & 127u);
  Stage *st = reinterpret_cast<Stage *>(base);
  uint64_t *full = reinterpret_cast<uint64_t *>(base + sizeof(Stage) * S);
  uint64_t *empty = full + S;
  uint32_t *meta = reinterpret_cast<uint32_t *>(empty + S);
  void *ex = reinterpret_cast<unsigned char *>(meta) + ((S * sizeof(uint32_t) + 15) & ~(size_t)15);

  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  if (threadIdx.x == 0) {
    for (int i = 0; i < S; ++i) {
      tma::mbar_init(&full[i], 1);
      tma::mbar_init(&empty[i], NC);
    }
    tma::mbar_fence_init();
  }
  op.init(ex);
  __syncthreads();

  const uint64_t ntiles = cap / T;
  const uint64_t t0 = blockIdx.x * ntiles / gridDim.x, t1 = (blockIdx.x + 1) * ntiles / gridDim.x;
  const uint64_t n = t1 - t0;
  const uint32_t lpt = T >> lgL;                     // leaves per tile

  if (warp == 0) {
    // ---------------- producer: heads of 32 tiles per batch (lane j -> tile b + j), the
    // batch after next prefetched so the dependent head loads never stall the ring
    const uint64_t pol = tma::policy_evict_first();
    auto head_at = [&](uint64_t t) -> uint64_t {      // head of the first leaf of tile t
      return t < ntiles ? __ldg(head + t * lpt) : ~0ull;
    };
    uint64_t hcur = head_at(t0 + lane), hnext = head_at(t0 + 32 + lane);
    for (uint64_t b = 0; b < n; b += 32) {
      const uint64_t hfar = head_at(t0 + b + 64 + lane);
      const uint64_t hcur32 = __shfl_sync(0xffffffffu, hnext, 0);   // head of tile b+32
      for (uint32_t j = 0; j < 32 && b + j < n; ++j) {
        const uint64_t i = b + j;
        const uint64_t h_lo = __shfl_sync(0xffffffffu, hcur, j);
        const uint64_t h_hi = j < 31 ? __shfl_sync(0xffffffffu, hcur, j + 1) : hcur32;
        if (lane == 0) {
          const uint32_t s = (uint32_t)(i % S);
          if (i >= S) tma::mbar_wait(&empty[s], (uint32_t)((i / S) & 1) ^ 1u);
          const uint64_t s0 = (t0 + i) * T;
          uint32_t m = 0;
          // expected bytes first (the copies may complete before the arrive otherwise)
          const uint32_t kb = T * 8, tb = (lpt * 4 + 15) & ~15u;
          uint32_t sb = op.side_bytes(s0, h_lo, h_hi, &m);
          meta[s] = m;
          tma::mbar_arrive_tx(&full[s], kb + tb + sb);
          tma::bulk_g2s(st[s].key, key + s0, kb, &full[s], pol);
          tma::bulk_g2s(st[s].tm, tmask + (s0 >> lgL), tb, &full[s], pol);
          if (sb) op.side_copy(s0, m, st[s].side, sb, &full[s]);
        }
      }
      hcur = hnext;
      hnext = hfar;
    }
  } else {
    // ---------------- consumers
    const uint32_t cw = warp - 1;
    constexpr uint32_t PER = T / NC;
    for (uint64_t i = 0; i < n; ++i) {
      const uint32_t s = (uint32_t)(i % S);
      tma::mbar_wait(&full[s], (uint32_t)((i / S) & 1));
      const uint64_t s0 = (t0 + i) * T;
      const uint32_t m = meta[s];
      op.template visit_warp<PER / 32>(st[s].key, st[s].tm, st[s].side, m, s0, cw * PER + lane, L, lgL, ex);
      __syncwarp();
      if (lane == 0) tma::mbar_arrive(&empty[s]);
    }
  }
  __syncthreads();
  op.finish(ex);
}

}  // namespace gp
