// dist.cu -- routing for the source-range sharded store (R24).
//
// owner(u) = floor(u / ceil(V / P)).  A batch slice is partitioned by owner with one stable
// counting pass (the radix kernels with a divide-by-chunk digit), so the per-owner pieces keep
// the slice's order and the rank-order concatenation at the owner keeps the global batch
// order (last occurrence wins, R10).  The exchange itself is a collective of the caller's
// communicator (NCCL all-to-all through torch.distributed).
#include <cuda_runtime.h>

#include <algorithm>

#include "gpma_internal.cuh"

namespace gp {

gpma_status route(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, uint32_t nranks,
                  uint64_t *out_keys, uint32_t *out_vals, uint64_t *counts_host, cudaStream_t s) {
  if (nranks == 0 || nranks > 256) return GPMA_ERR_INVALID_ARG;
  const uint32_t div = (uint32_t)(((uint64_t)g->V + nranks - 1) / nranks);
  if (n == 0) {
    for (uint32_t r = 0; r < nranks; ++r) counts_host[r] = 0;
    return GPMA_OK;
  }
  GP_CHECK(g, ensure(g, g->b_stage[2], n * 8, s));
  GP_CHECK(g, ensure(g, g->b_stage[3], ((n * 4 + 7) & ~7ull) + 8 * (nranks + 1), s));   // vals, then starts (8-B aligned)
  uint64_t *k0 = (uint64_t *)g->b_stage[2].p;
  uint32_t *v0 = (uint32_t *)g->b_stage[3].p;
  uint64_t *starts = (uint64_t *)((char *)g->b_stage[3].p + ((n * 4 + 7) & ~7ull));
  GP_CHECK(g, stage_in(g, k0, keys, n * 8, s));
  if (vals) GP_CHECK(g, stage_in(g, v0, vals, n * 4, s));
  else GP_CHECK(g, fill_zero(g, v0, n * 4, s));
  gpma_status st = radix_partition_owner(g, k0, v0, out_keys, out_vals, n, div, nranks, starts, s);
  if (st) return st;
  std::vector<uint64_t> h(nranks + 1);
  GP_CHECK(g, cudaMemcpyAsync(h.data(), starts, 8 * (nranks + 1), cudaMemcpyDeviceToHost, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  for (uint32_t r = 0; r < nranks; ++r) counts_host[r] = h[r + 1] - h[r];
  return GPMA_OK;
}

}  // namespace gp
