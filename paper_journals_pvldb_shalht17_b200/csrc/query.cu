// query.cu -- the dynamic query buffer (§3):
// batches of ad-hoc queries answered on the live store.
//   * edge lookup: locate + leaf scan per key (the update path's pre-pass, read-only);
//   * neighbourhoods: the live out-edges of a batch of vertices, as a CSR (row sizes from the
//     maintained out-degrees, one warp per row compacting its gapped slots);
//   * reachability between pairs (s_i, t_i) -- "queries to check the dynamic reachability
//     between pairs of vertices": a multi-source BFS that carries one bit per
//     query in a 64-bit mask per vertex (up to 64 queries per sweep), edge-centric sweeps
//     over the gapped CSR until every target is resolved or the frontiers die out.
#include <cuda_runtime.h>

#include <algorithm>

#include "gpma_internal.cuh"

namespace gp {

constexpr int TQ = 256;

__device__ __forceinline__ uint32_t q_locate(const uint64_t *__restrict__ head, uint32_t nleaves, uint64_t k) {
  uint32_t lo = 0, hi = nleaves;
  while (lo < hi) {
    uint32_t mid = (lo + hi) >> 1;
    if (__ldg(head + mid) <= k) lo = mid + 1;
    else hi = mid;
  }
  return lo ? lo - 1 : 0;
}

__global__ void k_query_edges(const uint64_t *__restrict__ q, uint64_t n, const uint64_t *__restrict__ key,
                              const uint32_t *__restrict__ val, const uint64_t *__restrict__ head, uint32_t nleaves,
                              uint32_t L, uint32_t *__restrict__ out_val, uint8_t *__restrict__ found) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    const uint64_t k = q[i];
    const uint32_t t = q_locate(head, nleaves, k);
    uint32_t v = VAL_TOMB;
    uint8_t f = 0;
    for (uint32_t p = 0; p < L; ++p) {
      const uint64_t x = key[(uint64_t)t * L + p];
      if (x == k) {
        v = val[(uint64_t)t * L + p];
        f = v != VAL_TOMB;
        break;
      }
      if (x == KEY_NONE || x > k) break;
    }
    if (out_val) out_val[i] = f ? v : VAL_TOMB;
    if (found) found[i] = f;
  }
}

// row sizes of the queried vertices (0 for rows outside the shard)
__global__ void k_query_rowsizes(const uint32_t *__restrict__ verts, uint64_t n, const uint32_t *__restrict__ deg,
                                 uint32_t rb, uint32_t nr, uint64_t *__restrict__ sz) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t u = verts[i] - rb;
    sz[i] = u < nr ? deg[u] : 0;
  }
}

// one warp per queried row: compact its live edges (ballot ranks) into col/val
__global__ void k_query_rows(const uint32_t *__restrict__ verts, uint64_t n, const uint64_t *__restrict__ row_offset,
                             const uint64_t *__restrict__ key, const uint32_t *__restrict__ val,
                             const uint32_t *__restrict__ tmask, uint32_t L, uint32_t rb, uint32_t nr,
                             const uint64_t *__restrict__ rp, uint32_t *__restrict__ col, uint32_t *__restrict__ cval) {
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint64_t warps = (uint64_t)gridDim.x * (blockDim.x / 32);
  for (uint64_t i = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32; i < n; i += warps) {
    const uint32_t u = verts[i] - rb;
    if (u >= nr) continue;
    const uint64_t a = row_offset[u], b = row_offset[u + 1];
    uint64_t out = rp[i];
    for (uint64_t s0 = a; s0 < b; s0 += 32) {
      const uint64_t s = s0 + lane;
      bool e = false;
      uint64_t k = KEY_NONE;
      if (s < b) {
        k = key[s];
        e = k != KEY_NONE && (uint32_t)k != COL_GUARD && !((tmask[leaf_div(s, L)] >> leaf_mod(s, L)) & 1u);
      }
      const uint32_t bal = __ballot_sync(0xffffffffu, e);
      if (e) {
        const uint64_t d = out + __popc(bal & lt);
        col[d] = (uint32_t)k;
        if (cval) cval[d] = val[s];
      }
      out += __popc(bal);
    }
  }
}

// ---- multi-source BFS reachability (64 queries per sweep)
__global__ void k_msbfs_init(const uint32_t *__restrict__ src, uint32_t nq, unsigned long long *seen,
                             unsigned long long *front) {
  for (uint32_t i = threadIdx.x; i < nq; i += blockDim.x) {
    atomicOr(seen + src[i], 1ull << i);
    atomicOr(front + src[i], 1ull << i);
  }
}

// next[v] |= front[u] & ~seen[v] over the live edges u -> v (4 slots per thread)
__global__ void __launch_bounds__(TQ) k_msbfs_sweep(const uint64_t *__restrict__ key, const uint32_t *__restrict__ tmask,
                                                    uint32_t L, uint64_t cap, const unsigned long long *__restrict__ front,
                                                    const unsigned long long *__restrict__ seen, unsigned long long *next) {
  const uint64_t n4 = cap / 4;
  for (uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; t < n4;
       t += (uint64_t)gridDim.x * blockDim.x) {
    const uint64_t s4 = t * 4;
    const ulonglong2 ka = __ldcs(reinterpret_cast<const ulonglong2 *>(key + s4));
    const ulonglong2 kb = __ldcs(reinterpret_cast<const ulonglong2 *>(key + s4 + 2));
    const uint64_t k[4] = {ka.x, ka.y, kb.x, kb.y};
    const uint32_t tb = (__ldg(tmask + leaf_div(s4, L)) >> leaf_mod(s4, L)) & 0xFu;
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      if (k[j] == KEY_NONE || (uint32_t)k[j] == COL_GUARD || ((tb >> j) & 1u)) continue;
      const unsigned long long f = __ldg(front + (k[j] >> 32));
      if (!f) continue;
      const unsigned long long nv = f & ~__ldcg(seen + (uint32_t)k[j]);
      if (nv) atomicOr(next + (uint32_t)k[j], nv);
    }
  }
}

// seen |= next; front = next; next = 0; *alive |= any front bit still open
__global__ void k_msbfs_advance(unsigned long long *seen, unsigned long long *front, unsigned long long *next,
                                uint32_t V, unsigned long long *alive) {
  unsigned long long any = 0;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x) {
    const unsigned long long nx = next[v];
    front[v] = nx;
    if (nx) {
      seen[v] |= nx;
      next[v] = 0;
      any |= nx;
    }
  }
  for (int o = 16; o; o >>= 1) any |= __shfl_xor_sync(0xffffffffu, any, o);
  if ((threadIdx.x & 31) == 0 && any) atomicOr(alive, any);
}

__global__ void k_msbfs_answer(const uint32_t *__restrict__ dst, uint32_t nq, const unsigned long long *__restrict__ seen,
                               uint8_t *__restrict__ out, unsigned long long *resolved) {
  for (uint32_t i = threadIdx.x; i < nq; i += blockDim.x) {
    const uint8_t r = (seen[dst[i]] >> i) & 1ull;
    out[i] = r;
    if (r) atomicOr(resolved, 1ull << i);
  }
}

gpma_status query_edges(gpma *g, const uint64_t *keys, uint64_t n, uint32_t *vals, uint8_t *found, cudaStream_t s) {
  Scratch &X = g->an[AN_QUERY];
  ScanScope scan_scope_(X.scan);
  if (!n) return GPMA_OK;
  GP_CHECK(g, ensure(g, X.stage[0], n * 8, s));
  uint64_t *q = (uint64_t *)X.stage[0].p;
  GP_CHECK(g, stage_in(g, q, keys, n * 8, s));
  GP_LAUNCH(g, k_query_edges, grid_for(n), TQ, 0, s, q, n, g->key, g->val, g->head, (uint32_t)(g->cap / g->L),
            g->L, vals, found);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status query_neighbors(gpma *g, const uint32_t *verts, uint64_t n, uint64_t *row_ptr, uint32_t *col,
                            uint32_t *val, uint64_t cap_nnz, uint64_t *nnz_out, cudaStream_t s) {
  Scratch &X = g->an[AN_QUERY];
  ScanScope scan_scope_(X.scan);
  GP_CHECK(g, ensure(g, X.stage[1], (n + 1) * 4, s));
  GP_CHECK(g, ensure(g, X.lpre, (n + 1) * 8, s));
  uint32_t *vq = (uint32_t *)X.stage[1].p;
  uint64_t *rp = (uint64_t *)X.lpre.p;
  if (n) GP_CHECK(g, stage_in(g, vq, verts, n * 4, s));
  if (n) GP_LAUNCH(g, k_query_rowsizes, grid_for(n), TQ, 0, s, vq, n, g->deg, g->rb, g->nr, rp);
  GP_CHECK(g, scan_u64(g, rp, rp, n, s));
  GP_CHECK(g, readback(g, &X.ctrl_h->sum, rp + n, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  const uint64_t nnz = n ? X.ctrl_h->sum : 0;
  if (nnz_out) *nnz_out = nnz;
  if (!col) return GPMA_OK;
  if (cap_nnz < nnz) {
    set_err(g, "query_neighbors: nnz_capacity too small");
    return GPMA_ERR_INVALID_ARG;
  }
  if (row_ptr) GP_CHECK(g, cudaMemcpyAsync(row_ptr, rp, (n + 1) * 8, cudaMemcpyDeviceToDevice, s));
  if (n)
    GP_LAUNCH(g, k_query_rows, grid_for(n * 32), TQ, 0, s, vq, n, g->row_offset, g->key, g->val, tmask_of(g), g->L,
              g->rb, g->nr, rp, col, val);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status query_reachable(gpma *g, const uint32_t *src, const uint32_t *dst, uint64_t n, uint8_t *out,
                            cudaStream_t s) {
  Scratch &X = g->an[AN_QUERY];
  ScanScope scan_scope_(X.scan);
  const uint64_t V = g->V;
  GP_CHECK(g, ensure(g, X.b[0], V * 8, s));
  GP_CHECK(g, ensure(g, X.b[1], V * 8, s));
  GP_CHECK(g, ensure(g, X.b[2], V * 8, s));
  GP_CHECK(g, ensure(g, X.stage[1], 2 * 64 * 4 + 16, s));
  unsigned long long *seen = (unsigned long long *)X.b[0].p, *front = (unsigned long long *)X.b[1].p,
                     *next = (unsigned long long *)X.b[2].p;
  uint32_t *qs = (uint32_t *)X.stage[1].p, *qd = qs + 64;
  unsigned long long *flags = (unsigned long long *)(qd + 64);   // [0] alive, [1] resolved
  for (uint64_t b0 = 0; b0 < n; b0 += 64) {
    const uint32_t nq = (uint32_t)std::min<uint64_t>(64, n - b0);
    GP_CHECK(g, stage_in(g, qs, src + b0, nq * 4, s));
    GP_CHECK(g, stage_in(g, qd, dst + b0, nq * 4, s));
    GP_CHECK(g, fill_zero(g, seen, V * 8, s));
    GP_CHECK(g, fill_zero(g, front, V * 8, s));
    GP_CHECK(g, fill_zero(g, next, V * 8, s));
    GP_LAUNCH(g, k_msbfs_init, 1, 64, 0, s, qs, nq, seen, front);
    const unsigned long long all = nq == 64 ? ~0ull : ((1ull << nq) - 1);
    for (;;) {
      GP_CHECK(g, fill_zero(g, flags, 16, s));
      GP_LAUNCH(g, k_msbfs_answer, 1, 64, 0, s, qd, nq, seen, out + b0, flags + 1);
      GP_LAUNCH(g, k_msbfs_sweep, grid_for(g->cap / 4), TQ, 0, s, g->key, tmask_of(g), g->L, g->cap, front, seen,
                next);
      GP_LAUNCH(g, k_msbfs_advance, grid_for(V), TQ, 0, s, seen, front, next, (uint32_t)V, flags);
      unsigned long long h[2];
      GP_CHECK(g, cudaMemcpyAsync(h, flags, 16, cudaMemcpyDeviceToHost, s));
      GP_CHECK(g, cudaStreamSynchronize(s));
      // stop when no frontier bit is alive, or every query is already resolved
      if (!(h[0] & all) || (h[1] & all) == all) break;
    }
    GP_LAUNCH(g, k_msbfs_answer, 1, 64, 0, s, qd, nq, seen, out + b0, flags + 1);
  }
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

}  // namespace gp
