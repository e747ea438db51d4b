// analytics.cu -- graph analytics that read the gapped CSR in place (sm_100a).
//
// "CSR on GPMA" (Fig. 5): row u occupies slots [row_offset[u], row_offset[u+1]);
// a slot holds an edge iff it is occupied, not a guard and not a tombstone -- the
// IsEntryExist test of Alg. 2 l.10 / Alg. 3 l.4.
//   BFS  (Table 1: Merrill et al. [37]): level-synchronous top-down frontier expansion,
//        one warp per frontier row (Neighbour Gathering, Alg. 3), visited checks by CAS.
//   CC   (Table 1: Soman et al. [43]): edge-centric hooking of roots (larger id under
//        smaller) with CAS + path halving, then full pointer jumping -> min-id labels.
//   PR   (Table 1: CUSP SpMV [2]): push SpMV over the live slots.
//   export: CSR compaction via per-leaf edge counts + scan.
#include <cuda_runtime.h>

#include <algorithm>

#include "gpma_internal.cuh"

namespace gp {

constexpr int TA = 256;

__device__ __forceinline__ bool edge_at(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val,
                                        uint64_t s, uint64_t *k) {
  uint64_t x = key[s];
  *k = x;
  return x != KEY_NONE && (uint32_t)x != COL_GUARD && val[s] != VAL_TOMB;
}

// ------------------------------------------------------------------ BFS
__global__ void k_bfs_init(int32_t *levels, uint32_t V, uint32_t root, uint32_t *frontier) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x)
    levels[v] = (v == root) ? 0 : -1;
  if (blockIdx.x == 0 && threadIdx.x == 0) frontier[0] = root;
}

__global__ void k_bfs_expand(const uint32_t *__restrict__ frontier, uint32_t fsize,
                             const uint64_t *__restrict__ row_offset, const uint64_t *__restrict__ key,
                             const uint32_t *__restrict__ val, int32_t *levels, int32_t depth,
                             uint32_t *__restrict__ next, uint32_t *next_count) {
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint64_t warps = (uint64_t)gridDim.x * (blockDim.x / 32);
  for (uint64_t i = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32; i < fsize; i += warps) {
    uint32_t u = frontier[i];
    uint64_t a = row_offset[u], b = row_offset[u + 1];
    for (uint64_t s0 = a; s0 < b; s0 += 32) {
      uint64_t s = s0 + lane;
      bool disc = false;
      uint32_t v = 0;
      uint64_t k;
      if (s < b && edge_at(key, val, s, &k)) {
        v = (uint32_t)k;
        if (levels[v] == -1) disc = atomicCAS(&levels[v], -1, depth) == -1;
      }
      uint32_t bal = __ballot_sync(0xffffffffu, disc);
      if (bal) {
        uint32_t base = 0;
        if (lane == 0) base = atomicAdd(next_count, __popc(bal));
        base = __shfl_sync(0xffffffffu, base, 0);
        if (disc) next[base + __popc(bal & lt)] = v;
      }
    }
  }
}

gpma_status bfs(gpma *g, uint32_t root, int32_t *levels, cudaStream_t s) {
  GP_CHECK(g, ensure(g->b_misc, ((uint64_t)g->V + 1) * 4, s));
  GP_CHECK(g, ensure(g->b_misc2, ((uint64_t)g->V + 1) * 4, s));
  uint32_t *fa = (uint32_t *)g->b_misc.p, *fb = (uint32_t *)g->b_misc2.p;
  uint32_t *cnt_d = &reinterpret_cast<uint32_t *>(&g->ctrl_d->sum)[0];
  GP_LAUNCH(g, k_bfs_init, grid_for(g->V), TA, 0, s, levels, g->V, root, fa);
  uint32_t fsize = 1;
  int32_t depth = 0;
  while (fsize) {
    ++depth;
    GP_CHECK(g, cudaMemsetAsync(cnt_d, 0, 4, s));
    GP_LAUNCH(g, k_bfs_expand, grid_for((uint64_t)fsize * 32), TA, 0, s, fa, fsize, g->row_offset,
              g->key, g->val, levels, depth, fb, cnt_d);
    GP_CHECK(g, cudaMemcpyAsync(&g->ctrl_h->sum, cnt_d, 4, cudaMemcpyDeviceToHost, s));
    GP_CHECK(g, cudaStreamSynchronize(s));
    fsize = (uint32_t)(g->ctrl_h->sum & 0xFFFFFFFFu);
    std::swap(fa, fb);
  }
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// ------------------------------------------------------------------ CC
__device__ __forceinline__ uint32_t cc_find(uint32_t *p, uint32_t x) {
  // path halving on a forest with parent[x] <= x (roots are the minima)
  volatile uint32_t *vp = p;
  uint32_t cur = vp[x];
  if (cur != x) {
    uint32_t prev = x, next;
    while (cur > (next = vp[cur])) {
      vp[prev] = next;
      prev = cur;
      cur = next;
    }
  }
  return cur;
}

__global__ void k_cc_init(uint32_t *p, uint32_t V) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x)
    p[v] = (uint32_t)v;
}

__global__ void k_cc_hook(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val, uint64_t cap,
                          uint32_t *p) {
  for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < cap;
       s += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t k;
    if (!edge_at(key, val, s, &k)) continue;
    uint32_t u = (uint32_t)(k >> 32), v = (uint32_t)k;
    if (u == v) continue;
    uint32_t ru = cc_find(p, u), rv = cc_find(p, v);
    bool repeat;
    do {
      repeat = false;
      if (ru != rv) {
        uint32_t ret;
        if (ru < rv) {
          if ((ret = atomicCAS(&p[rv], rv, ru)) != rv) { rv = ret; repeat = true; }
        } else {
          if ((ret = atomicCAS(&p[ru], ru, rv)) != ru) { ru = ret; repeat = true; }
        }
      }
    } while (repeat);
  }
}

__global__ void k_cc_final(uint32_t *p, uint32_t *labels, uint32_t V) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x) {
    volatile uint32_t *vp = p;
    uint32_t x = (uint32_t)v, nx;
    while ((nx = vp[x]) != x) x = nx;
    labels[v] = x;
  }
}

gpma_status cc(gpma *g, uint32_t *labels, cudaStream_t s) {
  GP_CHECK(g, ensure(g->b_misc, ((uint64_t)g->V + 1) * 4, s));
  uint32_t *p = (uint32_t *)g->b_misc.p;
  GP_LAUNCH(g, k_cc_init, grid_for(g->V), TA, 0, s, p, g->V);
  GP_LAUNCH(g, k_cc_hook, grid_for(g->cap), TA, 0, s, g->key, g->val, g->cap, p);
  GP_LAUNCH(g, k_cc_final, grid_for(g->V), TA, 0, s, p, labels, g->V);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// ------------------------------------------------------------------ PageRank
// out-degree of each row = live edges in it (warp-aggregated by source)
__global__ void k_pr_outdeg(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val, uint64_t cap,
                            uint32_t *deg) {
  const int lane = threadIdx.x & 31;
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  const uint64_t capr = (cap + 31) & ~31ull;
  for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < capr; s += stride) {
    uint64_t k = 0;
    bool e = s < cap && edge_at(key, val, s, &k);
    uint32_t src = e ? (uint32_t)(k >> 32) : 0xFFFFFFFFu;
    uint32_t peers = __match_any_sync(0xffffffffu, src);
    if (e && (__ffs(peers) - 1) == lane) atomicAdd(&deg[src], (uint32_t)__popc(peers));
  }
}

template <typename T>
__global__ void k_pr_init(T *x, uint32_t V) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x)
    x[v] = T(1) / T(V);
}

template <typename T>
__device__ __forceinline__ double block_sum_d(double v, double *red) {
  for (int o = 16; o; o >>= 1) v += __shfl_xor_sync(0xffffffffu, v, o);
  if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = v;
  __syncthreads();
  double s = 0;
  if (threadIdx.x == 0)
    for (int k = 0; k < (int)(blockDim.x >> 5); ++k) s += red[k];
  __syncthreads();
  return s;
}

// contrib[u] = x[u]/deg[u]; dangling mass D; y := 0
template <typename T>
__global__ void k_pr_contrib(const T *__restrict__ x, const uint32_t *__restrict__ deg, T *__restrict__ contrib,
                             T *__restrict__ y, uint32_t V, double *dsum) {
  __shared__ double red[32];
  double dl = 0;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t dg = deg[v];
    T xv = x[v];
    contrib[v] = dg ? xv / T(dg) : T(0);
    if (!dg) dl += (double)xv;
    y[v] = T(0);
  }
  double s = block_sum_d<T>(dl, red);
  if (threadIdx.x == 0 && s != 0) atomicAdd(dsum, s);
}

template <typename T>
__global__ void k_pr_push(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val, uint64_t cap,
                          const T *__restrict__ contrib, T *y) {
  for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < cap;
       s += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t k;
    if (!edge_at(key, val, s, &k)) continue;
    atomicAdd(&y[(uint32_t)k], contrib[k >> 32]);
  }
}

template <typename T>
__global__ void k_pr_update(T *__restrict__ x, const T *__restrict__ y, uint32_t V, T d,
                            const double *__restrict__ dsum, double *err) {
  __shared__ double red[32];
  const T base = (T(1) - d) / T(V) + d * T(*dsum / (double)V);
  double e = 0;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x) {
    T nx = base + d * y[v];
    e += fabs((double)nx - (double)x[v]);
    x[v] = nx;
  }
  double s = block_sum_d<T>(e, red);
  if (threadIdx.x == 0 && s != 0) atomicAdd(err, s);
}

template <typename T>
static gpma_status pagerank_t(gpma *g, T *x, int warm, T d, double tol, int max_iter, int *iters,
                              cudaStream_t s) {
  const uint64_t V = g->V;
  GP_CHECK(g, ensure(g->b_misc, (V + 1) * 4, s));
  GP_CHECK(g, ensure(g->b_misc2, (V + 1) * sizeof(T), s));
  GP_CHECK(g, ensure(g->b_misc3, (V + 1) * sizeof(T), s));
  uint32_t *deg = (uint32_t *)g->b_misc.p;
  T *contrib = (T *)g->b_misc2.p, *y = (T *)g->b_misc3.p;
  double *dsum = (double *)&g->ctrl_d->sum;
  double *err = (double *)&g->ctrl_d->sum2;
  GP_CHECK(g, cudaMemsetAsync(deg, 0, V * 4, s));
  GP_LAUNCH(g, k_pr_outdeg, grid_for(g->cap), TA, 0, s, g->key, g->val, g->cap, deg);
  if (!warm) GP_LAUNCH(g, k_pr_init<T>, grid_for(V), TA, 0, s, x, (uint32_t)V);
  int it = 0;
  while (it < max_iter) {
    GP_CHECK(g, cudaMemsetAsync(&g->ctrl_d->sum, 0, 16, s));
    GP_LAUNCH(g, k_pr_contrib<T>, grid_for(V), TA, 0, s, x, deg, contrib, y, (uint32_t)V, dsum);
    GP_LAUNCH(g, k_pr_push<T>, grid_for(g->cap), TA, 0, s, g->key, g->val, g->cap, contrib, y);
    GP_LAUNCH(g, k_pr_update<T>, grid_for(V), TA, 0, s, x, y, (uint32_t)V, d, dsum, err);
    ++it;
    GP_CHECK(g, cudaMemcpyAsync(&g->ctrl_h->sum2, &g->ctrl_d->sum2, 8, cudaMemcpyDeviceToHost, s));
    GP_CHECK(g, cudaStreamSynchronize(s));
    double e;
    memcpy(&e, &g->ctrl_h->sum2, 8);
    if (e < tol) break;
  }
  if (iters) *iters = it;
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status pagerank_f64(gpma *g, double *x, int warm, double d, double tol, int max_iter, int *iters,
                         cudaStream_t s) {
  return pagerank_t<double>(g, x, warm, d, tol, max_iter, iters, s);
}

gpma_status pagerank_f32(gpma *g, float *x, int warm, float d, float tol, int max_iter, int *iters,
                         cudaStream_t s) {
  return pagerank_t<float>(g, x, warm, d, (double)tol, max_iter, iters, s);
}

// ------------------------------------------------------------------ export CSR
__global__ void k_exp_leafcount(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val,
                                uint32_t L, uint64_t nleaves, uint64_t *lc) {
  for (uint64_t l = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; l < nleaves;
       l += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t c = 0, k;
    for (uint32_t p = 0; p < L; ++p) c += edge_at(key, val, l * L + p, &k);
    lc[l] = c;
  }
}

__global__ void k_exp_write(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val, uint32_t L,
                            uint64_t cap, const uint64_t *__restrict__ lbase, uint64_t *__restrict__ row_ptr,
                            uint32_t *__restrict__ col, uint32_t *__restrict__ cval) {
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint32_t leafmask = (L == 32 ? 0xffffffffu : ((1u << L) - 1u) << (lane & ~(L - 1)));
  const uint64_t capr = (cap + 31) & ~31ull;
  for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < capr;
       s += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t k = KEY_NONE;
    bool e = s < cap && edge_at(key, val, s, &k);
    uint32_t bal = __ballot_sync(0xffffffffu, e);
    if (s >= cap) continue;
    uint64_t r = lbase[s / L] + __popc(bal & leafmask & lt);
    if (e) {
      col[r] = (uint32_t)k;
      cval[r] = val[s];
    } else if (is_guard_key(k)) {
      row_ptr[(k >> 32) + 1] = r;
    }
  }
}

gpma_status export_csr(gpma *g, uint64_t *row_ptr, uint32_t *col, uint32_t *val, uint64_t cap_nnz,
                       uint64_t *nnz_out, cudaStream_t s) {
  const uint64_t nl = g->cap / g->L;
  GP_CHECK(g, ensure(g->b_lpre, (nl + 1) * 8, s));
  uint64_t *lc = (uint64_t *)g->b_lpre.p;
  GP_LAUNCH(g, k_exp_leafcount, grid_for(nl), TA, 0, s, g->key, g->val, g->L, nl, lc);
  scan_u64(g, lc, lc, nl, s);
  GP_CHECK(g, cudaMemcpyAsync(&g->ctrl_h->sum, lc + nl, 8, cudaMemcpyDeviceToHost, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  uint64_t nnz = g->ctrl_h->sum;
  if (nnz_out) *nnz_out = nnz;
  if (!col) return GPMA_OK;
  if (cap_nnz < nnz) {
    g->err = "export_csr: nnz_capacity too small";
    return GPMA_ERR_INVALID_ARG;
  }
  GP_CHECK(g, cudaMemsetAsync(row_ptr, 0, 8, s));
  GP_LAUNCH(g, k_exp_write, grid_for(g->cap), TA, 0, s, g->key, g->val, g->L, g->cap, lc, row_ptr, col,
            val);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

}  // namespace gp
