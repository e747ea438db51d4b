// analytics.cu -- graph analytics that read the gapped CSR in place (sm_100a).
//
// "CSR on GPMA" (Fig. 5): row u occupies slots [row_offset[u], row_offset[u+1]);
// a slot holds an edge iff it is occupied, not a guard and not a tombstone -- the
// IsEntryExist test of Alg. 2 l.10 / Alg. 3 l.4.  Sweeps read the key array
// and the per-leaf tombstone mask (8.25 B/slot) instead of key + value (12 B/slot); keys are
// loaded with streaming (evict-first) hints so the random-access vertex arrays keep L2.
//
//   BFS  (Table 1: Merrill et al. [37]): level-synchronous top-down BFS.  A level's frontier
//        is rebuilt from levels[] (bitmap + list, no atomics on the critical path); small
//        frontiers expand their rows load-balanced over slots (Neighbour Gathering, Alg. 3);
//        large ones sweep only the leaves whose source range meets the frontier.  Discovery
//        is a plain store of the depth (every racing writer stores the same value).
//   CC   (Table 1: Soman et al. [43]): hooking of roots (larger id under smaller) with CAS
//        and path halving; a sampled first round (first edge of every (source, leaf) run),
//        full compression, then a full pass that skips edges whose endpoints already share
//        a parent.  Roots are component minima -> canonical min-id labels (R19).
//   PR   (Table 1: CUSP SpMV [2]): push SpMV over the live slots with the
//        store-maintained out-degrees; x' / error / dangling / next contribution fused.  The
//        fp64 path accumulates y in exact 64-bit fixed point (2^-62 units; y <= total rank
//        mass <= 1) with integer REDs: order-independent and within 2^-63 per term.
//   export: per-leaf edge counts (leaf live counts minus guards), one scan, one sweep.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstdlib>
#include <cstring>

#include "gpma_internal.cuh"
#include "sweep.cuh"

namespace gp {

constexpr int TA = 256;

// ------------------------------------------------------------------ slot access
struct Slot4 {
  uint64_t k[4];
  uint32_t tb;   // tombstone bits of the four slots
};

// four consecutive slots (s4 % 4 == 0; L >= 4 so they share a leaf)
__device__ __forceinline__ void load4(const uint64_t *__restrict__ key, const uint32_t *__restrict__ tmask,
                                      uint32_t L, uint64_t s4, Slot4 &o) {
  ulonglong2 a = __ldcs(reinterpret_cast<const ulonglong2 *>(key + s4));
  ulonglong2 b = __ldcs(reinterpret_cast<const ulonglong2 *>(key + s4 + 2));
  o.k[0] = a.x; o.k[1] = a.y; o.k[2] = b.x; o.k[3] = b.y;
  o.tb = (__ldg(tmask + leaf_div(s4, L)) >> leaf_mod(s4, L)) & 0xFu;
}

__device__ __forceinline__ uint64_t l2_evict_last_policy() {
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(pol));
  return pol;
}

__device__ __forceinline__ bool live_key(uint64_t k) { return k != KEY_NONE && (uint32_t)k != COL_GUARD; }
__device__ __forceinline__ bool edge4(const Slot4 &o, int j) { return live_key(o.k[j]) && !((o.tb >> j) & 1u); }

__device__ __forceinline__ bool edge_at(const uint64_t *__restrict__ key, const uint32_t *__restrict__ tmask,
                                        uint32_t L, uint64_t s, uint64_t *k) {
  uint64_t x = __ldcs(key + s);
  *k = x;
  if (!live_key(x)) return false;
  return !((__ldg(tmask + leaf_div(s, L)) >> leaf_mod(s, L)) & 1u);
}

__device__ __forceinline__ uint32_t upper_bound_u64(const uint64_t *__restrict__ a, uint32_t lo, uint32_t hi,
                                                    uint64_t x) {
  while (lo < hi) {
    uint32_t mid = (lo + hi) >> 1;
    if (a[mid] <= x) lo = mid + 1;
    else hi = mid;
  }
  return lo;
}

// ------------------------------------------------------------------ out-degrees
// out-degree of each row = live edges in it.  Per thread: runs of equal source over its 4
// slots; the thread's first run is aggregated across the warp (hub rows span many lanes).
__global__ void __launch_bounds__(TA) k_deg_count(const uint64_t *__restrict__ key,
                                                  const uint32_t *__restrict__ tmask, uint32_t L, uint64_t cap,
                                                  uint32_t *deg, uint32_t rb) {
  const int lane = threadIdx.x & 31;
  const uint64_t n4 = cap / 4, n4r = (n4 + 31) & ~31ull;
  for (uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; t < n4r;
       t += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t first_src = 0xFFFFFFFFu, first_cnt = 0, cur = 0xFFFFFFFFu, c = 0;
    bool in_first = true;
    if (t < n4) {
      Slot4 sl;
      load4(key, tmask, L, t * 4, sl);
#pragma unroll
      for (int j = 0; j < 4; ++j) {
        if (!edge4(sl, j)) continue;
        uint32_t u = (uint32_t)(sl.k[j] >> 32) - rb;   // local row
        if (u == cur) { ++c; continue; }
        if (c) {
          if (in_first) { first_src = cur; first_cnt = c; in_first = false; }
          else atomicAdd(&deg[cur], c);
        }
        cur = u;
        c = 1;
      }
      if (c) {
        if (in_first) { first_src = cur; first_cnt = c; }
        else atomicAdd(&deg[cur], c);
      }
    }
    uint32_t peers = __match_any_sync(0xffffffffu, first_src);
    uint32_t sum = __reduce_add_sync(peers, first_cnt);
    if (first_src != 0xFFFFFFFFu && (__ffs(peers) - 1) == lane) atomicAdd(&deg[first_src], sum);
  }
}

gpma_status recompute_degrees(gpma *g, cudaStream_t s) {
  GP_CHECK(g, fill_zero(g, g->deg, (uint64_t)g->nr * 4, s));
  GP_LAUNCH(g, k_deg_count, grid_for(g->cap / 4), TA, 0, s, g->key, tmask_of(g), g->L, g->cap, g->deg, g->rb);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// ------------------------------------------------------------------ BFS
__global__ void k_bfs_init(int32_t *levels, uint32_t V, uint32_t root) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x)
    levels[v] = (v == root) ? 0 : -1;
}

__global__ void k_bfs_set_bit(uint32_t *bm, uint32_t v) {
  if (threadIdx.x == 0) bm[v >> 5] |= 1u << (v & 31);
}

// frontier of depth d: bitmap words written whole by one lane per 32 vertices; size into *F
// (one atomic per CTA)
__global__ void k_bfs_frontier(const int32_t *__restrict__ levels, uint32_t V, int32_t d,
                               uint32_t *__restrict__ bm, uint32_t *F) {
  __shared__ uint32_t cnt;
  if (threadIdx.x == 0) cnt = 0;
  __syncthreads();
  const int lane = threadIdx.x & 31;
  const uint64_t Vr = ((uint64_t)V + 31) & ~31ull;
  uint32_t mine = 0;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < Vr;
       v += (uint64_t)gridDim.x * blockDim.x) {
    bool in = v < V && levels[v] == d;
    uint32_t bal = __ballot_sync(0xffffffffu, in);
    if (lane == 0) {
      bm[v >> 5] = bal;
      mine += __popc(bal);
    }
  }
  if (lane == 0 && mine) atomicAdd(&cnt, mine);
  __syncthreads();
  if (threadIdx.x == 0 && cnt) atomicAdd(F, cnt);
}

// frontier list from the bitmap (sparse levels only: few set bits)
// (zero != nullptr: also clears the next level's frontier bitmap, same word range -- one launch less)
__global__ void k_bfs_list(const uint32_t *__restrict__ bm, uint32_t nwords, uint32_t *__restrict__ list,
                           uint32_t *n, uint32_t *__restrict__ zero) {
  for (uint64_t w = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; w < nwords;
       w += (uint64_t)gridDim.x * blockDim.x) {
    if (zero) zero[w] = 0u;
    uint32_t b = bm[w];
    if (!b) continue;
    uint32_t base = atomicAdd(n, (uint32_t)__popc(b));
    while (b) {
      int i = __ffs(b) - 1;
      b &= b - 1;
      list[base++] = (uint32_t)(w * 32 + i);
    }
  }
}

__global__ void k_bfs_rowlen(const uint32_t *__restrict__ frontier, uint32_t F,
                             const uint64_t *__restrict__ row_offset, uint32_t rb, uint32_t nr,
                             uint64_t *__restrict__ len) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < F;
       i += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t u = frontier[i] - rb;                  // rows outside the shard are empty here
    len[i] = u < nr ? row_offset[u + 1] - row_offset[u] : 0;
  }
}

// Discovery of v at `depth`.  With a next-frontier bitmap (single-store BFS) the first
// discoverer also sets v's bit and counts it, so the next level needs no sweep over `levels`
// to find its frontier.  Racing discoverers all store the same depth; the atomicOr's old
// value picks exactly one of them for the count.
__device__ __forceinline__ uint32_t bfs_discover(int32_t *levels, uint32_t v, int32_t depth, uint32_t *bm_next) {
  if (levels[v] != -1) return 0;
  levels[v] = depth;
  if (!bm_next) return 0;
  const uint32_t bit = 1u << (v & 31);
  return (atomicOr(bm_next + (v >> 5), bit) & bit) ? 0u : 1u;
}

__device__ __forceinline__ void bfs_count(uint32_t found, uint32_t *fnext) {
  found = __reduce_add_sync(0xffffffffu, found);
  if ((threadIdx.x & 31) == 0 && found) atomicAdd(fnext, found);
}

// Sparse levels -- Neighbour Gathering over the concatenated frontier rows (Alg. 3),
// load-balanced: warp w owns the contiguous slot range [w*C, (w+1)*C) of the concatenation,
// binary-searches its first row once, then walks forward 32 slots at a time.
__global__ void __launch_bounds__(TA) k_bfs_expand(const uint32_t *__restrict__ frontier, uint32_t F,
                                                   const uint64_t *__restrict__ off,
                                                   const uint64_t *__restrict__ row_offset,
                                                   const uint64_t *__restrict__ key,
                                                   const uint32_t *__restrict__ tmask, uint32_t L,
                                                   int32_t *levels, int32_t depth, uint32_t rb,
                                                   uint32_t *bm_next, uint32_t *fnext) {
  const int lane = threadIdx.x & 31;
  const uint64_t total = off[F];
  const uint64_t nwarps = (uint64_t)gridDim.x * (blockDim.x / 32);
  const uint64_t w = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32;
  const uint64_t chunk = ((total + nwarps - 1) / nwarps + 31) & ~31ull;
  const uint64_t beg = w * chunk, end = min(beg + chunk, total);
  if (beg >= end) return;
  uint32_t i0 = 0;
  if (lane == 0) i0 = upper_bound_u64(off, 0, F + 1, beg) - 1;
  i0 = __shfl_sync(0xffffffffu, i0, 0);
  uint32_t found = 0;
  for (uint64_t base = beg; base < end; base += 32) {
    const uint64_t gi = base + lane;
    uint32_t i = i0;
    if (gi < end) {
      while (off[i + 1] <= gi) ++i;
      uint32_t u = frontier[i] - rb;
      uint64_t s = row_offset[u] + (gi - off[i]);
      uint64_t k;
      if (edge_at(key, tmask, L, s, &k)) found += bfs_discover(levels, (uint32_t)k, depth, bm_next);
    }
    i0 = __shfl_sync(0xffffffffu, i, 31);
  }
  if (fnext) bfs_count(found, fnext);
}

// A leaf is active when its source range holds a frontier vertex.  The range comes from the
// locate heads (every vertex has a guard, so a leaf spans at most L sources).
// Active leaves appended to alist: a CTA tests 4 x 256 consecutive leaves (head loads first,
// then the bitmap probes), ranks them with ballots + a 32-entry CTA scan and reserves its
// slots with ONE atomic.  The CTA order in alist does not matter to the sweep.
constexpr int BFS_LA_K = 4;
__global__ void __launch_bounds__(TA) k_bfs_leaf_active(const uint64_t *__restrict__ head, uint64_t nleaves,
                                                        uint32_t V, const uint32_t *__restrict__ bm,
                                                        uint32_t *__restrict__ alist, uint32_t *__restrict__ nact,
                                                        uint32_t *__restrict__ zero, uint32_t zwords) {
  static_assert(BFS_LA_K * (TA / 32) == 32, "one warp scans the per-warp counts");
  __shared__ uint32_t wofs[BFS_LA_K * (TA / 32)];
  if (zero)                                              // the next level's frontier bitmap
    for (uint64_t w = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; w < zwords;
         w += (uint64_t)gridDim.x * blockDim.x)
      zero[w] = 0u;
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint64_t per = (uint64_t)TA * BFS_LA_K;
  for (uint64_t b0 = blockIdx.x * per; b0 < nleaves; b0 += (uint64_t)gridDim.x * per) {
    uint64_t h0[BFS_LA_K], h1[BFS_LA_K];
#pragma unroll
    for (int k = 0; k < BFS_LA_K; ++k) {
      const uint64_t l = b0 + k * TA + threadIdx.x;
      h0[k] = l < nleaves ? head[l] : KEY_NONE;
      h1[k] = l + 1 < nleaves ? head[l + 1] : KEY_NONE;
    }
    uint32_t act[BFS_LA_K], bal[BFS_LA_K];
#pragma unroll
    for (int k = 0; k < BFS_LA_K; ++k) {
      act[k] = 0;
      if (h0[k] != KEY_NONE) {
        const uint32_t ua = (uint32_t)(h0[k] >> 32);
        const uint32_t ub = min(h1[k] == KEY_NONE ? V - 1 : (uint32_t)(h1[k] >> 32), V - 1);
        // frontier bits of sources [ua, ub], a word at a time (one or two words when every
        // row has its guard: a leaf spans at most L + 1 sources)
        const uint32_t w0 = ua >> 5, w1 = ub >> 5;
        for (uint32_t w = w0; w <= w1 && ua <= ub; ++w) {
          uint32_t m = __ldg(bm + w);
          if (w == w0) m &= ~0u << (ua & 31);
          if (w == w1 && (ub & 31) != 31) m &= (2u << (ub & 31)) - 1u;
          if (m) { act[k] = 1; break; }
        }
      }
      bal[k] = __ballot_sync(0xffffffffu, act[k]);
      if (lane == 0) wofs[k * (TA / 32) + warp] = __popc(bal[k]);
    }
    __syncthreads();
    if (threadIdx.x < 32) {                         // exclusive scan of the 32 warp counts
      const uint32_t v = wofs[threadIdx.x];
      uint32_t x = v;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
        if (lane >= o) x += y;
      }
      const uint32_t tot = __shfl_sync(0xffffffffu, x, 31);
      uint32_t base = 0;
      if (lane == 0 && tot) base = atomicAdd(nact, tot);
      base = __shfl_sync(0xffffffffu, base, 0);
      wofs[threadIdx.x] = base + x - v;
    }
    __syncthreads();
    const uint32_t lt = (1u << lane) - 1u;
#pragma unroll
    for (int k = 0; k < BFS_LA_K; ++k)
      if (act[k]) alist[wofs[k * (TA / 32) + warp] + __popc(bal[k] & lt)] = (uint32_t)(b0 + k * TA + threadIdx.x);
    __syncthreads();
  }
}

// Dense levels: sweep the active leaves, two groups of 4 slots per thread, expanding the
// edges whose source is in the frontier bitmap.
__global__ void __launch_bounds__(TA) k_bfs_sweep(const uint64_t *__restrict__ key,
                                                  const uint32_t *__restrict__ tmask, uint32_t L,
                                                  const uint32_t *__restrict__ alist,
                                                  const uint32_t *__restrict__ nact_p,
                                                  const uint32_t *__restrict__ bm, int32_t *levels,
                                                  int32_t depth, uint32_t *bm_next, uint32_t *fnext) {
  const uint32_t tpl = L / 4;
  uint32_t found = 0;
  const uint64_t n4 = (uint64_t)(*nact_p) * tpl;
  for (uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; t < n4;
       t += (uint64_t)gridDim.x * blockDim.x) {
    Slot4 sl;
    load4(key, tmask, L, (uint64_t)alist[leaf_div(t, tpl)] * L + leaf_mod(t, tpl) * 4, sl);   // tpl = L/4: a power of two
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      if (!edge4(sl, j)) continue;
      uint32_t u = (uint32_t)(sl.k[j] >> 32), v = (uint32_t)sl.k[j];
      if (!((__ldg(bm + (u >> 5)) >> (u & 31)) & 1u)) continue;
      found += bfs_discover(levels, v, depth, bm_next);
    }
  }
  if (fnext) bfs_count(found, fnext);
}

// frontiers up to this size use row expansion (GPMA_BFS_SPARSE overrides)
static uint32_t bfs_sparse_f() {
  const char *e = getenv("GPMA_BFS_SPARSE");              // read per call: tests switch it
  return e ? (uint32_t)atol(e) : 32768u;
}

// read back nwords words to pinned host memory, then clear zwords words at zero (one launch)
__global__ void k_readback_zero(uint32_t *dst, const uint32_t *src, uint32_t nwords, uint32_t *zero, uint32_t zwords) {
  for (uint32_t i = threadIdx.x; i < nwords; i += blockDim.x) dst[i] = src[i];
  __syncwarp();
  for (uint32_t i = threadIdx.x; i < zwords; i += blockDim.x) zero[i] = 0u;
}

gpma_status bfs_init(gpma *g, uint32_t root, int32_t *levels, cudaStream_t s) {
  GP_LAUNCH(g, k_bfs_init, grid_for(g->V), TA, 0, s, levels, g->V, root);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// Expand the frontier bitmap `bm` (F vertices) by one level: sparse -- row expansion over the
// frontier list; dense -- sweep of the active leaves.  Discoveries get `depth`; with bm_next
// they are also marked there and counted into *fnext (device).
static gpma_status bfs_expand_level(gpma *g, Scratch &X, int32_t *levels, int32_t depth, const uint32_t *bm,
                                    uint32_t F, uint32_t *bm_next, uint32_t *fnext, cudaStream_t s,
                                    uint32_t *zero_next = nullptr, bool cnt_zeroed = false) {
  const uint64_t V = g->V, nl = g->cap / g->L;
  GP_CHECK(g, ensure(g, X.b[0], (V + 1) * 4, s));
  GP_CHECK(g, ensure(g, X.misc, (nl + 2) * 4, s));
  uint32_t *list = (uint32_t *)X.b[0].p;
  uint32_t *alist = (uint32_t *)X.misc.p;
  uint32_t *cnt_d = reinterpret_cast<uint32_t *>(&X.ctrl_d->sum2);   // list / active-leaf count
  const uint32_t *tmask = tmask_of(g);
  if (!cnt_zeroed) GP_CHECK(g, fill_zero(g, cnt_d, 4, s));
  if (F <= bfs_sparse_f()) {
    GP_CHECK(g, ensure(g, X.b[2], ((uint64_t)bfs_sparse_f() + 2) * 8, s));   // fixed size: no regrowth per level
    uint64_t *off = (uint64_t *)X.b[2].p;
    GP_LAUNCH(g, k_bfs_list, grid_for((V + 31) / 32), TA, 0, s, bm, (uint32_t)((V + 31) / 32), list, cnt_d, zero_next);
    GP_LAUNCH(g, k_bfs_rowlen, grid_for(F), TA, 0, s, list, F, g->row_offset, g->rb, g->nr, off);
    GP_CHECK(g, scan_u64(g, off, off, F, s));
    GP_LAUNCH(g, k_bfs_expand, grid_cap(), TA, 0, s, list, F, off, g->row_offset, g->key, tmask, g->L,
              levels, depth, g->rb, bm_next, fnext);
  } else {
    GP_LAUNCH(g, k_bfs_leaf_active, grid_for(nl), TA, 0, s, g->head, nl, (uint32_t)V, bm, alist, cnt_d, zero_next,
              (uint32_t)((V + 31) / 32 + 1));
    GP_LAUNCH(g, k_bfs_sweep, grid_cap(), TA, 0, s, g->key, tmask, g->L, alist, cnt_d, bm, levels, depth,
              bm_next, fnext);
  }
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// Multi-GPU BFS exchange: a rank's discoveries of one level as a bitmap
// (bit v = levels[v] == depth), and the merge of every rank's bitmap into levels.
__global__ void k_bfs_bits(const int32_t *__restrict__ levels, uint32_t V, int32_t d, uint32_t *__restrict__ bm) {
  const uint64_t Vr = ((uint64_t)V + 31) & ~31ull;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < Vr; v += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t b = __ballot_sync(0xffffffffu, v < V && levels[v] == d);
    if ((threadIdx.x & 31) == 0) bm[v >> 5] = b;
  }
}

__global__ void k_bfs_merge(int32_t *__restrict__ levels, uint32_t V, const uint32_t *__restrict__ bms,
                            uint32_t nbm, uint64_t words, int32_t d) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V; v += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t any = 0;
    for (uint32_t r = 0; r < nbm; ++r) any |= __ldg(bms + r * words + (v >> 5));
    if (((any >> (v & 31)) & 1u) && levels[v] == -1) levels[v] = d;
  }
}

gpma_status bfs_bits(gpma *g, const int32_t *levels, int32_t depth, uint32_t *bm, cudaStream_t s) {
  GP_LAUNCH(g, k_bfs_bits, grid_for(((uint64_t)g->V + 31) & ~31ull), TA, 0, s, levels, g->V, depth, bm);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status bfs_merge(gpma *g, int32_t *levels, const uint32_t *bms, uint32_t nbm, int32_t depth, cudaStream_t s) {
  const uint64_t words = ((uint64_t)g->V + 31) / 32;
  GP_LAUNCH(g, k_bfs_merge, grid_for(g->V), TA, 0, s, levels, g->V, bms, nbm, words, depth);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// One BFS level of a (possibly sharded) store: the frontier is {v : levels[v] == depth-1}
// (levels may be replicated across shards); the owned rows of the frontier are expanded and
// newly reached vertices get `depth`.  *frontier = the frontier size (0: nothing expanded).
gpma_status bfs_level(gpma *g, int32_t *levels, int32_t depth, uint32_t *frontier, cudaStream_t s) {
  Scratch &X = g->an[AN_BFS];
  ScanScope scan_scope_(X.scan);
  const uint64_t V = g->V;
  GP_CHECK(g, ensure(g, X.b[3], (V / 32 + 2) * 4, s));
  uint32_t *bm = (uint32_t *)X.b[3].p;
  uint32_t *F_d = reinterpret_cast<uint32_t *>(&X.ctrl_d->sum);
  GP_CHECK(g, fill_zero(g, F_d, 4, s));
  GP_LAUNCH(g, k_bfs_frontier, grid_for(V), TA, 0, s, levels, (uint32_t)V, depth - 1, bm, F_d);
  GP_CHECK(g, readback(g, &X.ctrl_h->sum, F_d, 4, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  const uint32_t F = (uint32_t)(X.ctrl_h->sum & 0xFFFFFFFFu);
  *frontier = F;
  if (!F) return GPMA_OK;
  return bfs_expand_level(g, X, levels, depth, bm, F, nullptr, nullptr, s);
}

// Whole-store BFS (Alg. 3 level by level): each level's discoveries build the next frontier
// bitmap directly; one host read of the frontier size per level.
gpma_status bfs(gpma *g, uint32_t root, int32_t *levels, cudaStream_t s) {
  Scratch &X = g->an[AN_BFS];
  ScanScope scan_scope_(X.scan);
  const uint64_t V = g->V, words = (V + 31) / 32 + 1;
  GP_CHECK(g, ensure(g, X.b[3], words * 4, s));
  GP_CHECK(g, ensure(g, X.b[1], words * 4, s));
  uint32_t *bm[2] = {(uint32_t *)X.b[3].p, (uint32_t *)X.b[1].p};
  uint32_t *F_d = reinterpret_cast<uint32_t *>(&X.ctrl_d->sum);
  GP_CHECK(g, fill_zero(g, bm[0], words * 4, s));
  GP_LAUNCH(g, k_bfs_init, grid_for(V), TA, 0, s, levels, g->V, root);
  GP_LAUNCH(g, k_bfs_set_bit, 1, 32, 0, s, bm[0], root);
  uint32_t F = 1;
  int cur = 0;
  // per level: the expansion kernels clear the next frontier bitmap themselves and the read-back
  // of the frontier size clears the level counters (k_readback_zero) -- no zero-fill launches
  GP_CHECK(g, fill_zero(g, &X.ctrl_d->sum, 16, s));     // F_d and the list / active-leaf counter
  for (int32_t depth = 1; F; ++depth, cur ^= 1) {
    gpma_status st = bfs_expand_level(g, X, levels, depth, bm[cur], F, bm[cur ^ 1], F_d, s, bm[cur ^ 1], true);
    if (st) return st;
    g->launches++;
    k_readback_zero<<<1, 32, 0, s>>>((uint32_t *)&X.ctrl_h->sum, (const uint32_t *)F_d, 1u,
                                     (uint32_t *)&X.ctrl_d->sum, 4u);
    GP_CHECK(g, cudaGetLastError());
    GP_CHECK(g, cudaStreamSynchronize(s));
    F = (uint32_t)(X.ctrl_h->sum & 0xFFFFFFFFu);
  }
  return GPMA_OK;
}

// ------------------------------------------------------------------ CC
// Parent-array accesses may carry an L2 evict_last hint (H): the 64 MB forest stays resident
// while the key stream passes through L2 evict-first.

template <bool H>
__device__ __forceinline__ uint32_t cc_ld(const uint32_t *a, uint64_t pol) {
  uint32_t v;
  if (H) asm volatile("ld.relaxed.gpu.global.L2::cache_hint.u32 %0, [%1], %2;" : "=r"(v) : "l"(a), "l"(pol) : "memory");
  else v = *(const volatile uint32_t *)a;
  return v;
}

template <bool H>
__device__ __forceinline__ void cc_st(uint32_t *a, uint32_t v, uint64_t pol) {
  if (H) asm volatile("st.relaxed.gpu.global.L2::cache_hint.u32 [%0], %1, %2;" ::"l"(a), "r"(v), "l"(pol) : "memory");
  else *(volatile uint32_t *)a = v;
}

template <bool H>
__device__ __forceinline__ uint32_t cc_cas(uint32_t *a, uint32_t cmp, uint32_t v, uint64_t) {
  return atomicCAS(a, cmp, v);                 // (atom.cas takes no L2 cache hint on sm_100a)
}

// F: chain steps through L1 (a stale parent is still an ancestor; the CAS in cc_hook checks
// rootness against L2), so a giant component's root word is not re-read from one L2 slice by
// every chain
template <bool H, bool F = false>
__device__ __forceinline__ uint32_t cc_find(uint32_t *p, uint32_t x, uint64_t pol) {
  // path halving on a forest with parent[x] <= x (roots are the minima)
  uint32_t cur = cc_ld<H>(p + x, pol);
  if (cur != x) {
    uint32_t prev = x, next;
    while (cur > (next = F ? __ldca(p + cur) : cc_ld<H>(p + cur, pol))) {
      cc_st<H>(p + prev, next, pol);
      prev = cur;
      cur = next;
    }
  }
  return cur;
}

template <bool H, bool F = false>
__device__ __forceinline__ void cc_hook(uint32_t *p, uint32_t u, uint32_t v, uint64_t pol) {
  uint32_t ru = cc_find<H, F>(p, u, pol), rv = cc_find<H, F>(p, v, pol);
  bool repeat;
  do {
    repeat = false;
    if (ru != rv) {
      uint32_t ret;
      if (ru < rv) {
        if ((ret = cc_cas<H>(&p[rv], rv, ru, pol)) != rv) { rv = ret; repeat = true; }
      } else {
        if ((ret = cc_cas<H>(&p[ru], ru, rv, pol)) != ru) { ru = ret; repeat = true; }
      }
    }
  } while (repeat);
}

__global__ void k_cc_init(uint32_t *p, uint32_t V) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x)
    p[v] = (uint32_t)v;
}

// Sample round: hook the first edge of every (source, leaf) run -- roughly the first one or
// two edges of every row (Afforest-style neighbour sampling; any edge subset is a valid first
// round), skipping pairs that already share a parent.  (A CAS-free atomicMin linking of the
// same sample was measured: it halves this round but leaves 4x more work to the full pass.)
template <bool H>
__global__ void __launch_bounds__(TA) k_cc_sample(const uint64_t *__restrict__ key,
                                                  const uint32_t *__restrict__ tmask, uint64_t cap, uint32_t L,
                                                  uint32_t *p) {
  const int lane = threadIdx.x & 31;
  const uint64_t pol = H ? l2_evict_last_policy() : 0;
  const uint64_t n4 = cap / 4, n4r = (n4 + 31) & ~31ull;
  for (uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; t < n4r;
       t += (uint64_t)gridDim.x * blockDim.x) {
    Slot4 sl;
    sl.k[0] = sl.k[1] = sl.k[2] = sl.k[3] = KEY_NONE;
    sl.tb = 0;
    if (t < n4) load4(key, tmask, L, t * 4, sl);
    uint64_t prev = __shfl_up_sync(0xffffffffu, sl.k[3], 1);
    if (lane == 0 && t < n4 && t > 0) prev = key[t * 4 - 1];
    if (t >= n4) continue;
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      const uint64_t s = t * 4 + j;
      const uint64_t pk = j ? sl.k[j - 1] : prev;
      if (!edge4(sl, j)) continue;
      const bool first = (leaf_mod(s, L) == 0) || pk == KEY_NONE || (pk >> 32) != (sl.k[j] >> 32);
      if (!first) continue;
      uint32_t u = (uint32_t)(sl.k[j] >> 32), v = (uint32_t)sl.k[j];
      if (u != v && cc_ld<H>(p + u, pol) != cc_ld<H>(p + v, pol)) cc_hook<H>(p, u, v, pol);
    }
  }
}

// Sample round over the rows (guard-indexed stores): each owned row hooks its first NS live
// edges, found from row_offset (R8) -- slot row_offset[u] + 1 follows guard u-1 -- instead
// of sweeping every slot; the scan skips a leaf's empty tail and stops at guard u.
template <bool H, int NS, bool F = false>
__global__ void __launch_bounds__(TA) k_cc_sample_rows(const uint64_t *__restrict__ key,
                                                       const uint32_t *__restrict__ tmask,
                                                       const uint64_t *__restrict__ row_offset, uint32_t L,
                                                       uint32_t nr, uint32_t rb, uint32_t *p) {
  const uint64_t pol = H ? l2_evict_last_policy() : 0;
  for (uint64_t r = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; r < nr; r += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t sl = r ? row_offset[r] + 1 : 0;
    const uint64_t e = row_offset[r + 1];
    const uint32_t u = (uint32_t)r + rb;
    int found = 0;
    for (int it = 0; sl < e && found < NS && it < 64; ++it, ++sl) {
      const uint64_t k = __ldcs(key + sl);
      if (k == KEY_NONE) {                 // empty tail of a leaf: continue at the next leaf
        sl |= (uint64_t)(L - 1);
        continue;
      }
      if ((__ldg(tmask + leaf_div(sl, L)) >> leaf_mod(sl, L)) & 1u) continue;   // tombstone
      const uint32_t v = (uint32_t)k;
      ++found;
      if (u != v && cc_ld<H>(p + u, pol) != cc_ld<H>(p + v, pol)) cc_hook<H, F>(p, u, v, pol);
    }
  }
}

// Root of every vertex, CC_ILP vertices per thread chased in lockstep.  Chain steps load
// through L1 (ld.global.ca): almost every chain ends on the giant component's root, and one L2
// word read by every warp serialised the pass on its slice.  A stale L1 value is still an
// ancestor (compression only moves parents toward the root, roots never change here), so
// every chain still ends on its root.  out == p: full compression in place; else out[v] = root.
constexpr int CC_ILP = 4;
__device__ __forceinline__ void cc_roots(uint32_t *p, uint32_t *out, uint32_t V) {
  volatile uint32_t *vp = p;
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t v0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v0 < V; v0 += CC_ILP * stride) {
    uint32_t x[CC_ILP];
    uint32_t live = 0;                                     // bit j: chain j not at its root yet
#pragma unroll
    for (int j = 0; j < CC_ILP; ++j) {
      const uint64_t v = v0 + j * stride;
      x[j] = v < V ? vp[v] : 0u;
      if (v < V) live |= 1u << j;
    }
    while (live) {
#pragma unroll
      for (int j = 0; j < CC_ILP; ++j) {
        if (!((live >> j) & 1u)) continue;
        const uint32_t nx = __ldca(p + x[j]);
        if (nx == x[j]) live &= ~(1u << j);
        else x[j] = nx;
      }
    }
#pragma unroll
    for (int j = 0; j < CC_ILP; ++j) {
      const uint64_t v = v0 + j * stride;
      if (v < V) {
        if (out == p) vp[v] = x[j];
        else out[v] = x[j];
      }
    }
  }
}

__global__ void k_cc_compress(uint32_t *p, uint32_t V) { cc_roots(p, p, V); }

template <bool H, bool F = false>
__device__ __forceinline__ void cc_group(const Slot4 &sl, uint32_t *p, uint64_t pol) {
  uint32_t pu[4], pv[4];
#pragma unroll
  for (int j = 0; j < 4; ++j) {             // independent parent loads first
    pu[j] = pv[j] = 0;
    if (edge4(sl, j)) {
      if (F) {            // same-tree filter through L1: a stale parent is an ancestor, so equal
                          // parents still prove one tree; a miss costs the exact find + CAS
        pu[j] = __ldca(p + (uint32_t)(sl.k[j] >> 32));
        pv[j] = __ldca(p + (uint32_t)sl.k[j]);
      } else {
        pu[j] = cc_ld<H>(p + (uint32_t)(sl.k[j] >> 32), pol);
        pv[j] = cc_ld<H>(p + (uint32_t)sl.k[j], pol);
      }
    }
  }
#pragma unroll
  for (int j = 0; j < 4; ++j) {
    if (!edge4(sl, j) || pu[j] == pv[j]) continue;   // same tree already (fast path)
    uint32_t u = (uint32_t)(sl.k[j] >> 32), v = (uint32_t)sl.k[j];
    if (u != v) cc_hook<H, F>(p, u, v, pol);
  }
}

template <bool H, bool F = false>
__global__ void __launch_bounds__(TA) k_cc_hook(const uint64_t *__restrict__ key,
                                                const uint32_t *__restrict__ tmask, uint32_t L, uint64_t cap,
                                                uint32_t *p) {
  const uint64_t pol = H ? l2_evict_last_policy() : 0;
  const uint64_t n4 = cap / 4, stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; t < n4; t += 2 * stride) {
    Slot4 a, b;
    const bool hb = t + stride < n4;
    load4(key, tmask, L, t * 4, a);
    if (hb) load4(key, tmask, L, (t + stride) * 4, b);
    cc_group<H, F>(a, p, pol);
    if (hb) cc_group<H, F>(b, p, pol);
  }
}

// find() chain steps through L1 (GPMA_CC_L1, read per call): 0 never, 1 sampled round,
// 2 (default) sampled round and full pass
static int cc_l1_mode() {
  const char *e = getenv("GPMA_CC_L1");
  return e ? atoi(e) : 2;
}
static bool cc_l1() { return cc_l1_mode() != 0; }

static int cc_hint() {
  static const int v = [] { const char *e = getenv("GPMA_CC_HINT"); return e ? atoi(e) : 1; }();
  return v;
}

// sampled first round: row based when every row has its guard (GPMA_CC_SAMPLE=0 forces the
// slot sweep), else the (source, leaf)-run sweep
static int cc_sample_mode() {
  const char *e = getenv("GPMA_CC_SAMPLE");               // read per call: tests switch it
  return e ? atoi(e) : 2;
}

static cudaError_t cc_sample(gpma *g, uint32_t *p, cudaStream_t s) {
  const uint32_t *tmask = tmask_of(g);
  const int m = cc_sample_mode();
  if (g->rows_indexed && m > 0) {
    if (m == 1) GP_LAUNCH(g, (k_cc_sample_rows<true, 1>), grid_for(g->nr, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->row_offset, g->L,
                          g->nr, g->rb, p);
    else if (cc_l1()) GP_LAUNCH(g, (k_cc_sample_rows<true, 2, true>), grid_for(g->nr, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask,
                                g->row_offset, g->L, g->nr, g->rb, p);
    else GP_LAUNCH(g, (k_cc_sample_rows<true, 2>), grid_for(g->nr, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->row_offset, g->L,
                   g->nr, g->rb, p);
  } else if (cc_hint()) {
    GP_LAUNCH(g, k_cc_sample<true>, grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->cap, g->L, p);
  } else {
    GP_LAUNCH(g, k_cc_sample<false>, grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->cap, g->L, p);
  }
  return cudaGetLastError();
}

__global__ void k_cc_final(uint32_t *p, uint32_t *labels, uint32_t V) { cc_roots(p, labels, V); }

__global__ void k_cc_changed(const uint32_t *__restrict__ a, const uint32_t *__restrict__ b, uint32_t V, Ctrl *c) {
  uint64_t n = 0;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x)
    n += a[v] != b[v];
  for (int o = 16; o; o >>= 1) n += __shfl_xor_sync(0xffffffffu, n, o);
  if ((threadIdx.x & 31) == 0 && n) atomicAdd((unsigned long long *)&c->sum, (unsigned long long)n);
}

// One hooking round over the owned edges on top of `labels` (a forest with p[x] <= x, e.g.
// the element-wise minimum of other shards' labels): sampled round, compression, full pass,
// full compression.  *changed = vertices whose label moved (0 on every shard = fixpoint).
gpma_status cc_round(gpma *g, uint32_t *labels, int init, uint64_t *changed, cudaStream_t s) {
  Scratch &X = g->an[AN_CC];
  ScanScope scan_scope_(X.scan);
  const uint64_t V = g->V;
  GP_CHECK(g, ensure(g, X.b[1], (V + 1) * 4, s));
  uint32_t *prev = (uint32_t *)X.b[1].p;
  const uint32_t *tmask = tmask_of(g);
  if (init) GP_LAUNCH(g, k_cc_init, grid_for(V), TA, 0, s, labels, g->V);
  GP_CHECK(g, cudaMemcpyAsync(prev, labels, V * 4, cudaMemcpyDeviceToDevice, s));
  GP_CHECK(g, cc_sample(g, labels, s));
  GP_LAUNCH(g, k_cc_compress, grid_for(V), TA, 0, s, labels, g->V);
  if (cc_l1_mode() >= 2) GP_LAUNCH(g, (k_cc_hook<true, true>), grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->L, g->cap, labels);
  else if (cc_hint()) GP_LAUNCH(g, k_cc_hook<true>, grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->L, g->cap, labels);
  else GP_LAUNCH(g, k_cc_hook<false>, grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->L, g->cap, labels);
  GP_LAUNCH(g, k_cc_compress, grid_for(V), TA, 0, s, labels, g->V);
  GP_CHECK(g, fill_zero(g, &X.ctrl_d->sum, 8, s));
  GP_LAUNCH(g, k_cc_changed, grid_for(V), TA, 0, s, labels, prev, g->V, X.ctrl_d);
  if (!changed) return GPMA_OK;        // (changed == nullptr: the count stays in the control block)
  GP_CHECK(g, readback(g, &X.ctrl_h->sum, &X.ctrl_d->sum, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  *changed = X.ctrl_h->sum;
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status cc(gpma *g, uint32_t *labels, cudaStream_t s) {
  Scratch &X = g->an[AN_CC];
  ScanScope scan_scope_(X.scan);
  GP_CHECK(g, ensure(g, X.b[0], ((uint64_t)g->V + 1) * 4, s));
  uint32_t *p = (uint32_t *)X.b[0].p;
  const uint32_t *tmask = tmask_of(g);
  GP_LAUNCH(g, k_cc_init, grid_for(g->V), TA, 0, s, p, g->V);
  GP_CHECK(g, cc_sample(g, p, s));
  GP_LAUNCH(g, k_cc_compress, grid_for(g->V), TA, 0, s, p, g->V);
  if (cc_l1_mode() >= 2) GP_LAUNCH(g, (k_cc_hook<true, true>), grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->L, g->cap, p);
  else if (cc_hint()) GP_LAUNCH(g, k_cc_hook<true>, grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->L, g->cap, p);
  else GP_LAUNCH(g, k_cc_hook<false>, grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, tmask, g->L, g->cap, p);
  GP_LAUNCH(g, k_cc_final, grid_for(g->V), TA, 0, s, p, labels, g->V);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// ------------------------------------------------------------------ PageRank
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

// Accumulator of the push: exact fixed point for fp64 ranks, plain fp32 for the fp32 API.
template <typename T>
struct PrAcc;
template <>
struct PrAcc<double> {
  using A = unsigned long long;
  static constexpr double SCALE = 4611686018427387904.0;   // 2^62
  __device__ static A enc(double c) { return __double2ull_rn(c * SCALE); }
  __device__ static double dec(A a) { return (double)a * (1.0 / SCALE); }
};
template <>
struct PrAcc<float> {
  using A = float;
  __device__ static A enc(float c) { return c; }
  __device__ static float dec(A a) { return a; }
};

// first iteration: x (given or 1/V), contrib = x/deg, dangling mass D, y = 0
template <typename T>
__global__ void k_pr_prep(T *__restrict__ x, const uint32_t *__restrict__ deg,
                          typename PrAcc<T>::A *__restrict__ contrib, typename PrAcc<T>::A *__restrict__ y,
                          uint32_t V, int init, double *dsum) {
  __shared__ double red[32];
  double dl = 0;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x) {
    T xv = init ? T(1) / T(V) : x[v];
    if (init) x[v] = xv;
    uint32_t dg = deg[v];
    contrib[v] = PrAcc<T>::enc(dg ? xv / T(dg) : T(0));
    if (!dg) dl += (double)xv;
    y[v] = 0;
  }
  double s = block_sum_d(dl, red);
  if (threadIdx.x == 0 && s != 0) atomicAdd(dsum, s);
}

// RED with an L2 eviction-priority hint (evict_last keeps the scattered y lines resident
// while the key stream, loaded evict-first, passes through L2).
__device__ __forceinline__ void red_add_hint(unsigned long long *p, unsigned long long v, uint64_t pol) {
  asm volatile("red.global.add.L2::cache_hint.u64 [%0], %1, %2;" ::"l"(p), "l"(v), "l"(pol) : "memory");
}
__device__ __forceinline__ void red_add_hint(float *p, float v, uint64_t pol) {
  asm volatile("red.global.add.L2::cache_hint.f32 [%0], %1, %2;" ::"l"(p), "f"(v), "l"(pol) : "memory");
}

// Row-window push: warp w sweeps the contiguous slot chunk [beg, end) (leaf aligned).  Keys
// are sorted, so the sources met along the chunk never decrease: lane j keeps contrib[ub + j]
// of a 32-row window in a register and every slot fetches its source's contribution with a
// shuffle -- the sweep is a pure key stream plus fire-and-forget REDs, with no dependent
// global load per slot.  The window moves forward (coalesced 256-B refill) when a source
// leaves it.
template <typename A, int U>
__global__ void __launch_bounds__(TA) k_pr_push_win(const uint64_t *__restrict__ key,
                                                    const uint32_t *__restrict__ tmask,
                                                    const uint64_t *__restrict__ head, uint32_t L, uint64_t cap,
                                                    const A *__restrict__ contrib, A *y, uint32_t rb,
                                                    uint32_t nr, uint32_t dlo, uint32_t dhi, int hint,
                                                    const uint32_t *__restrict__ done) {
  if (done && *done) return;                             // converged on the device (pagerank_t)
  const int lane = threadIdx.x & 31;
  uint64_t pol = 0;
  if (hint == 1) asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(pol));
  if (hint == 2) asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 0.5;" : "=l"(pol));
  const uint64_t nwarps = (uint64_t)gridDim.x * (blockDim.x / 32);
  const uint64_t w = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32;
  const uint64_t chunk = (((cap + nwarps - 1) / nwarps) + 32 * U - 1) / (32 * U) * (32 * U);
  const uint64_t beg = w * chunk, end = min(beg + chunk, cap);
  if (beg >= end) return;
  const uint64_t h0 = head[leaf_div(beg, L)];
  if (h0 == KEY_NONE) return;                            // no key at or after this chunk
  uint32_t ub = (uint32_t)(h0 >> 32) - rb;               // lower bound of the chunk's rows
  A win = (ub + lane < nr) ? __ldcs(contrib + ub + lane) : A(0);
  uint64_t k[U], kn[U];
  uint32_t tb[U], tbn[U];
  auto fetch = [&](uint64_t base, uint64_t *kk, uint32_t *tt) {
#pragma unroll
    for (int j = 0; j < U; ++j) {
      const uint64_t s = base + j * 32 + lane;
      kk[j] = s < end ? __ldcs(key + s) : KEY_NONE;
      tt[j] = s < end ? (__ldg(tmask + leaf_div(s, L)) >> leaf_mod(s, L)) & 1u : 1u;
    }
  };
  fetch(beg, k, tb);
  for (uint64_t base = beg; base < end; base += 32 * U) {
    if (base + 32 * U < end) fetch(base + 32 * U, kn, tbn);      // next group in flight
#pragma unroll
    for (int j = 0; j < U; ++j) {
      const uint32_t dv = (uint32_t)k[j];
      const bool e = live_key(k[j]) && !tb[j] && dv >= dlo && dv < dhi;   // this pass's targets
      const uint32_t u = (uint32_t)(k[j] >> 32) - rb;
      uint32_t pending = __ballot_sync(0xffffffffu, e);
      while (pending) {
        const bool mine = (pending >> lane) & 1u;
        const uint32_t off = mine ? u - ub : 0u;
        const bool in = mine && off < 32u;
        const A c = __shfl_sync(0xffffffffu, win, off & 31u);
        if (in) {
          if (hint) red_add_hint(&y[dv], c, pol);
          else atomicAdd(&y[dv], c);
        }
        pending &= ~__ballot_sync(0xffffffffu, in);
        if (pending) {                                   // slide the window to the next source
          ub = __reduce_min_sync(0xffffffffu, ((pending >> lane) & 1u) ? u : 0xFFFFFFFFu);
          win = (ub + lane < nr) ? __ldcs(contrib + ub + lane) : A(0);
        }
      }
    }
#pragma unroll
    for (int j = 0; j < U; ++j) {
      k[j] = kn[j];
      tb[j] = tbn[j];
    }
  }
}

// Split push (GPMA_PR_SPLIT=1): y is just larger than L2 (8 B x 2^24 = 128 MB vs 126 MB), so
// its REDs miss (RED-bound, not HBM-bound).  The sweep REDs only the edges whose
// destination is in the lower half of y (64 MB, held with evict_last) and appends the others
// as (dst, contribution) records to a spill list (a warp-aggregated append, streamed); a second
// kernel streams the records and REDs them into the upper half (also 64 MB).  Records beyond
// the spill capacity are RED'd directly (always correct).
template <typename A, int U>
__global__ void __launch_bounds__(TA) k_pr_push_split(const uint64_t *__restrict__ key,
                                                      const uint32_t *__restrict__ tmask,
                                                      const uint64_t *__restrict__ head, uint32_t L, uint64_t cap,
                                                      const A *__restrict__ contrib, A *y, uint32_t rb, uint32_t nr,
                                                      uint32_t dsplit, uint32_t *__restrict__ sd, A *__restrict__ sc,
                                                      unsigned long long *__restrict__ scount,
                                                      const uint32_t *__restrict__ done) {
  if (done && *done) return;
  const int lane = threadIdx.x & 31;
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(pol));
  const uint64_t nwarps = (uint64_t)gridDim.x * (blockDim.x / 32);
  const uint64_t w = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32;
  const uint64_t chunk = (((cap + nwarps - 1) / nwarps) + 32 * U - 1) / (32 * U) * (32 * U);
  const uint64_t beg = w * chunk, end = min(beg + chunk, cap);
  if (beg >= end) {
    if (lane == 0) scount[w] = 0;
    return;
  }
  uint64_t nsp = 0;                                      // records spilled by this warp (<= its slots)
  const uint64_t h0 = head[leaf_div(beg, L)];
  if (h0 == KEY_NONE) {
    if (lane == 0) scount[w] = 0;
    return;
  }
  uint32_t ub = (uint32_t)(h0 >> 32) - rb;
  A win = (ub + lane < nr) ? __ldcs(contrib + ub + lane) : A(0);
  uint64_t k[U], kn[U];
  uint32_t tb[U], tbn[U];
  auto fetch = [&](uint64_t base, uint64_t *kk, uint32_t *tt) {
#pragma unroll
    for (int j = 0; j < U; ++j) {
      const uint64_t s = base + j * 32 + lane;
      kk[j] = s < end ? __ldcs(key + s) : KEY_NONE;
      tt[j] = s < end ? (__ldg(tmask + leaf_div(s, L)) >> leaf_mod(s, L)) & 1u : 1u;
    }
  };
  fetch(beg, k, tb);
  for (uint64_t base = beg; base < end; base += 32 * U) {
    if (base + 32 * U < end) fetch(base + 32 * U, kn, tbn);
#pragma unroll
    for (int j = 0; j < U; ++j) {
      const uint32_t dv = (uint32_t)k[j];
      const bool e = live_key(k[j]) && !tb[j];
      const uint32_t u = (uint32_t)(k[j] >> 32) - rb;
      uint32_t pending = __ballot_sync(0xffffffffu, e);
      while (pending) {
        const bool mine = (pending >> lane) & 1u;
        const uint32_t off = mine ? u - ub : 0u;
        const bool in = mine && off < 32u;
        const A c = __shfl_sync(0xffffffffu, win, off & 31u);
        const bool spill = in && dv >= dsplit;
        const uint32_t sb = __ballot_sync(0xffffffffu, spill);
        if (in) {
          if (spill) {                                   // the warp's private spill run (no atomics)
            const uint64_t q = beg + nsp + __popc(sb & ((1u << lane) - 1u));
            __stcs(sd + q, dv);
            __stcs(sc + q, c);
          } else {
            red_add_hint(&y[dv], c, pol);
          }
        }
        nsp += __popc(sb);
        pending &= ~__ballot_sync(0xffffffffu, in);
        if (pending) {
          ub = __reduce_min_sync(0xffffffffu, ((pending >> lane) & 1u) ? u : 0xFFFFFFFFu);
          win = (ub + lane < nr) ? __ldcs(contrib + ub + lane) : A(0);
        }
      }
    }
#pragma unroll
    for (int j = 0; j < U; ++j) {
      k[j] = kn[j];
      tb[j] = tbn[j];
    }
  }
  if (lane == 0) scount[w] = nsp;
}

// the spill runs: warp w of the push wrote scount[w] records at the start of its slot chunk
template <typename A>
__global__ void __launch_bounds__(TA) k_pr_spill_apply(const uint32_t *__restrict__ sd, const A *__restrict__ sc,
                                                       const unsigned long long *__restrict__ scount, uint64_t cap,
                                                       uint64_t nwarps_push, A *y, const uint32_t *__restrict__ done) {
  if (done && *done) return;
  uint64_t pol;
  asm volatile("createpolicy.fractional.L2::evict_last.b64 %0, 1.0;" : "=l"(pol));
  const int lane = threadIdx.x & 31;
  const uint64_t chunk = (((cap + nwarps_push - 1) / nwarps_push) + 32 * 4 - 1) / (32 * 4) * (32 * 4);
  const uint64_t nwarps = (uint64_t)gridDim.x * (blockDim.x / 32);
  for (uint64_t w = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32; w < nwarps_push; w += nwarps) {
    const uint64_t n = scount[w], base = w * chunk;
    for (uint64_t i = lane; i < n; i += 32) red_add_hint(&y[__ldcs(sd + base + i)], __ldcs(sc + base + i), pol);
  }
}

// x' = (1-d)/V + d (y + D/V); err += |x'-x|; next contrib / dangling; y := 0
template <typename T>
__global__ void k_pr_step(T *__restrict__ x, typename PrAcc<T>::A *__restrict__ y,
                          const uint32_t *__restrict__ deg, typename PrAcc<T>::A *__restrict__ contrib,
                          uint32_t V, T d, const double *__restrict__ dsum_in, double *dsum_out, double *err,
                          const uint32_t *__restrict__ done) {
  if (*done) return;
  __shared__ double red[32];
  const T base = (T(1) - d) / T(V) + d * T(*dsum_in / (double)V);
  double e = 0, dl = 0;
  constexpr int PU = 4;                                  // 4 vertices in flight per thread
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t v0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v0 < V; v0 += PU * stride) {
    typename PrAcc<T>::A yo[PU];
    T xo[PU];
    uint32_t dg[PU];
#pragma unroll
    for (int j = 0; j < PU; ++j) {
      const uint64_t v = v0 + j * stride;
      if (v < V) {
        yo[j] = __ldcs(y + v);
        xo[j] = __ldcs(x + v);
        dg[j] = __ldcs(deg + v);
      }
    }
#pragma unroll
    for (int j = 0; j < PU; ++j) {
      const uint64_t v = v0 + j * stride;
      if (v >= V) continue;
      const T nx = base + d * PrAcc<T>::dec(yo[j]);
      e += fabs((double)nx - (double)xo[j]);
      x[v] = nx;
      y[v] = 0;
      contrib[v] = PrAcc<T>::enc(dg[j] ? nx / T(dg[j]) : T(0));
      if (!dg[j]) dl += (double)nx;
    }
  }
  double se = block_sum_d(e, red);
  double sd = block_sum_d(dl, red);
  if (threadIdx.x == 0) {
    if (se != 0) atomicAdd(err, se);
    if (sd != 0) atomicAdd(dsum_out, sd);
  }
}

// Iteration bookkeeping on the device: zero the next error / dangling accumulators (first
// kernel of an iteration), then, after the step, count the iteration and raise `done` once
// the L1 change drops below tol (R20).  Every kernel of a later iteration returns
// at once after `done`, so the host can queue iterations ahead and read back once per batch.
struct PrLoop {
  uint32_t done, iters;
};
__global__ void k_pr_iter_begin(double *acc, int nxt, const PrLoop *lp) {
  if (lp->done || threadIdx.x) return;
  acc[2] = 0.0;
  acc[nxt] = 0.0;
}
__global__ void k_pr_iter_end(const double *acc, double tol, PrLoop *lp) {
  if (lp->done || threadIdx.x) return;
  lp->iters += 1;
  if (acc[2] < tol) lp->done = 1;
}

// Destination passes of the push (GPMA_PR_PASSES, default 1).  Random REDs run ~3x faster
// while their target fits in L2 (tools/micro/red_bench.cu), but each pass re-sweeps the keys;
// at V = 2^24 one pass measured fastest.
// y REDs carry an L2 evict_last hint (GPMA_PR_HINT=0 disables): push 4.72 -> 3.99 ms / 3 iters
// at configs[2]
static int pr_hint() {
  static const int v = [] { const char *e = getenv("GPMA_PR_HINT"); return e ? atoi(e) : 1; }();
  return v;
}

// GPMA_PR_SPLIT=1: the split push (lower-half REDs in the sweep, upper half through a spill list)
static bool pr_split() {
  const char *e = getenv("GPMA_PR_SPLIT");
  return e && atoi(e) != 0;
}

static uint32_t pr_passes(uint64_t ybytes) {
  (void)ybytes;
  uint64_t p = 1;
  if (const char *e = getenv("GPMA_PR_PASSES")) p = (uint64_t)atoi(e);
  return (uint32_t)std::max<uint64_t>(1, std::min<uint64_t>(p, 8));
}

template <typename T>
static gpma_status pagerank_t(gpma *g, T *x, int warm, T d, double tol, int max_iter, int *iters,
                              cudaStream_t s) {
  Scratch &X = g->an[AN_PR];
  ScanScope scan_scope_(X.scan);
  using A = typename PrAcc<T>::A;
  const uint64_t V = g->V;
  GP_CHECK(g, ensure(g, X.b[1], (V + 1) * sizeof(A), s));
  GP_CHECK(g, ensure(g, X.b[2], (V + 1) * sizeof(A), s));
  GP_CHECK(g, ensure(g, X.b[3], 8 * sizeof(double), s));   // acc[0..3], PrLoop at acc + 4, spill count at acc + 6
  const uint32_t *deg = g->deg;
  A *contrib = (A *)X.b[1].p, *y = (A *)X.b[2].p;
  double *acc = (double *)X.b[3].p;   // [0],[1] dangling ping-pong, [2] error, then the loop state
  PrLoop *lp = (PrLoop *)(acc + 4);
  const uint32_t passes = pr_passes(V * sizeof(A));
  // split push: a spill list for half of the slots (records past it are RED'd directly)
  const bool split = pr_split() && passes == 1;
  uint32_t *sd = nullptr;
  A *sc = nullptr;
  unsigned long long *scount = nullptr;
  uint64_t scap = 0;
  if (split) {                                     // a private run per push warp: cap records
    scap = g->cap + 32 * 4 * (uint64_t)SWEEP_BLOCKS * (TA / 32);
    GP_CHECK(g, ensure(g, X.stage[0], scap * 4 + 16, s));
    GP_CHECK(g, ensure(g, X.stage[1], scap * sizeof(A) + 16, s));
    GP_CHECK(g, ensure(g, X.misc, (uint64_t)SWEEP_BLOCKS * (TA / 32) * 8, s));
    sd = (uint32_t *)X.stage[0].p;
    sc = (A *)X.stage[1].p;
    scount = (unsigned long long *)X.misc.p;
  }
  GP_CHECK(g, fill_zero(g, acc, 4 * sizeof(double) + sizeof(PrLoop), s));
  GP_LAUNCH(g, k_pr_prep<T>, grid_for(V), TA, 0, s, x, deg, contrib, y, (uint32_t)V, warm ? 0 : 1, acc);
  // Iterations are queued in batches (2 first: a warm start rarely stops after one, then 1
  // at a time) and gated on the device, so the common 2-3 iteration call reads back once or
  // twice instead of once per iteration; the iterations that run are exactly those of the
  // per-iteration host loop.
  int queued = 0, cur = 0;
  uint32_t it = 0;
  while (queued < max_iter) {
    // (tol <= 0 never stops early -- the fixed-K parity mode, R20: queue every iteration at once)
    const int batch = tol <= 0.0 ? max_iter - queued : std::min(queued == 0 ? 2 : 1, max_iter - queued);
    for (int b = 0; b < batch; ++b, ++queued) {
      GP_LAUNCH(g, k_pr_iter_begin, 1, 32, 0, s, acc, cur ^ 1, lp);
      if (split) {
        GP_LAUNCH(g, (k_pr_push_split<A, 4>), SWEEP_BLOCKS, TA, 0, s, g->key, tmask_of(g), g->head, g->L, g->cap,
                  contrib, y, 0u, g->nr, (uint32_t)(V / 2), sd, sc, scount, &lp->done);
        GP_LAUNCH(g, k_pr_spill_apply<A>, grid_cap(), TA, 0, s, sd, sc, scount, g->cap,
                  (uint64_t)SWEEP_BLOCKS * (TA / 32), y, &lp->done);
      } else {
        // destination passes: random REDs run ~3x faster while their target fits in L2
        for (uint32_t q = 0; q < passes; ++q)
          GP_LAUNCH(g, (k_pr_push_win<A, 4>), SWEEP_BLOCKS, TA, 0, s, g->key, tmask_of(g), g->head, g->L,
                    g->cap, contrib, y, 0u, g->nr, (uint32_t)(V * q / passes), (uint32_t)(V * (q + 1) / passes),
                    pr_hint(), &lp->done);
      }
      GP_LAUNCH(g, k_pr_step<T>, grid_for(V), TA, 0, s, x, y, deg, contrib, (uint32_t)V, d, acc + cur,
                acc + (cur ^ 1), acc + 2, &lp->done);
      GP_LAUNCH(g, k_pr_iter_end, 1, 32, 0, s, acc, tol, lp);
      cur ^= 1;
    }
    GP_CHECK(g, readback(g, &X.ctrl_h->sum2, lp, sizeof(PrLoop), s));
    GP_CHECK(g, cudaStreamSynchronize(s));
    PrLoop h;
    memcpy(&h, &X.ctrl_h->sum2, sizeof h);
    it = h.iters;
    if (h.done) break;
  }
  if (iters) *iters = (int)it;
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// ---- distributed PageRank primitives (replicated x, exact fixed-point partial sums)
__global__ void k_prd_init(double *x, uint32_t V) {
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x)
    x[v] = 1.0 / (double)V;
}

// contributions of the owned rows; their dangling mass (fixed point) into y[V]
__global__ void k_prd_contrib(const double *__restrict__ x, const uint32_t *__restrict__ deg, uint32_t rb,
                              uint32_t nr, unsigned long long *__restrict__ contrib, unsigned long long *y,
                              uint32_t V) {
  unsigned long long dl = 0;
  for (uint64_t u = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; u < nr;
       u += (uint64_t)gridDim.x * blockDim.x) {
    const double xv = x[u + rb];
    const uint32_t dg = deg[u];
    contrib[u] = dg ? PrAcc<double>::enc(xv / (double)dg) : 0ull;
    if (!dg) dl += PrAcc<double>::enc(xv);
  }
  for (int o = 16; o; o >>= 1) dl += __shfl_xor_sync(0xffffffffu, dl, o);
  if ((threadIdx.x & 31) == 0 && dl) atomicAdd(y + V, dl);
}

// x' = (1-d)/V + d (y + D/V) for every vertex (replicated), err = ||x'-x||_1, y := 0
__global__ void k_prd_update(double *__restrict__ x, unsigned long long *__restrict__ y, uint32_t V, double d,
                             double *err) {
  __shared__ double red[32];
  const double base = (1.0 - d) / (double)V + d * (PrAcc<double>::dec(y[V]) / (double)V);
  double e = 0;
  for (uint64_t v = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; v < V;
       v += (uint64_t)gridDim.x * blockDim.x) {
    const double nx = base + d * PrAcc<double>::dec(y[v]);
    e += fabs(nx - x[v]);
    x[v] = nx;
    y[v] = 0;
  }
  double se = block_sum_d(e, red);
  if (threadIdx.x == 0 && se != 0) atomicAdd(err, se);
}

gpma_status pr_push(gpma *g, double *x, int init, uint64_t *y, cudaStream_t s) {
  Scratch &X = g->an[AN_PR];
  ScanScope scan_scope_(X.scan);
  GP_CHECK(g, ensure(g, X.b[1], ((uint64_t)g->nr + 1) * 8, s));
  unsigned long long *contrib = (unsigned long long *)X.b[1].p;
  unsigned long long *yy = (unsigned long long *)y;
  if (init) GP_LAUNCH(g, k_prd_init, grid_for(g->V), TA, 0, s, x, g->V);
  GP_LAUNCH(g, k_prd_contrib, grid_for(g->nr), TA, 0, s, x, g->deg, g->rb, g->nr, contrib, yy, g->V);
  const uint32_t passes = pr_passes((uint64_t)g->V * 8);
  for (uint32_t q = 0; q < passes; ++q)
    GP_LAUNCH(g, (k_pr_push_win<unsigned long long, 4>), SWEEP_BLOCKS, TA, 0, s, g->key, tmask_of(g),
              g->head, g->L, g->cap, contrib, yy, g->rb, g->nr, (uint32_t)((uint64_t)g->V * q / passes),
              (uint32_t)((uint64_t)g->V * (q + 1) / passes), pr_hint(), nullptr);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status pr_update(gpma *g, double *x, uint64_t *y, double d, double *err, cudaStream_t s) {
  Scratch &X = g->an[AN_PR];
  ScanScope scan_scope_(X.scan);
  double *e_d = reinterpret_cast<double *>(&X.ctrl_d->sum2);
  GP_CHECK(g, fill_zero(g, e_d, 8, s));
  GP_LAUNCH(g, k_prd_update, grid_for(g->V), TA, 0, s, x, (unsigned long long *)y, g->V, d, e_d);
  GP_CHECK(g, fill_zero(g, y + g->V, 8, s));
  GP_CHECK(g, readback(g, &X.ctrl_h->sum2, e_d, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  memcpy(err, &X.ctrl_h->sum2, 8);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// Owned-rows update after a reduce-scatter of y (multi-GPU): y_rows[0..nr) =
// the summed pushes into the owned vertices, y_rows[nr] = the total dangling mass.
// x'[rb+i] = (1-d)/V + d (y_rows[i] + y_rows[nr]/V); err = sum |x'-x| over the owned rows.
__global__ void k_prd_update_rows(double *__restrict__ x, const unsigned long long *__restrict__ yr, uint32_t rb,
                                  uint32_t nr, uint32_t V, double d, double *err) {
  __shared__ double red[32];
  const double base = (1.0 - d) / (double)V + d * (PrAcc<double>::dec(yr[nr]) / (double)V);
  double e = 0;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < nr; i += (uint64_t)gridDim.x * blockDim.x) {
    const double nx = base + d * PrAcc<double>::dec(yr[i]);
    e += fabs(nx - x[rb + i]);
    x[rb + i] = nx;
  }
  double se = block_sum_d(e, red);
  if (threadIdx.x == 0 && se != 0) atomicAdd(err, se);
}

gpma_status pr_update_rows_dev(gpma *g, double *x, const uint64_t *y_rows, double d, double *err_dev,
                              cudaStream_t s) {
  GP_LAUNCH(g, k_prd_update_rows, grid_for(g->nr), TA, 0, s, x, (const unsigned long long *)y_rows, g->rb, g->nr,
            g->V, d, err_dev);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status pr_update_rows(gpma *g, double *x, const uint64_t *y_rows, double d, double *err, cudaStream_t s) {
  Scratch &X = g->an[AN_PR];
  ScanScope scan_scope_(X.scan);
  double *e_d = reinterpret_cast<double *>(&X.ctrl_d->sum2);
  GP_CHECK(g, fill_zero(g, e_d, 8, s));
  GP_LAUNCH(g, k_prd_update_rows, grid_for(g->nr), TA, 0, s, x, (const unsigned long long *)y_rows, g->rb, g->nr,
            g->V, d, e_d);
  if (!err) return GPMA_OK;            // (err == nullptr: the error stays in the control block, device)
  GP_CHECK(g, readback(g, &X.ctrl_h->sum2, e_d, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  memcpy(err, &X.ctrl_h->sum2, 8);
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
// edges per leaf = live entries - guards (both maintained per leaf by every rewrite)
// Compaction sweep, 4 slots per thread.  A warp's 128 slots are leaf aligned and their
// edges land contiguously in the output from lbase[first leaf]: ranks come from a warp scan,
// the (col, val) pairs are staged in shared memory and stored as full coalesced lines.
__global__ void __launch_bounds__(TA) k_exp_write(const uint64_t *__restrict__ key,
                                                  const uint32_t *__restrict__ val,
                                                  const uint32_t *__restrict__ tmask, uint32_t L, uint64_t cap,
                                                  const uint64_t *__restrict__ lbase,
                                                  uint64_t *__restrict__ row_ptr, uint32_t *__restrict__ col,
                                                  uint32_t *__restrict__ cval, uint32_t rb) {
  __shared__ uint32_t s_col[TA / 32][128], s_val[TA / 32][128];
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const uint64_t n4 = cap / 4, n4r = (n4 + 31) & ~31ull;
  for (uint64_t t = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; t < n4r;
       t += (uint64_t)gridDim.x * blockDim.x) {
    Slot4 sl;
    uint32_t e = 0;
    if (t < n4) {
      load4(key, tmask, L, t * 4, sl);
#pragma unroll
      for (int j = 0; j < 4; ++j) e |= (edge4(sl, j) ? 1u : 0u) << j;
    } else {
      sl.k[0] = sl.k[1] = sl.k[2] = sl.k[3] = KEY_NONE;
    }
    const uint32_t c = __popc(e);
    uint32_t incl = c;
    for (int o = 1; o < 32; o <<= 1) {
      uint32_t y = __shfl_up_sync(0xffffffffu, incl, o);
      if (lane >= o) incl += y;
    }
    const uint32_t total = __shfl_sync(0xffffffffu, incl, 31);
    const uint64_t t0 = t - lane;                               // warp's first slot group
    const uint64_t wbase = t0 < n4 ? lbase[leaf_div(t0 * 4, L)] : 0;
    uint4 vv = make_uint4(0, 0, 0, 0);
    if (e) vv = __ldcs(reinterpret_cast<const uint4 *>(val + t * 4));
    const uint32_t vs[4] = {vv.x, vv.y, vv.z, vv.w};
    uint32_t r = incl - c;
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      if ((e >> j) & 1u) {
        s_col[w][r] = (uint32_t)sl.k[j];
        s_val[w][r] = vs[j];
        ++r;
      } else if (is_guard_key(sl.k[j])) {
        row_ptr[(sl.k[j] >> 32) - rb + 1] = wbase + r;
      }
    }
    __syncwarp();
    for (uint32_t i = lane; i < total; i += 32) {
      col[wbase + i] = s_col[w][i];
      cval[wbase + i] = s_val[w][i];
    }
    __syncwarp();
  }
}

// TMA-fed export (sweep.cuh): each stage holds a tile's keys, tombstone masks, values and the
// output offsets of its leaves (lbase); consumer warps rank the live edges of each 32-slot
// group with one ballot (a leaf's edges are contiguous in the output from lbase[leaf]) and
// store (col, val) as coalesced runs, guards setting row_ptr (R8).
constexpr int EX_T = 1024, EX_S = 3, EX_NC = 4, EX_PER_SM = 4;

struct ExportOp {
  static constexpr int SIDE = EX_T * 4 + (EX_T / 4) * 8;   // values + lbase of up to T/4 leaves
  static constexpr int EXTRA = 0;
  const uint32_t *val;
  const uint64_t *lbase;
  uint64_t *row_ptr;
  uint32_t *col, *cval;
  uint32_t rb, lgL;
  __device__ void init(void *) const {}
  __device__ void finish(void *) const {}
  __device__ uint32_t side_bytes(uint64_t, uint64_t, uint64_t, uint32_t *m) const {
    *m = 0;
    return EX_T * 4 + ((EX_T >> lgL) * 8 + 15) / 16 * 16;
  }
  __device__ void side_copy(uint64_t s0, uint32_t, void *dst, uint32_t bytes, uint64_t *bar) const {
    const uint64_t pol = tma::policy_evict_first();
    tma::bulk_g2s(dst, val + s0, EX_T * 4, bar, pol);
    tma::bulk_g2s((unsigned char *)dst + EX_T * 4, lbase + (s0 >> lgL), bytes - EX_T * 4, bar, pol);
  }
  template <int G>
  __device__ __forceinline__ void visit_warp(const uint64_t *sk, const uint32_t *stm, const void *side, uint32_t,
                                             uint64_t, uint32_t i0, uint32_t L, uint32_t lgL_, void *) const {
    const uint32_t *sv = (const uint32_t *)side;
    const uint64_t *lb = (const uint64_t *)((const unsigned char *)side + EX_T * 4);
    const uint32_t lane = threadIdx.x & 31;
    const uint32_t below = (1u << lane) - 1u;
    // lanes of the same leaf inside a 32-slot group (L <= 32, groups are leaf aligned)
    const uint32_t lmask = L >= 32 ? 0xffffffffu : (((1u << L) - 1u) << (lane & ~(L - 1u)));
    uint64_t k[G];
    uint32_t tw[G];
#pragma unroll
    for (int j = 0; j < G; ++j) {
      const uint32_t i = i0 + 32 * j;
      k[j] = sk[i];
      tw[j] = stm[i >> lgL_] >> (i & (L - 1));
    }
#pragma unroll
    for (int j = 0; j < G; ++j) {
      const uint32_t i = i0 + 32 * j;
      const bool e = live_key(k[j]) && !(tw[j] & 1u);
      const uint32_t bal = __ballot_sync(0xffffffffu, e);
      const uint64_t pos = lb[i >> lgL_] + __popc(bal & below & lmask);
      if (e) {
        col[pos] = (uint32_t)k[j];
        cval[pos] = sv[i];
      } else if (is_guard_key(k[j])) {
        row_ptr[(k[j] >> 32) - rb + 1] = pos;
      }
    }
  }
};

__global__ void __launch_bounds__(32 * (EX_NC + 1), 1)
    k_exp_tma(const uint64_t *__restrict__ key, const uint32_t *__restrict__ tmask, const uint64_t *__restrict__ head,
              uint64_t cap, uint32_t L, uint32_t lgL, ExportOp op) {
  sweep_run<EX_T, EX_S, EX_NC>(key, tmask, head, cap, L, lgL, op);
}

// guard-indexed or not, any store with whole leaf-aligned tiles (GPMA_EXPORT_TMA=0 disables)
static bool export_use_tma(const gpma *g) {
  static const int v = [] { const char *e = getenv("GPMA_EXPORT_TMA"); return e ? atoi(e) : 1; }();
  return v && g->cap >= (uint64_t)EX_T && g->cap % EX_T == 0 && g->L <= 32;
}

gpma_status export_csr(gpma *g, uint64_t *row_ptr, uint32_t *col, uint32_t *val, uint64_t cap_nnz,
                       uint64_t *nnz_out, cudaStream_t s) {
  Scratch &X = g->an[AN_EXPORT];
  ScanScope scan_scope_(X.scan);
  const uint64_t nl = g->cap / g->L;
  GP_CHECK(g, ensure(g, X.lpre, (nl + 1) * 8, s));
  uint64_t *lc = (uint64_t *)X.lpre.p;
  GP_CHECK(g, scan_leaf_edges(g, g->cnt, gcnt_of(g), lc, nl, s));   // live edges per leaf, scanned
  GP_CHECK(g, readback(g, &X.ctrl_h->sum, lc + nl, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  uint64_t nnz = X.ctrl_h->sum;
  if (nnz_out) *nnz_out = nnz;
  if (!col) return GPMA_OK;
  if (cap_nnz < nnz) {
    set_err(g, "export_csr: nnz_capacity too small");
    return GPMA_ERR_INVALID_ARG;
  }
  GP_CHECK(g, fill_zero(g, row_ptr, 8, s));
  if (export_use_tma(g)) {
    constexpr size_t sm = sweep_smem<EX_T, EX_S, ExportOp>();
    static std::atomic<bool> attr{false};
    if (!attr.load()) {
      GP_CHECK(g, cudaFuncSetAttribute(k_exp_tma, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sm));
      attr.store(true);
    }
    ExportOp op{g->val, lc, row_ptr, col, val, g->rb, ilog2(g->L)};
    GP_LAUNCH(g, k_exp_tma, num_sms() * EX_PER_SM, 32 * (EX_NC + 1), sm, s, g->key, tmask_of(g), g->head, g->cap,
              g->L, ilog2(g->L), op);
  } else {
    GP_LAUNCH(g, k_exp_write, grid_for(g->cap / 4, TA, SWEEP_BLOCKS), TA, 0, s, g->key, g->val, tmask_of(g), g->L,
              g->cap, lc, row_ptr, col, val, g->rb);
  }
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

}  // namespace gp
