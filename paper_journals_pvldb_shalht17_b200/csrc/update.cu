// update.cu -- GPMA+ batch update on sm_100a (Alg. 4).
//
// Per batch:  validate -> Sort(U) (l.2, radix sort of the integer keys)
//   -> unique (last occurrence wins, R10) -> BinarySearchLeafSegments (l.3, R9)
//   -> pre-pass: overwrite / revive / lazy-delete in place
//   -> level loop i = 0..h (l.4-15): UniqueSegments = RLE + ExclusiveScan (l.18-21),
//      CountSegment + CountUpdatesInSegment + density test (l.23-25, R5 integer
//      bounds), Merge + re-dispatch evenly (l.26-27, R7 proportional split), promote
//      the rest to the parent segment (l.12-15)
//   -> root resize (l.16-17, R14) -> locate-index (head) fix-up.
//
// Data layout in HBM: key u64[cap] and val u32[cap] as two
// SoA arrays (16-B vector moves on both), live count u32 per leaf, head u64 per leaf,
// row_offset u64[V+1].  Every window is rewritten out of place through a dense scratch
// list (gather -> scatter), so no kernel ever reads a slot another CTA writes.
#include <cuda_runtime.h>

#include <cooperative_groups.h>

#include <algorithm>
#include <chrono>
#include <cstdio>
#include <atomic>

#include "gpma_internal.cuh"

namespace gp {

constexpr int TB = 256;

__device__ __forceinline__ uint32_t locate_leaf(const uint64_t *__restrict__ head, uint32_t nleaves,
                                                uint64_t k) {
  // R9: upper_bound over the monotone head array, minus one, clamped at leaf 0.
  uint32_t lo = 0, hi = nleaves;
  while (lo < hi) {
    uint32_t mid = (lo + hi) >> 1;
    if (__ldg(head + mid) <= k) lo = mid + 1;
    else hi = mid;
  }
  return lo ? lo - 1 : 0;
}

// The same leaf through the row index (R8): key (u, v) lies between guard u-1 (slot
// row_offset[u], leaf a) and guard u (slot row_offset[u+1], leaf b), and head[a] <= guard u-1
// < key < head[b+1], so the upper bound over head[a..b] equals the global one (row 0: a = 0).
// A few dependent loads instead of log2(nleaves).  ro == nullptr (raw layouts without
// guards): the global search.
__device__ __forceinline__ uint32_t locate_leaf_rows(const uint64_t *__restrict__ head, uint32_t nleaves,
                                                     const uint64_t *__restrict__ ro, uint32_t rb, uint32_t L,
                                                     uint64_t k) {
  if (!ro) return locate_leaf(head, nleaves, k);
  const uint32_t u = (uint32_t)(k >> 32) - rb;
  const ulonglong2 r = make_ulonglong2(__ldg(ro + u), __ldg(ro + u + 1));
  const uint32_t a = (uint32_t)leaf_div(r.x, L);
  // the answer is >= a either way, so head[a] is never probed (monotone heads: if head[a] > k
  // every later head is too and the search ends at a)
  uint32_t lo = a + 1, hi = min((uint32_t)leaf_div(r.y, L) + 1, nleaves);
  while (lo < hi) {
    uint32_t mid = (lo + hi) >> 1;
    if (__ldg(head + mid) <= k) lo = mid + 1;
    else hi = mid;
  }
  return lo - 1;
}

// Slot of key k in leaf `base` (or -1): the occupied prefix of a leaf is sorted and the empty
// tail is KEY_NONE (> every key), so the scan stops at the first key >= k.  Eight slots are
// fetched per round with independent 16-B loads (one round trip instead of one per slot).
__device__ __forceinline__ int find_in_leaf(const uint64_t *__restrict__ key, uint64_t base, uint32_t L,
                                            uint64_t k) {
  for (uint32_t p0 = 0; p0 < L; p0 += 8) {
    ulonglong2 a[4];
#pragma unroll
    for (int j = 0; j < 4; ++j)
      a[j] = p0 + 2 * j < L ? __ldg(reinterpret_cast<const ulonglong2 *>(key + base + p0 + 2 * j))
                            : make_ulonglong2(KEY_NONE, KEY_NONE);
#pragma unroll
    for (int j = 0; j < 4; ++j) {
      if (a[j].x == k) return (int)(p0 + 2 * j);
      if (a[j].x > k) return -1;
      if (a[j].y == k) return (int)(p0 + 2 * j + 1);
      if (a[j].y > k) return -1;
    }
  }
  return -1;
}

// ------------------------------------------------------------------ validate
__global__ void k_validate(const uint64_t *__restrict__ keys, const uint32_t *__restrict__ vals,
                           uint64_t n, uint32_t V, uint32_t rb, uint32_t nr, int check_vals, Ctrl *c) {
  uint32_t e = 0;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t k = keys[i];
    uint32_t src = (uint32_t)(k >> 32), dst = (uint32_t)k;
    if (dst == COL_GUARD) e |= 2u;
    if (check_vals && vals[i] == VAL_TOMB) e |= 2u;
    if (src - rb >= nr || dst >= V) e |= 1u;    // src outside the owned rows (wraps)
  }
  e = __reduce_or_sync(0xffffffffu, e);
  if (e && (threadIdx.x & 31) == 0) atomicOr(&c->err, e);
}

// ------------------------------------------------------------------ pre-pass
// One thread per sorted update; only the last copy of a key acts (R10).
__global__ void k_prepass(const uint64_t *__restrict__ sk, const uint32_t *__restrict__ sv,
                          uint64_t n, const uint64_t *__restrict__ key, uint32_t *__restrict__ val,
                          uint32_t *__restrict__ cnt, const uint64_t *__restrict__ head,
                          uint32_t nleaves, uint32_t L, int op, int mode,
                          uint32_t *__restrict__ keep, uint32_t *__restrict__ tgt, Ctrl *c,
                          uint32_t *__restrict__ tmask, uint32_t *__restrict__ deg, uint32_t rb,
                          const uint64_t *__restrict__ ro) {
  if (c->err) return;                                // rejected batch: nothing may change
  uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
  uint32_t uniq = 0;
  if (i < n) {
    uint64_t k = sk[i];
    uint32_t kp = 0, t = 0;
    if (i + 1 == n || sk[i + 1] != k) {
      uniq = 1;
      t = locate_leaf_rows(head, nleaves, ro, rb, L, k);
      const uint64_t base = (uint64_t)t * L;
      const int hp = find_in_leaf(key, base, L, k);
      const uint64_t hit = hp >= 0 ? base + (uint64_t)hp : KEY_NONE;
      const uint32_t src = (uint32_t)(k >> 32) - rb;   // local row
      const uint32_t bit = hit != KEY_NONE ? 1u << (uint32_t)(hit - base) : 0u;
      if (op == GPMA_INSERT) {
        if (hit != KEY_NONE) {                      // overwrite (R11) or revive (R12)
          uint32_t old = val[hit];
          val[hit] = sv[i];
          if (old == VAL_TOMB) {
            atomicAdd(&cnt[t], 1u);
            atomicAnd(&tmask[t], ~bit);
            atomicAdd(&deg[src], 1u);
          }
        } else {
          kp = 1;                                   // new key: inserted by the level loop
          atomicAdd(&deg[src], 1u);
        }
      } else if (mode == GPMA_DELETE_LAZY) {        // mark, no maintenance
        if (hit != KEY_NONE && val[hit] != VAL_TOMB) {
          val[hit] = VAL_TOMB;
          atomicSub(&cnt[t], 1u);
          atomicOr(&tmask[t], bit);
          atomicSub(&deg[src], 1u);
        }
      } else {                                      // strict delete: live keys only
        if (hit != KEY_NONE && val[hit] != VAL_TOMB) {
          kp = 1;
          atomicSub(&deg[src], 1u);
        }
      }
    }
    keep[i] = kp;
    tgt[i] = t;
  }
  uint32_t u = __reduce_add_sync(0xffffffffu, uniq);
  if ((threadIdx.x & 31) == 0 && u) atomicAdd((unsigned long long *)&c->nunique, (unsigned long long)u);
}

// Lazy deletion (R12) needs no order: every key of the batch is located and
// its live slot marked in place.  Duplicates race on the same slot; the CAS on the value
// lets exactly one of them account the deletion (live count, tombstone bit, out-degree).
__global__ void k_lazy_delete(const uint64_t *__restrict__ keys, uint64_t n, const uint64_t *__restrict__ key,
                              uint32_t *val, uint32_t *__restrict__ cnt, const uint64_t *__restrict__ head,
                              uint32_t nleaves, uint32_t L, uint32_t *__restrict__ tmask,
                              uint32_t *__restrict__ deg, uint32_t rb, const Ctrl *c,
                              const uint64_t *__restrict__ ro) {
  if (c->err) return;                                // rejected batch: nothing may change
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    const uint64_t k = keys[i];
    const uint32_t t = locate_leaf_rows(head, nleaves, ro, rb, L, k);
    const uint64_t base = (uint64_t)t * L;
    const int p = find_in_leaf(key, base, L, k);
    if (p < 0) continue;
    uint32_t old = val[base + p];
    while (old != VAL_TOMB) {
      const uint32_t seen = atomicCAS(&val[base + p], old, VAL_TOMB);
      if (seen == old) {
        atomicSub(&cnt[t], 1u);
        atomicOr(&tmask[t], 1u << p);
        atomicSub(&deg[(uint32_t)(k >> 32) - rb], 1u);
        break;
      }
      old = seen;
    }
  }
}

// Lazy deletion on the SORTED batch (R12): duplicates are adjacent, so only the
// last copy of a key acts and no CAS is needed; sorted keys walk the rows (row_offset, deg) and
// the leaves in address order, so the sectors a warp touches are shared across its lanes instead
// of one random 32-B sector per access.  The live count / tombstone bit of a leaf and the
// out-degree of a row are updated once per warp-run of equal leaf / row (__match_any_sync).
__global__ void __launch_bounds__(256) k_del_mark(const uint64_t *__restrict__ sk, uint64_t n,
                                                  const uint64_t *__restrict__ key, uint32_t *__restrict__ val,
                                                  uint32_t *__restrict__ cnt, const uint64_t *__restrict__ head,
                                                  uint32_t nleaves, uint32_t L, uint32_t *__restrict__ tmask,
                                                  uint32_t *__restrict__ deg, uint32_t rb, Ctrl *c,
                                                  const uint64_t *__restrict__ ro) {
  if (c->err) return;                                // rejected batch: nothing may change
  const int lane = threadIdx.x & 31;
  const uint64_t nr = (n + 31) & ~31ull;             // whole warps: the match below is full-mask
  uint32_t marked = 0;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < nr;
       i += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t k = KEY_NONE;
    uint32_t t = 0xFFFFFFFFu, bit = 0;
    if (i < n) {
      k = sk[i];
      // every key is located (duplicates too), so the targets of a warp are non-decreasing
      // and lanes of one leaf form one contiguous run
      t = locate_leaf_rows(head, nleaves, ro, rb, L, k);
      if (i + 1 == n || sk[i + 1] != k) {            // the last copy of a key acts (R10)
        const uint64_t base = (uint64_t)t * L;
        const int p = find_in_leaf(key, base, L, k);
        if (p >= 0 && val[base + p] != VAL_TOMB) {
          val[base + p] = VAL_TOMB;
          bit = 1u << p;
        }
      }
    }
    const bool hit = bit != 0;
    // per leaf run: one count update and one OR of the tombstone bits (segmented scan)
    const uint32_t peers = __match_any_sync(0xffffffffu, t);
    const uint32_t hitm = __ballot_sync(0xffffffffu, hit);
    const int first = __ffs(peers) - 1, last = 31 - __clz(peers);
    uint32_t orb = bit;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, orb, o);
      if (lane - o >= first) orb |= y;
    }
    const uint32_t m = __popc(peers & hitm);
    if (lane == last && m) {
      atomicSub(&cnt[t], m);
      atomicOr(&tmask[t], orb);
    }
    // per row: one out-degree update
    const uint32_t src = hit ? (uint32_t)(k >> 32) - rb : 0xFFFFFFFFu;
    const uint32_t rp = __match_any_sync(0xffffffffu, src);
    if (hit && lane == __ffs(rp) - 1) atomicSub(&deg[src], (uint32_t)__popc(rp));
    marked += lane == 0 ? __popc(hitm) : 0;
  }
  if (lane == 0 && marked) atomicAdd((unsigned long long *)&c->sum, (unsigned long long)marked);
}

// Target leaf of every sorted update (Alg. 4 l.3 BinarySearchLeafSegments, R9) and the head
// flags of the leaf groups (UniqueSegments at level 0, l.18-21): a group starts where the
// target changes.  The previous key's target comes from the neighbouring thread (shared
// memory); only the first thread of a block searches it again.
constexpr int LOC_T = 256;
__global__ void __launch_bounds__(LOC_T) k_locate(const uint64_t *__restrict__ sk, uint64_t n,
                                                  const uint64_t *__restrict__ head, uint32_t nleaves, uint32_t L,
                                                  uint32_t rb, const uint64_t *__restrict__ ro,
                                                  uint32_t *__restrict__ tgt, uint32_t *__restrict__ hf,
                                                  const Ctrl *c) {
  __shared__ uint32_t st[LOC_T];
  if (c->err) return;
  const uint64_t stride = (uint64_t)gridDim.x * LOC_T;
  for (uint64_t b = blockIdx.x * (uint64_t)LOC_T; b < n; b += stride) {   // block-uniform
    const uint64_t i = b + threadIdx.x;
    uint32_t t = 0, tp = 0xFFFFFFFFu;
    if (i < n) {
      t = locate_leaf_rows(head, nleaves, ro, rb, L, sk[i]);
      tgt[i] = t;
      if (threadIdx.x == 0 && i > 0) tp = locate_leaf_rows(head, nleaves, ro, rb, L, sk[i - 1]);
    }
    st[threadIdx.x] = t;
    __syncthreads();
    if (i < n) {
      if (threadIdx.x) tp = st[threadIdx.x - 1];
      hf[i] = (i == 0 || tp != t) ? 1u : 0u;
    }
    __syncthreads();
  }
}

__global__ void k_gstart(const uint32_t *__restrict__ hf, const uint32_t *__restrict__ gid, uint64_t n,
                         uint32_t *__restrict__ gstart, const Ctrl *c) {
  if (c->err) return;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    if (hf[i]) gstart[gid[i]] = (uint32_t)i;
    if (i == 0) gstart[gid[n]] = (uint32_t)n;
  }
}

// Fused insert pre-pass + level 0 (Alg. 4 l.3-15 at the leaves, R10-R12): one
// L-lane sub-warp per leaf group of the sorted batch (group starts from k_gstart), the leaf
// read ONCE.  Lane l holds slot l.  The group's updates are taken L at a time: the last copy
// of a key acts (R10); its position among the occupied slots comes from a shuffle binary
// search, a hit overwrites the value in place (R11) or revives a tombstone (R12), the new keys
// are collected (shared memory) for the merge.  Density test n_live + u_new <= max_0 (R5); on
// success the leaf is merged in registers and re-dispatched left-packed (R7 for one leaf),
// otherwise the hits are written in place and the new keys stay pending for level 1
// (keep[j] = 1).  Out-degrees count every new key and every revive once per row run.
constexpr int IL_T = 256;
__global__ void __launch_bounds__(IL_T) k_ins_leaf(const uint64_t *__restrict__ sk, const uint32_t *__restrict__ sv,
                                                   const uint32_t *__restrict__ tgt, const uint32_t *__restrict__ gstart,
                                                   const uint32_t *__restrict__ ng_dev, uint64_t *key, uint32_t *val,
                                                   uint32_t *__restrict__ cnt, uint32_t *__restrict__ tmask,
                                                   uint64_t *__restrict__ head, uint64_t *__restrict__ row_offset,
                                                   uint32_t *__restrict__ deg, uint32_t rb, uint32_t L, uint32_t bound,
                                                   uint32_t *__restrict__ keep, uint2 *__restrict__ dirty, Ctrl *c) {
  __shared__ uint64_t s_nk[IL_T];                    // new keys of each sub-warp (<= L kept)
  __shared__ uint32_t s_nv[IL_T], s_nj[IL_T];
  __shared__ uint32_t s_hv[IL_T];                    // value a hit writes into slot l
  if (c->err) return;
  const uint32_t ng = *ng_dev;
  const int lane = threadIdx.x & 31;
  const uint32_t nsub = 32 / L, sub = lane / L, sl = lane % L;
  const uint32_t sub0 = sub * L;                     // first lane of my sub-warp
  const uint32_t lmask = L == 32 ? 0xffffffffu : (1u << L) - 1u;
  const uint32_t below_me = (1u << sl) - 1u;
  const int wb = threadIdx.x & ~31;                  // this warp's first entry in the smem arrays
  const uint32_t lgL = __ffs(L) - 1;
  const uint64_t nwarps = (uint64_t)gridDim.x * (blockDim.x / 32);
  uint32_t accepted = 0, news = 0, effs = 0;
  for (uint64_t gw = ((blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32) * nsub; gw < ng;
       gw += nwarps * nsub) {                        // warp-uniform trip count
    const uint64_t gi = gw + sub;
    const bool have = gi < ng;
    uint32_t j0 = 0, j1 = 0, t = 0;
    if (have) {
      j0 = gstart[gi];
      j1 = gstart[gi + 1];
      t = tgt[j0];
    }
    const uint64_t lb = (uint64_t)t * L;
    uint64_t ks = KEY_NONE;
    uint32_t vs = 0;
    if (have) {
      ks = key[lb + sl];
      vs = val[lb + sl];
    }
    const bool occ = ks != KEY_NONE;
    const uint32_t obits = (__ballot_sync(0xffffffffu, occ) >> sub0) & lmask;
    const uint32_t nocc = __popc(obits);               // occupied prefix (sorted, left-packed)
    const bool was_tomb = occ && vs == VAL_TOMB;
    uint32_t hitbits = 0, nnew = 0;
    const uint32_t u = j1 - j0;
    const uint32_t umax = __reduce_max_sync(0xffffffffu, u);
    for (uint32_t c0 = 0; c0 < umax; c0 += L) {        // the group's updates, L at a time
      const uint32_t j = j0 + c0 + sl;
      const bool inb = have && c0 + sl < u;
      uint64_t uk = KEY_NONE;
      uint32_t uv = 0;
      bool eff = false;
      if (inb) {
        uk = sk[j];
        uv = sv[j];
        eff = c0 + sl + 1 == u || sk[j + 1] != uk;
      }
      // pos = #occupied slots with key < uk (shuffle binary search over the sorted prefix)
      uint32_t lo = 0, hi = nocc;
      for (uint32_t step = L; step; step >>= 1) {      // log2(L) + 1 rounds, uniform
        const uint32_t mid = (lo + hi) >> 1;
        const uint64_t km = __shfl_sync(0xffffffffu, ks, (int)(sub0 + (mid < L ? mid : L - 1)));
        if (lo < hi) {
          if (km < uk) lo = mid + 1;
          else hi = mid;
        }
      }
      const uint32_t pos = lo;
      const uint64_t kp = __shfl_sync(0xffffffffu, ks, (int)(sub0 + (pos < L ? pos : L - 1)));
      const uint32_t vp = __shfl_sync(0xffffffffu, vs, (int)(sub0 + (pos < L ? pos : L - 1)));
      const bool hit = eff && pos < nocc && kp == uk;
      if (hit) s_hv[wb + sub0 + pos] = uv;
      const uint32_t hb = __reduce_or_sync(0xffffffffu, hit ? 1u << (sub0 + pos) : 0u);
      hitbits |= (hb >> sub0) & lmask;
      const bool isnew = eff && !hit;
      const uint32_t nb = (__ballot_sync(0xffffffffu, isnew) >> sub0) & lmask;
      if (isnew) {
        const uint32_t q = nnew + __popc(nb & below_me);
        if (q < L) {
          s_nk[wb + sub0 + q] = uk;
          s_nv[wb + sub0 + q] = uv;
          s_nj[wb + sub0 + q] = j;
        }
        keep[j] = 1u;                                   // pending unless the leaf takes it
      } else if (inb) {
        keep[j] = 0u;
      }
      nnew += __popc(nb);
      effs += eff;
      // out-degree: every new key and every revived tombstone, once per row run
      const bool dinc = isnew || (hit && vp == VAL_TOMB);
      const uint32_t src = dinc ? (uint32_t)(uk >> 32) - rb : 0xFFFFFFFFu;
      const uint32_t rp = __match_any_sync(0xffffffffu, src);
      if (dinc && lane == __ffs(rp) - 1) atomicAdd(&deg[src], (uint32_t)__popc(rp));
    }
    __syncwarp();
    news += sl == 0 ? nnew : 0;
    const bool myhit = (hitbits >> sl) & 1u;
    if (myhit) vs = s_hv[wb + lane];                    // overwrite (R11) / revive (R12)
    const bool live = occ && vs != VAL_TOMB;
    const uint32_t lbits = (__ballot_sync(0xffffffffu, live) >> sub0) & lmask;
    const uint32_t n = __popc(lbits);
    const bool ok = have && nnew > 0 && nnew <= bound && n + nnew <= bound;
    // merge: a live entry's rank = its live rank + the new keys below it; a new key's rank =
    // its index + the live entries below it (one round per new key, nnew <= max_0)
    uint64_t uk = KEY_NONE;
    uint32_t uv = 0;
    if (ok && sl < nnew) {
      uk = s_nk[wb + lane];
      uv = s_nv[wb + lane];
    }
    uint32_t below_u = 0, below_l = 0;
    const uint32_t rmax = __reduce_max_sync(0xffffffffu, ok ? nnew : 0u);
    for (uint32_t i = 0; i < rmax; ++i) {
      const bool vi = ok && i < nnew;
      const uint64_t ui = __shfl_sync(0xffffffffu, uk, (int)(sub0 + (i < L ? i : 0)));
      below_u += vi && ui < ks;
      const uint32_t bl = __popc((__ballot_sync(0xffffffffu, vi && live && ks < ui) >> sub0) & lmask);
      if (sl == i) below_l = bl;
    }
    const uint32_t N = n + nnew;
    const uint32_t lpos = __popc(lbits & below_me) + below_u;
    const uint32_t upos = sl + below_l;
    const bool l0 = live && lpos == 0;
    const bool u0 = ok && sl < nnew && upos == 0;
    const uint32_t b0 = (__ballot_sync(0xffffffffu, l0 || u0) >> sub0) & lmask;
    const uint64_t h_new = __shfl_sync(0xffffffffu, l0 ? ks : uk, (int)(sub0 + (b0 ? __ffs(b0) - 1 : 0)));
    const uint64_t h_old = __shfl_sync(0xffffffffu, ks, (int)sub0);
    __syncwarp();
    if (ok) {
      if (live) {
        key[lb + lpos] = ks;
        val[lb + lpos] = vs;
        if (is_guard_key(ks)) row_offset[(ks >> 32) - rb + 1] = lb + lpos;
      }
      if (sl < nnew) {
        key[lb + upos] = uk;
        val[lb + upos] = uv;
        keep[s_nj[wb + lane]] = 0u;
      }
    } else if (myhit) {
      val[lb + sl] = vs;                                // in place: the leaf is not rewritten
    }
    __syncwarp();
    if (ok && sl >= N) {
      key[lb + sl] = KEY_NONE;
      val[lb + sl] = 0;
    }
    const uint32_t revived = hitbits & ((__ballot_sync(0xffffffffu, was_tomb) >> sub0) & lmask);
    if (have && sl == 0) {
      if (ok) {
        cnt[t] = N;
        tmask[t] = 0u;                                  // tombstones are dropped by the rewrite
        if (h_new != h_old && N) {
          head[t] = h_new;
          // empty leaves to the left carry this head (R9): leave them to the final fix-up
          if (t > 0 && key[lb - L] == KEY_NONE) {
            const uint64_t d = atomicAdd((unsigned long long *)&c->ndirty, 1ull);
            dirty[d] = make_uint2(t, 1u);
          }
        }
        ++accepted;
      } else if (revived) {
        cnt[t] += __popc(revived);
        tmask[t] &= ~revived;
      }
    }
    __syncwarp();
  }
  accepted = __reduce_add_sync(0xffffffffu, accepted);
  news = __reduce_add_sync(0xffffffffu, news);
  effs = __reduce_add_sync(0xffffffffu, effs);
  if (lane == 0) {
    if (accepted) atomicAdd((unsigned long long *)&c->windows_rewritten, (unsigned long long)accepted);
    if (news) atomicAdd((unsigned long long *)&c->sum, (unsigned long long)news);
    if (effs) atomicAdd((unsigned long long *)&c->nunique, (unsigned long long)effs);
  }
}

// Fused insert pre-pass + level 0, ONE THREAD PER LEAF GROUP (the common shape: a 2^20-key
// batch over 2^24 leaves gives ~1 update per touched leaf).  The thread holds its leaf in
// registers (L keys + L values, 16-B vector loads and stores, statically indexed), so a group
// costs a handful of instructions per warp instead of a sub-warp's shuffle rounds:
//   pass 1 over the group's updates (sorted; the last copy of a key acts, R10): a key equal to
//     an occupied slot overwrites its value (R11) or revives a tombstone (R12); the others are new;
//   density test n_live + u_new <= max_0 (Alg. 4 l.25, R5);
//   accepted: tombstones dropped (left-pack by a static select network), the new keys inserted
//     in key order (one static shift each), the leaf written back left-packed (R7 for a single
//     leaf), count / tombstone mask / head / guard row offsets maintained;
//   rejected: the hits written in place, the new keys flagged pending for level 1 (keep[j] = 1).
// Out-degrees: +1 per new key and per revive (one atomic per row run of the thread).
template <int L>
__global__ void __launch_bounds__(256) k_ins_leaf_t(const uint64_t *__restrict__ sk, const uint32_t *__restrict__ sv,
                                                    const uint32_t *__restrict__ tgt, const uint32_t *__restrict__ gstart,
                                                    const uint32_t *__restrict__ ng_dev, uint64_t *key, uint32_t *val,
                                                    uint32_t *__restrict__ cnt, uint32_t *__restrict__ tmask,
                                                    uint64_t *__restrict__ head, uint64_t *__restrict__ row_offset,
                                                    uint32_t *__restrict__ deg, uint32_t rb, uint32_t bound,
                                                    uint32_t *__restrict__ keep, uint2 *__restrict__ dirty, Ctrl *c) {
  if (c->err) return;
  const uint32_t ng = *ng_dev;
  uint32_t accepted = 0, news = 0, effs = 0;
  for (uint64_t gi = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; gi < ng; gi += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t j0 = gstart[gi], j1 = gstart[gi + 1];
    const uint32_t t = tgt[j0];
    const uint64_t lb = (uint64_t)t * L;
    uint64_t K[L];
    uint32_t Vv[L];
#pragma unroll
    for (int p = 0; p < L; p += 2) {
      const ulonglong2 kk = *reinterpret_cast<const ulonglong2 *>(key + lb + p);
      K[p] = kk.x;
      K[p + 1] = kk.y;
    }
#pragma unroll
    for (int p = 0; p < L; p += 4) {
      const uint4 vv = *reinterpret_cast<const uint4 *>(val + lb + p);
      Vv[p] = vv.x;
      Vv[p + 1] = vv.y;
      Vv[p + 2] = vv.z;
      Vv[p + 3] = vv.w;
    }
    uint32_t occ = 0, tomb = 0;
#pragma unroll
    for (int p = 0; p < L; ++p) {
      occ |= (K[p] != KEY_NONE ? 1u : 0u) << p;
      tomb |= (K[p] != KEY_NONE && Vv[p] == VAL_TOMB ? 1u : 0u) << p;
    }
    // pass 1: hits (overwrite / revive) and the count of new keys
    uint32_t hitm = 0, revm = 0, nnew = 0;
    uint32_t dsrc = 0xFFFFFFFFu, dcnt = 0;             // out-degree run of this thread
    for (uint32_t j = j0; j < j1; ++j) {
      const uint64_t uk = sk[j];
      if (j + 1 < j1 && sk[j + 1] == uk) continue;     // not the last copy (R10)
      ++effs;
      const uint32_t uv = sv[j];
      uint32_t h = 0;
#pragma unroll
      for (int p = 0; p < L; ++p)
        if (K[p] == uk) {
          h = 1u << p;
          Vv[p] = uv;
        }
      const bool inc = !h || (h & tomb);               // a new key or a revived tombstone
      hitm |= h;
      revm |= h & tomb;
      nnew += h ? 0u : 1u;
      if (inc) {
        const uint32_t src = (uint32_t)(uk >> 32) - rb;
        if (src != dsrc) {
          if (dcnt) atomicAdd(&deg[dsrc], dcnt);
          dsrc = src;
          dcnt = 0;
        }
        ++dcnt;
      }
    }
    if (dcnt) atomicAdd(&deg[dsrc], dcnt);
    const uint32_t live = occ & ~(tomb & ~revm);
    const uint32_t n = __popc(live);
    const bool ok = nnew > 0 && nnew <= bound && n + nnew <= bound;
    news += nnew;
    if (ok) {
      const uint64_t h_old = K[0];
      if (live != ((1u << n) - 1u)) {                   // drop the tombstones (highest first: the
        uint32_t dead = occ & ~live;                    // lower positions stay valid), left-packing
        while (dead) {
          const int pd = 31 - __clz(dead);
#pragma unroll
          for (int p = 0; p < L - 1; ++p)
            if (p >= pd) {
              K[p] = K[p + 1];
              Vv[p] = Vv[p + 1];
            }
          K[L - 1] = KEY_NONE;
          Vv[L - 1] = 0;
          dead &= ~(1u << pd);
        }
      }
      uint32_t N = n;
      for (uint32_t j = j0; j < j1; ++j) {
        const uint64_t uk = sk[j];
        if (j + 1 < j1 && sk[j + 1] == uk) continue;
        bool present = false;
        uint32_t pos = 0;
#pragma unroll
        for (int p = 0; p < L; ++p) {
          present |= (p < (int)N) && K[p] == uk;
          pos += (p < (int)N) && K[p] < uk;
        }
        if (present) continue;                         // a hit (already applied)
        const uint32_t uv = sv[j];
#pragma unroll
        for (int p = L - 1; p > 0; --p)
          if ((uint32_t)p > pos) {
            K[p] = K[p - 1];
            Vv[p] = Vv[p - 1];
          }
#pragma unroll
        for (int p = 0; p < L; ++p)
          if ((uint32_t)p == pos) {
            K[p] = uk;
            Vv[p] = uv;
          }
        ++N;
      }
#pragma unroll
      for (int p = 0; p < L; ++p)
        if ((uint32_t)p >= N) {
          K[p] = KEY_NONE;
          Vv[p] = 0;
        }
#pragma unroll
      for (int p = 0; p < L; p += 2)
        *reinterpret_cast<ulonglong2 *>(key + lb + p) = make_ulonglong2(K[p], K[p + 1]);
#pragma unroll
      for (int p = 0; p < L; p += 4)
        *reinterpret_cast<uint4 *>(val + lb + p) = make_uint4(Vv[p], Vv[p + 1], Vv[p + 2], Vv[p + 3]);
#pragma unroll
      for (int p = 0; p < L; ++p)
        if (is_guard_key(K[p])) row_offset[(K[p] >> 32) - rb + 1] = lb + p;   // R8: guards that moved
      cnt[t] = N;
      tmask[t] = 0u;                                   // tombstones are dropped by the rewrite
      if (K[0] != h_old) {
        head[t] = K[0];
        // empty leaves to the left carry this head (R9): leave them to the final fix-up
        if (t > 0 && key[lb - L] == KEY_NONE) {
          const uint64_t d = atomicAdd((unsigned long long *)&c->ndirty, 1ull);
          dirty[d] = make_uint2(t, 1u);
        }
      }
      for (uint32_t j = j0; j < j1; ++j) keep[j] = 0u;
      ++accepted;
    } else {
      // rejected (or nothing new): the hits in place, the new keys pending for level 1
      if (hitm) {
#pragma unroll
        for (int p = 0; p < L; ++p)
          if ((hitm >> p) & 1u) val[lb + p] = Vv[p];
      }
      if (revm) {
        cnt[t] += __popc(revm);
        tmask[t] &= ~revm;
      }
      for (uint32_t j = j0; j < j1; ++j) {
        const uint64_t uk = sk[j];
        bool pend = false;
        if (!(j + 1 < j1 && sk[j + 1] == uk)) {
          bool present = false;
#pragma unroll
          for (int p = 0; p < L; ++p) present |= ((occ >> p) & 1u) && K[p] == uk;
          pend = !present;
        }
        keep[j] = pend ? 1u : 0u;
      }
    }
  }
  accepted = __reduce_add_sync(0xffffffffu, accepted);
  news = __reduce_add_sync(0xffffffffu, news);
  effs = __reduce_add_sync(0xffffffffu, effs);
  if ((threadIdx.x & 31) == 0) {
    if (accepted) atomicAdd((unsigned long long *)&c->windows_rewritten, (unsigned long long)accepted);
    if (news) atomicAdd((unsigned long long *)&c->sum, (unsigned long long)news);
    if (effs) atomicAdd((unsigned long long *)&c->nunique, (unsigned long long)effs);
  }
}

// ---- leaf-keyed insert prefix (the default): Alg. 4 l.2-3 sort the batch so that the updates
// of one segment are contiguous (UniqueSegments, l.18-21).  Level 0 needs exactly that grouping,
// and R9 targets are monotone in the key, so the batch is located FIRST (unsorted, one thread per
// key) and stably sorted by target leaf: ceil(log2 leaves / 8) radix passes of (leaf, arrival
// index) instead of 2*ceil(log2 V / 8) passes of (key, value).  Inside a group the arrival order
// is kept, so "the last occurrence wins" (R10) is decided in the group kernel; the key order
// inside a leaf is rebuilt by the merge; the few updates the leaves reject are sorted by key
// before the level loop (which works on key-sorted pending lists, l.12-15).
__global__ void k_locate_u(const uint64_t *__restrict__ ik, uint64_t n, const uint64_t *__restrict__ head,
                           uint32_t nleaves, uint32_t L, uint32_t rb, const uint64_t *__restrict__ ro,
                           uint64_t *__restrict__ tk, uint32_t *__restrict__ tix, const Ctrl *c) {
  if (c->err) return;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    tk[i] = locate_leaf_rows(head, nleaves, ro, rb, L, ik[i]);
    tix[i] = (uint32_t)i;
  }
}

__global__ void k_gflags(const uint64_t *__restrict__ tk, uint64_t n, uint32_t *__restrict__ hf, const Ctrl *c) {
  if (c->err) return;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x)
    hf[i] = (i == 0 || tk[i] != tk[i - 1]) ? 1u : 0u;
}

// Group starts of the leaf-sorted batch in ONE pass (UniqueSegments, Alg. 4 l.18-21, for level
// 0): a decoupled look-back compaction of the head flags (tk[j] != tk[j-1]) -- gstart[g] = first
// index of group g, gstart[ng] = n, *ng_out = ng.  Replaces flags + scan + scatter (three passes
// over the batch and two launches more).  status[0] is the tile counter, status[1 + t] tile t's
// (flag:2 | count) word; the caller zeroes both.
constexpr int GS_T = 1024, GS_I = 16, GS_TILE = GS_T * GS_I;   // 16K-item tiles: fewer look-back rounds
// (generic: items tk[i] >> shift of type K; hf / widx optional per-item outputs -- the head flag
// and the exclusive head count, as UniqueSegments' flags + scan; widx[n] = the group count)
template <typename K>
__global__ void __launch_bounds__(GS_T) k_group_starts(const K *__restrict__ tk, uint64_t n, uint32_t shift,
                                                       uint32_t *__restrict__ gstart, uint32_t *__restrict__ ng_out,
                                                       uint32_t *__restrict__ hf, uint32_t *__restrict__ widx,
                                                       unsigned long long *status, const Ctrl *c) {
  __shared__ uint32_t s_tile, s_prefix;
  __shared__ uint32_t wcnt[GS_T / 32];
  if (c->err) return;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  if (threadIdx.x == 0) s_tile = (uint32_t)atomicAdd(status, 1ull);
  __syncthreads();
  const uint32_t tile = s_tile;
  volatile unsigned long long *st = status + 1;
  const uint64_t base = (uint64_t)tile * GS_TILE + (uint64_t)w * (32 * GS_I);
  // all of the warp's loads first (the flag's left neighbour comes from the next lane down,
  // or from the previous row's lane 31; one extra load per warp)
  uint64_t a[GS_I];
#pragma unroll
  for (int j = 0; j < GS_I; ++j) {
    const uint64_t i = base + j * 32 + lane;
    a[j] = i < n ? (uint64_t)(tk[i] >> shift) : 0ull;
  }
  const uint64_t before = (lane == 0 && base > 0 && base <= n) ? (uint64_t)(tk[base - 1] >> shift) : 0ull;
  uint32_t bal[GS_I];
  uint32_t mine = 0;
  uint64_t carry = __shfl_sync(0xffffffffu, before, 0);
#pragma unroll
  for (int j = 0; j < GS_I; ++j) {
    const uint64_t i = base + j * 32 + lane;
    uint64_t left = __shfl_up_sync(0xffffffffu, a[j], 1);
    if (lane == 0) left = carry;
    carry = __shfl_sync(0xffffffffu, a[j], 31);
    const bool f = i < n && (i == 0 || a[j] != left);
    bal[j] = __ballot_sync(0xffffffffu, f);
    mine += __popc(bal[j]);
  }
  if (lane == 0) wcnt[w] = mine;
  __syncthreads();
  if (w == 0) {
    const uint32_t wc = lane < GS_T / 32 ? wcnt[lane] : 0u;
    uint32_t x = wc;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
      if (lane >= o) x += y;
    }
    const uint32_t agg = __shfl_sync(0xffffffffu, x, 31);
    if (lane < GS_T / 32) wcnt[lane] = x - wc;          // warp offsets inside the tile
    const unsigned long long VMASK = (1ull << 62) - 1;
    if (lane == 0) {
      __threadfence();
      st[tile] = ((tile == 0 ? 2ull : 1ull) << 62) | (unsigned long long)agg;
    }
    uint64_t prefix = 0;
    for (int64_t t = (int64_t)tile - 1; t >= 0; t -= 32) {   // warp-parallel look-back
      const int64_t q = t - lane;
      unsigned long long v = 2ull << 62;
      if (q >= 0) {
        do { v = st[q]; } while ((v >> 62) == 0);
      }
      const uint32_t inc = __ballot_sync(0xffffffffu, (v >> 62) == 2);
      const int stop = inc ? __ffs(inc) - 1 : 31;
      uint64_t contrib = lane <= stop ? (v & VMASK) : 0ull;
      for (int o = 16; o; o >>= 1) contrib += __shfl_xor_sync(0xffffffffu, contrib, o);
      prefix += contrib;
      if (inc) break;
    }
    if (lane == 0) {
      if (tile) {
        __threadfence();
        st[tile] = (2ull << 62) | (unsigned long long)(prefix + agg);
      }
      s_prefix = (uint32_t)prefix;
      if ((uint64_t)(tile + 1) * GS_TILE >= n) {        // last tile: the end sentinel and the count
        gstart[prefix + agg] = (uint32_t)n;
        if (ng_out) *ng_out = (uint32_t)(prefix + agg);
        if (widx) widx[n] = (uint32_t)(prefix + agg);
      }
    }
  }
  __syncthreads();
  uint32_t r = s_prefix + wcnt[w];
  const uint32_t lt = (1u << lane) - 1u;
#pragma unroll
  for (int j = 0; j < GS_I; ++j) {
    const uint64_t i = base + j * 32 + lane;
    const uint32_t f = (bal[j] >> lane) & 1u;
    const uint32_t x = r + __popc(bal[j] & lt);
    if (f) gstart[x] = (uint32_t)i;
    if (widx && i < n) {
      widx[i] = x;
      hf[i] = f;
    }
    r += __popc(bal[j]);
  }
}

// GPMA_GSTART_FUSED=0: group starts (level 0) and the segments of every
// host-driven level by flags + scan + scatter (read per call)
static bool gstart_fused() {
  const char *e = getenv("GPMA_GSTART_FUSED");
  return !e || atoi(e) != 0;
}

static gpma_status group_starts(gpma *g, const uint64_t *tk, uint64_t n, uint32_t *gstart, uint32_t *ng_out,
                                cudaStream_t s) {
  const uint64_t nt = std::max<uint64_t>(1, (n + GS_TILE - 1) / GS_TILE);
  DevBuf &sb = tl_scan ? *tl_scan : g->b_scan;
  GP_CHECK(g, ensure(g, sb, (nt + 1) * sizeof(unsigned long long), s));
  GP_CHECK(g, fill_zero(g, sb.p, (nt + 1) * sizeof(unsigned long long), s));
  GP_LAUNCH(g, k_group_starts<uint64_t>, (unsigned)nt, GS_T, 0, s, tk, n, 0u, gstart, ng_out, (uint32_t *)nullptr,
            (uint32_t *)nullptr, (unsigned long long *)sb.p, g->ctrl_d);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// One thread per leaf group of the leaf-sorted batch (updates in arrival order): the leaf in
// registers as in k_ins_leaf_t.  Pass 1 decides every update -- a later copy of the same key in
// the group supersedes it (R10); a key equal to an occupied slot overwrites / revives it
// (R11, R12); the rest are new -- and writes keep[j] = 1 for the new ones.  Accepted (density
// n_live + u_new <= max_0): tombstones dropped, the new keys inserted at their key rank (one
// static shift each, any order), the leaf written back; rejected: hits in place, keep stays 1.
// ---- one leaf group, the leaf in a row of shared memory (rk, rv): Alg. 4 l.3-15 at the leaves
// for the updates j0..j1 of the group (any order; U.key(j) / U.val(j)).  The last copy of a key
// in the group acts (R10); a key equal to an occupied slot overwrites (R11) / revives (R12) it;
// the rest are new.  Density n_live + u_new <= max_0 (l.25, R5): the tombstones are dropped,
// the new keys inserted at their key rank, the row left-packed (R7 for one leaf) and the leaf's
// count / tombstone mask / head / guard row offsets maintained; otherwise the hits stay in
// place and keep[j] = 1 flags the new keys pending for level 1.  Out-degrees: +1 per new key
// or revive.  The caller writes the row back (keys when ok, values when ok or hitm).
struct LeafOut {
  bool ok = false;
  uint32_t hitm = 0, nnew = 0, effs = 0;
};

struct UpdIdx {                 // the leaf-sorted batch: arrival indices into the staged batch
  const uint64_t *ik;
  const uint32_t *iv;
  const uint32_t *tix;
  __device__ uint64_t key(uint32_t j) const { return ik[tix[j]]; }
  __device__ uint32_t val(uint32_t j) const { return iv[tix[j]]; }
};

struct UpdDirect {              // a key-sorted batch (shared or global memory)
  const uint64_t *k;
  const uint32_t *v;
  __device__ uint64_t key(uint32_t j) const { return k[j]; }
  __device__ uint32_t val(uint32_t j) const { return v[j]; }
};

template <bool SORTED, class Upd>
__device__ __forceinline__ LeafOut leaf_group_merge(uint64_t *rk, uint32_t *rv, uint32_t L, uint32_t t, uint32_t j0,
                                                    uint32_t j1, const Upd &U, uint32_t bound, uint32_t *keep,
                                                    const uint64_t *key, uint32_t *cnt, uint32_t *tmask,
                                                    uint64_t *head, uint64_t *row_offset, uint32_t *deg, uint32_t rb,
                                                    uint2 *dirty, Ctrl *c) {
  LeafOut o;
  const uint64_t lb = (uint64_t)t * L;
  uint32_t nocc = 0, tomb = 0;
  for (; nocc < L && rk[nocc] != KEY_NONE; ++nocc) tomb |= (rv[nocc] == VAL_TOMB ? 1u : 0u) << nocc;
  const uint64_t h_old = rk[0];
  uint32_t revm = 0;
  for (uint32_t j = j0; j < j1; ++j) {
    const uint64_t uk = U.key(j);
    bool last = true;                                    // R10: a later copy in the group wins
    if (SORTED) last = j + 1 == j1 || U.key(j + 1) != uk;   // (key-sorted: copies are adjacent)
    else
      for (uint32_t j2 = j + 1; j2 < j1 && last; ++j2) last = U.key(j2) != uk;   // (groups <= IL_BIG)
    uint32_t h = 0;
    if (last) {
      ++o.effs;
      uint32_t lo = 0, hi = nocc;                        // the occupied prefix is sorted
      while (lo < hi) {
        const uint32_t mid = (lo + hi) >> 1;
        if (rk[mid] < uk) lo = mid + 1;
        else hi = mid;
      }
      if (lo < nocc && rk[lo] == uk) {                   // overwrite (R11) / revive (R12)
        h = 1u << lo;
        rv[lo] = U.val(j);
      }
      o.hitm |= h;
      revm |= h & tomb;
      o.nnew += h ? 0u : 1u;
      if (!h || (h & tomb)) atomicAdd(&deg[(uint32_t)(uk >> 32) - rb], 1u);   // new key or revive
    }
    keep[j] = (last && !h) ? 1u : 0u;
  }
  const uint32_t dead = tomb & ~revm;
  const uint32_t n = nocc - __popc(dead);
  o.ok = o.nnew > 0 && o.nnew <= bound && n + o.nnew <= bound;
  if (o.ok) {
    uint32_t N = n;
    if (dead) {                                          // drop the tombstones: left-pack the live
      uint32_t w2 = 0;
      for (uint32_t p = 0; p < nocc; ++p)
        if (!((dead >> p) & 1u)) {
          rk[w2] = rk[p];
          rv[w2] = rv[p];
          ++w2;
        }
    }
    for (uint32_t j = j0; j < j1; ++j) {                 // the new keys at their key rank
      if (!keep[j]) continue;
      keep[j] = 0u;
      const uint64_t uk = U.key(j);
      uint32_t pos = N;
      while (pos > 0 && rk[pos - 1] > uk) {
        rk[pos] = rk[pos - 1];
        rv[pos] = rv[pos - 1];
        --pos;
      }
      rk[pos] = uk;
      rv[pos] = U.val(j);
      ++N;
    }
    for (uint32_t p = N; p < nocc; ++p) {
      rk[p] = KEY_NONE;
      rv[p] = 0;
    }
    for (uint32_t p = 0; p < N; ++p)
      if (is_guard_key(rk[p])) row_offset[(rk[p] >> 32) - rb + 1] = lb + p;   // R8: guards that moved
    cnt[t] = N;
    if (tomb) tmask[t] = 0u;                             // (no tombstone in the leaf: already 0)
    if (rk[0] != h_old) {
      head[t] = rk[0];
      if (t > 0 && key[lb - L] == KEY_NONE) {            // empty leaves to the left carry this head
        const uint64_t d = atomicAdd((unsigned long long *)&c->ndirty, 1ull);
        dirty[d] = make_uint2(t, 1u);
      }
    }
  } else if (revm) {
    cnt[t] += __popc(revm);
    tmask[t] &= ~revm;
  }
  return o;
}

constexpr int ILU_T = 128;      // 4 warps: 4 x 32 leaves staged in shared memory
constexpr uint32_t IL_BIG = 64;  // larger leaf groups take the key-sorted fallback (no O(u^2) dedupe)
template <int L>
__global__ void __launch_bounds__(ILU_T) k_ins_leaf_u(const uint64_t *__restrict__ ik, const uint32_t *__restrict__ iv,
                                                    const uint64_t *__restrict__ tk, const uint32_t *__restrict__ tix,
                                                    const uint32_t *__restrict__ gstart,
                                                    const uint32_t *__restrict__ ng_dev, uint64_t *key, uint32_t *val,
                                                    uint32_t *__restrict__ cnt, uint32_t *__restrict__ tmask,
                                                    uint64_t *__restrict__ head, uint64_t *__restrict__ row_offset,
                                                    uint32_t *__restrict__ deg, uint32_t rb, uint32_t bound,
                                                    uint32_t *__restrict__ keep, uint32_t *__restrict__ bigf,
                                                    uint2 *__restrict__ dirty, Ctrl *c) {
  // Leaf I/O is warp-cooperative: the 32 leaves of a warp's 32 groups move through shared memory
  // in coalesced 16-B chunks (L/2 lanes per leaf for the keys, L/4 for the values), so a leaf is
  // whole 128-B lines instead of 32 single-sector requests per load instruction.
  constexpr int KS = L + 1;                            // padded row (u64 / u32 words)
  __shared__ uint64_t sK[ILU_T / 32][32 * KS];
  __shared__ uint32_t sV[ILU_T / 32][32 * KS];
  if (c->err) return;
  const uint32_t ng = *ng_dev;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  uint64_t *const mk = sK[w];
  uint32_t *const mv = sV[w];
  constexpr int KL = L / 2, KQ = 32 / KL;               // key chunks per leaf, leaves per load round
  constexpr int VL = L / 4 > 0 ? L / 4 : 1, VQ = 32 / VL;
  uint32_t accepted = 0, news = 0, effs = 0;
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t gb = (blockIdx.x * (uint64_t)blockDim.x) + (threadIdx.x & ~31); gb < ng; gb += stride) {  // warp-uniform
    const uint64_t gi = gb + lane;
    const bool have = gi < ng;
    uint32_t j0 = 0, j1 = 0, t = 0;
    if (have) {
      j0 = gstart[gi];
      j1 = gstart[gi + 1];
      t = (uint32_t)tk[j0];
    }
    const uint64_t lb = (uint64_t)t * L;
    // cooperative load of the 32 leaves into shared memory
#pragma unroll
    for (int it = 0; it < 32 / KQ; ++it) {
      const int q = it * KQ + lane / KL, cc = lane % KL;
      const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
      const bool hq = __shfl_sync(0xffffffffu, have, q);
      if (hq) {
        const ulonglong2 kk = *reinterpret_cast<const ulonglong2 *>(key + lq + 2 * cc);
        mk[q * KS + 2 * cc] = kk.x;
        mk[q * KS + 2 * cc + 1] = kk.y;
      }
    }
#pragma unroll
    for (int it = 0; it < 32 / VQ; ++it) {
      const int q = it * VQ + lane / VL, cc = lane % VL;
      const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
      const bool hq = __shfl_sync(0xffffffffu, have, q);
      if (hq) {
        if (L >= 4) {
          const uint4 vv = *reinterpret_cast<const uint4 *>(val + lq + 4 * cc);
          mv[q * KS + 4 * cc] = vv.x;
          mv[q * KS + 4 * cc + 1] = vv.y;
          mv[q * KS + 4 * cc + 2] = vv.z;
          mv[q * KS + 4 * cc + 3] = vv.w;
        }
      }
    }
    __syncwarp();
    // the thread's leaf is its row of shared memory: dynamic indexing is free there, so the
    // merge is a few moves per update instead of static select networks over registers
    const UpdIdx U{ik, iv, tix};
    // an oversized group (> IL_BIG updates: an adversarial batch piling into one leaf) is left to
    // the key-sorted fallback after the kernel; its updates are flagged in bigf
    const bool big = have && j1 - j0 > IL_BIG;
    if (have)
      for (uint32_t j = j0; j < j1; ++j) {
        bigf[j] = big ? 1u : 0u;
        if (big) keep[j] = 0u;
      }
    if (big) atomicAdd((unsigned long long *)&c->big, (unsigned long long)(j1 - j0));
    const LeafOut lo_ = have && !big ? leaf_group_merge<false>(mk + lane * KS, mv + lane * KS, (uint32_t)L, t, j0, j1, U,
                                                               bound, keep, key, cnt, tmask, head, row_offset, deg,
                                                               rb, dirty, c)
                                     : LeafOut{};
    const bool ok = lo_.ok;
    const uint32_t hitm = lo_.hitm;
    news += lo_.nnew;
    effs += lo_.effs;
    accepted += ok ? 1u : 0u;
    const bool vdirty = ok || hitm;                      // the values go back for hits too
    __syncwarp();
    // cooperative store of the accepted (rewritten) leaves
#pragma unroll
    for (int it = 0; it < 32 / KQ; ++it) {
      const int q = it * KQ + lane / KL, cc = lane % KL;
      const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
      const bool oq = __shfl_sync(0xffffffffu, ok, q);
      if (oq)
        *reinterpret_cast<ulonglong2 *>(key + lq + 2 * cc) = make_ulonglong2(mk[q * KS + 2 * cc], mk[q * KS + 2 * cc + 1]);
    }
#pragma unroll
    for (int it = 0; it < 32 / VQ; ++it) {
      const int q = it * VQ + lane / VL, cc = lane % VL;
      const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
      const bool oq = __shfl_sync(0xffffffffu, vdirty, q);
      if (oq)
        *reinterpret_cast<uint4 *>(val + lq + 4 * cc) =
            make_uint4(mv[q * KS + 4 * cc], mv[q * KS + 4 * cc + 1], mv[q * KS + 4 * cc + 2], mv[q * KS + 4 * cc + 3]);
    }
    __syncwarp();
  }
  accepted = __reduce_add_sync(0xffffffffu, accepted);
  news = __reduce_add_sync(0xffffffffu, news);
  effs = __reduce_add_sync(0xffffffffu, effs);
  if (lane == 0) {
    if (accepted) atomicAdd((unsigned long long *)&c->windows_rewritten, (unsigned long long)accepted);
    if (news) atomicAdd((unsigned long long *)&c->sum, (unsigned long long)news);
    if (effs) atomicAdd((unsigned long long *)&c->nunique, (unsigned long long)effs);
  }
}

// ---- R-way interleaved locate (memory-level parallelism): the random loads of R independent
// keys -- row offsets, head probes, the first 8 slots of the target leaf -- are issued together,
// so a thread keeps R dependent chains in flight instead of one (the kernels below are bound by
// DRAM latency at full occupancy: one chain per thread left DRAM at ~43 % of its bandwidth).
template <int R>
__device__ __forceinline__ void locate_leaf_rows_r(const uint64_t *__restrict__ head, uint32_t nleaves,
                                                   const uint64_t *__restrict__ ro, uint32_t rb, uint32_t L,
                                                   const uint64_t (&k)[R], const bool (&v)[R], uint32_t (&t)[R],
                                                   float fv = 0.f) {
  uint32_t lo[R], hi[R], a[R];
  if (!ro) {
#pragma unroll
    for (int q = 0; q < R; ++q) t[q] = v[q] ? locate_leaf(head, nleaves, k[q]) : 0u;
    return;
  }
  ulonglong2 r[R];
#pragma unroll
  for (int q = 0; q < R; ++q) {
    const uint32_t u = (uint32_t)(k[q] >> 32) - rb;
    r[q] = v[q] ? make_ulonglong2(__ldg(ro + u), __ldg(ro + u + 1)) : make_ulonglong2(0, 0);
  }
#pragma unroll
  for (int q = 0; q < R; ++q) {
    // the answer is >= a either way (see locate_leaf_rows), so the search starts past a: one
    // random probe less per key, none for a row inside one leaf
    a[q] = (uint32_t)leaf_div(r[q].x, L);
    lo[q] = a[q] + 1;
    hi[q] = v[q] ? min((uint32_t)leaf_div(r[q].y, L) + 1, nleaves) : a[q];
  }
  if (fv > 0.f) {
    // Interpolation step for rows over more than 8 leaves (fv = 1/V): the row's keys are sorted
    // by dst, so the leaf of (u, dst) sits near a + dst/V * (row leaves).  The aligned 64-B line
    // of 8 heads around that guess is read in one access; it either brackets the answer (done)
    // or cuts the range at its edge.  Replaces the ~5 dependent head probes an RMAT delete made
    // (edge-weighted row spans are hundreds of leaves) by about one; exact for any data (a bad
    // guess only leaves more range for the binary search below).
    ulonglong2 hl[R][4];
    uint32_t ls[R];
    bool use[R];
#pragma unroll
    for (int q = 0; q < R; ++q) {
      use[q] = v[q] && hi[q] > lo[q] + 8;
      uint32_t g = a[q] + (uint32_t)((float)(uint32_t)k[q] * fv * (float)(hi[q] - a[q]));
      g = min(max(g, lo[q]), hi[q] - 1);
      ls[q] = g & ~7u;
#pragma unroll
      for (int j = 0; j < 4; ++j)
        hl[q][j] = use[q] ? __ldg(reinterpret_cast<const ulonglong2 *>(head + ls[q]) + j) : make_ulonglong2(0, 0);
    }
#pragma unroll
    for (int q = 0; q < R; ++q) {
      if (!use[q]) continue;
      const uint32_t wlo = max(ls[q], lo[q]), whi = min(ls[q] + 8, hi[q]);
      uint32_t cnt = 0;
#pragma unroll
      for (int j = 0; j < 8; ++j) {
        const uint32_t idx = ls[q] + j;
        const uint64_t h = (j & 1) ? hl[q][j >> 1].y : hl[q][j >> 1].x;
        cnt += (idx >= wlo && idx < whi && h <= k[q]) ? 1u : 0u;
      }
      if (cnt < whi - wlo) {                             // a head > k inside the line
        if (cnt > 0 || wlo == lo[q]) lo[q] = hi[q] = wlo + cnt;
        else hi[q] = wlo;
      } else {
        lo[q] = whi;
      }
    }
  }
  bool any = true;
  while (any) {
    uint64_t hv[R];
    uint32_t mid[R];
#pragma unroll
    for (int q = 0; q < R; ++q) {
      mid[q] = (lo[q] + hi[q]) >> 1;
      hv[q] = lo[q] < hi[q] ? __ldg(head + mid[q]) : 0ull;
    }
    any = false;
#pragma unroll
    for (int q = 0; q < R; ++q)
      if (lo[q] < hi[q]) {
        if (hv[q] <= k[q]) lo[q] = mid[q] + 1;
        else hi[q] = mid[q];
        any |= lo[q] < hi[q];
      }
  }
#pragma unroll
  for (int q = 0; q < R; ++q) t[q] = v[q] ? lo[q] - 1 : a[q];
}

// slot of k[q] in its leaf t[q] (or -1) for R keys: the leaves' slots fetched 8 at a time, the
// R leaves of a round together (the occupied prefix is sorted, KEY_NONE > every key)
template <int R>
__device__ __forceinline__ void find_in_leaf_r(const uint64_t *__restrict__ key, uint32_t L, const uint64_t (&k)[R],
                                               const bool (&v)[R], const uint32_t (&t)[R], int (&pos)[R]) {
  bool more[R];
#pragma unroll
  for (int q = 0; q < R; ++q) {
    pos[q] = -1;
    more[q] = v[q];
  }
  for (uint32_t p0 = 0; p0 < L; p0 += 8) {
    bool any = false;
#pragma unroll
    for (int q = 0; q < R; ++q) any |= more[q];
    if (!any) break;
    ulonglong2 a[R][4];
#pragma unroll
    for (int q = 0; q < R; ++q)
#pragma unroll
      for (int j = 0; j < 4; ++j)
        a[q][j] = more[q] && p0 + 2 * j < L
                      ? __ldg(reinterpret_cast<const ulonglong2 *>(key + (uint64_t)t[q] * L + p0 + 2 * j))
                      : make_ulonglong2(KEY_NONE, KEY_NONE);
#pragma unroll
    for (int q = 0; q < R; ++q) {
#pragma unroll
      for (int j = 0; j < 4; ++j) {
        if (!more[q]) break;
        if (a[q][j].x == k[q]) { pos[q] = (int)(p0 + 2 * j); more[q] = false; }
        else if (a[q][j].x > k[q]) more[q] = false;
        else if (a[q][j].y == k[q]) { pos[q] = (int)(p0 + 2 * j + 1); more[q] = false; }
        else if (a[q][j].y > k[q]) more[q] = false;
      }
    }
  }
}

// The control block mirrored into pinned host memory by the kernel's thread 0 (after a barrier):
// the fields, a system fence, then the sequence number -- the host sees the whole block once it
// sees the number (wait_ctrl), without waiting for the kernel's completion to reach the stream.
__device__ __forceinline__ void mirror_ctrl(const Ctrl *c, Ctrl *c_host, uint32_t seq) {
  *c_host = *c;                    // (device data reaches the host's later stream work in order)
  __threadfence_system();
  *reinterpret_cast<volatile uint32_t *>(&c_host->seq) = seq;
}

// ---- small batches in ONE kernel (n <= SB_MAX): the paper names kernel-call overheads as what
// dominates small batches.  A single CTA validates the batch (nothing changes on
// an error), sorts it by key in shared memory (bitonic, arrival index breaks ties: stable, R10),
// locates every key (R9), forms the leaf groups, merges them (leaf_group_merge, leaves staged
// in shared-memory rows), compacts the rejected keys -- already key-sorted -- into the pending
// list for level 1 and mirrors its control block to pinned host memory: one launch and one
// host synchronisation per call instead of a dozen launches.  Lazy deletes likewise.
constexpr int SB_T = 1024, SB_MAX = 2048, SB_ROWS = 512, SB_DEL_MAX = 4096;
constexpr size_t SB_ROWK_OFF = ((size_t)SB_MAX * 8 + (size_t)SB_MAX * 4 * 2 + (size_t)(SB_MAX + 1) * 4 * 2 + 15) & ~(size_t)15;
__host__ __device__ constexpr size_t sb_smem_bytes(int L) { return SB_ROWK_OFF + (size_t)SB_ROWS * (L + 1) * 12; }

__device__ __forceinline__ void sb_block_scan2(uint32_t (&v)[2], uint32_t *wsum, uint32_t *total) {
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t t = v[0] + v[1];
  uint32_t x = t;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  if (lane == 31) wsum[warp] = x;
  __syncthreads();
  if (warp == 0) {
    uint32_t w = wsum[lane];
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, w, o);
      if (lane >= o) w += y;
    }
    wsum[lane] = w;
  }
  __syncthreads();
  const uint32_t base = (warp ? wsum[warp - 1] : 0) + x - t;
  *total = wsum[31];
  __syncthreads();
  v[1] = base + v[0];
  v[0] = base;
}

template <int L>
__global__ void __launch_bounds__(SB_T) k_small_insert(const uint64_t *__restrict__ ik, const uint32_t *__restrict__ iv,
                                                       uint32_t n, uint64_t *key, uint32_t *val, uint32_t *cnt,
                                                       uint32_t *tmask, uint64_t *head, uint64_t *row_offset,
                                                       uint32_t *deg, uint32_t nleaves, uint32_t rb, uint32_t nr,
                                                       uint32_t V, uint32_t bound, const uint64_t *__restrict__ ro,
                                                       uint64_t *pk, uint32_t *pv, uint32_t *pt, uint2 *dirty, Ctrl *c,
                                                       Ctrl *c_host, uint32_t seq, uint32_t pbd, float fv) {
  extern __shared__ __align__(16) unsigned char sb_smem[];
  uint64_t *sk = reinterpret_cast<uint64_t *>(sb_smem);           // [SB_MAX] keys (sorted)
  uint32_t *si = reinterpret_cast<uint32_t *>(sk + SB_MAX);       // [SB_MAX] arrival index -> sorted values
  uint32_t *st = si + SB_MAX;                                     // [SB_MAX] target leaves
  uint32_t *kp = st + SB_MAX;                                     // [SB_MAX + 1] keep flags / group starts
  uint32_t *gs = kp + SB_MAX + 1;                                 // [SB_MAX + 1] group starts
  uint64_t *rowk = reinterpret_cast<uint64_t *>(sb_smem + SB_ROWK_OFF);   // [SB_ROWS][L + 1]
  uint32_t *rowv = reinterpret_cast<uint32_t *>(rowk + SB_ROWS * (L + 1));
  __shared__ uint32_t wsum[32];
  __shared__ uint32_t s_stats[3];
  const int tid = threadIdx.x;
  if (tid == 0) {
    c->err = 0;
    c->nunique = 0;
    c->windows_rewritten = 0;
    c->ndirty = 0;
    c->sum = 0;
    c->sum2 = 0;
    c->big = 0;
    s_stats[0] = s_stats[1] = s_stats[2] = 0;
  }
  // load + validate (RESERVED beats RANGE; nothing is mutated on either) + locate (R9): each
  // thread's two keys located together while the batch is still in arrival order (an invalid
  // key is not located); values and targets parked by arrival index in kp / gs
  uint32_t e = 0;
  {
    uint64_t k[2];
    bool v[2];
    for (int q = 0; q < 2; ++q) {
      const uint32_t i = tid + q * SB_T;
      v[q] = i < n;
      k[q] = v[q] ? ik[i] : 0ull;
      const uint32_t x = v[q] ? iv[i] : 0u;
      if (v[q]) {
        const uint32_t src = (uint32_t)(k[q] >> 32), dst = (uint32_t)k[q];
        uint32_t ee = 0;
        if (dst == COL_GUARD || x == VAL_TOMB) ee |= 2u;
        if (src - rb >= nr || dst >= V) ee |= 1u;
        e |= ee;
        v[q] = ee == 0;
        sk[i] = k[q];
        si[i] = i;
        kp[i] = x;
      }
    }
    uint32_t t[2];
    locate_leaf_rows_r<2>(head, nleaves, ro, rb, L, k, v, t, fv);
    for (int q = 0; q < 2; ++q) {
      const uint32_t i = tid + q * SB_T;
      if (i < n) gs[i] = t[q];
    }
  }
  e = __syncthreads_or(e) ? (__reduce_or_sync(0xffffffffu, e)) : 0u;
  if (e) atomicOr(&c->err, e);
  __syncthreads();
  if (c->err) {
    if (tid == 0) mirror_ctrl(c, c_host, seq);
    return;
  }
  // stable sort by key (the arrival index breaks ties), padding up to a power of two
  uint32_t np2 = 2;
  while (np2 < n) np2 <<= 1;
  if (pbd) {
    np2 = np2 < 64 ? 64 : np2;                         // (the merge sort's register phase is 64 wide)
    // (src - rb, dst, arrival) packed into one distinct u64 (pbd = dst bits; the host checks
    // that row bits + pbd + 11 <= 64): half the shuffles and one compare per stage
    for (uint32_t i = tid; i < np2; i += SB_T)
      sk[i] = i < n ? ((((sk[i] >> 32) - rb) << (pbd + 11)) | ((sk[i] & 0xFFFFFFFFull) << 11) | i) : ~0ull;
    __syncthreads();
    cta_merge_sort_u64(sk, np2);
    for (uint32_t i = tid; i < n; i += SB_T) {
      const uint64_t pw = sk[i];
      si[i] = (uint32_t)(pw & (SB_MAX - 1));
      sk[i] = (((pw >> (pbd + 11)) + rb) << 32) | ((pw >> 11) & ((1ull << pbd) - 1));
    }
    __syncthreads();
  } else {
    for (uint32_t i = n + tid; i < np2; i += SB_T) {
      sk[i] = KEY_NONE;
      si[i] = i;
    }
    __syncthreads();
    cta_bitonic_sort(sk, si, np2);
  }
  // values and targets in key order, group heads
  uint32_t f[2], sv_[2], st_[2];
  for (int q = 0; q < 2; ++q) {
    const uint32_t i = tid * 2 + q;
    if (i < n) {
      sv_[q] = kp[si[i]];
      st_[q] = gs[si[i]];
    }
  }
  __syncthreads();
  for (int q = 0; q < 2; ++q) {
    const uint32_t i = tid * 2 + q;
    if (i < n) {
      si[i] = sv_[q];
      st[i] = st_[q];
    }
  }
  __syncthreads();
  for (int q = 0; q < 2; ++q) {
    const uint32_t i = tid * 2 + q;
    f[q] = (i < n && (i == 0 || st[i] != st[i - 1])) ? 1u : 0u;
  }
  uint32_t fe[2] = {f[0], f[1]}, ng = 0;
  sb_block_scan2(fe, wsum, &ng);
  for (int q = 0; q < 2; ++q)
    if (f[q]) gs[fe[q]] = tid * 2 + q;
  if (tid == 0) gs[ng] = n;
  __syncthreads();
  // the leaf groups, SB_ROWS at a time, each leaf in a shared-memory row
  const UpdDirect U{sk, si};
  uint32_t a_ok = 0, a_new = 0, a_effs = 0;
  // Leaf I/O is warp-cooperative (as in k_ins_leaf_u): the 32 leaves of a warp's rows move in
  // 16-B chunks, L/2 lanes per leaf row of keys and L/4 per row of values, so one warp
  // instruction moves whole lines of 32 / (L/2) leaves instead of 32 scattered slots (per-thread
  // slot loops made a 512-row round ~17 us, bound by the SM's memory request rate).
  constexpr int KL = L / 2, KQ = 32 / KL, VL = L / 4, VQ = 32 / VL;
  for (uint32_t g0 = 0; g0 < ng; g0 += SB_ROWS) {
    if (tid < SB_ROWS) {                                 // whole warps (SB_ROWS % 32 == 0)
      const uint32_t gi = g0 + tid;
      const int lane = tid & 31;
      const uint32_t wb = tid & ~31u;
      const bool have = gi < ng;
      uint32_t j0 = 0, j1 = 0, t = 0;
      if (have) {
        j0 = gs[gi];
        j1 = gs[gi + 1];
        t = st[j0];
      }
      const uint64_t lb = (uint64_t)t * L;
      uint64_t *rk = rowk + tid * (L + 1);
      uint32_t *rv = rowv + tid * (L + 1);
      ulonglong2 kx[32 / KQ];
      uint4 vx[32 / VQ];
#pragma unroll
      for (int it = 0; it < 32 / KQ; ++it) {
        const int q = it * KQ + lane / KL, cc = lane % KL;
        const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
        const bool hq = __shfl_sync(0xffffffffu, have, q);
        kx[it] = hq ? __ldcg(reinterpret_cast<const ulonglong2 *>(key + lq) + cc) : make_ulonglong2(0, 0);
      }
#pragma unroll
      for (int it = 0; it < 32 / VQ; ++it) {
        const int q = it * VQ + lane / VL, cc = lane % VL;
        const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
        const bool hq = __shfl_sync(0xffffffffu, have, q);
        vx[it] = hq ? __ldcg(reinterpret_cast<const uint4 *>(val + lq) + cc) : make_uint4(0, 0, 0, 0);
      }
#pragma unroll
      for (int it = 0; it < 32 / KQ; ++it) {
        const int q = it * KQ + lane / KL, cc = lane % KL;
        uint64_t *r = rowk + (wb + q) * (L + 1) + 2 * cc;
        r[0] = kx[it].x;
        r[1] = kx[it].y;
      }
#pragma unroll
      for (int it = 0; it < 32 / VQ; ++it) {
        const int q = it * VQ + lane / VL, cc = lane % VL;
        uint32_t *r = rowv + (wb + q) * (L + 1) + 4 * cc;
        r[0] = vx[it].x;
        r[1] = vx[it].y;
        r[2] = vx[it].z;
        r[3] = vx[it].w;
      }
      __syncwarp();
      LeafOut o;
      if (have)
        o = leaf_group_merge<true>(rk, rv, (uint32_t)L, t, j0, j1, U, bound, kp, key, cnt, tmask, head, row_offset,
                                   deg, rb, dirty, c);
      __syncwarp();
      const bool vdirty = o.ok || o.hitm;
#pragma unroll
      for (int it = 0; it < 32 / KQ; ++it) {
        const int q = it * KQ + lane / KL, cc = lane % KL;
        const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
        const bool oq = __shfl_sync(0xffffffffu, o.ok, q);
        const uint64_t *r = rowk + (wb + q) * (L + 1) + 2 * cc;
        if (oq) *reinterpret_cast<ulonglong2 *>(key + lq + 2 * cc) = make_ulonglong2(r[0], r[1]);
      }
#pragma unroll
      for (int it = 0; it < 32 / VQ; ++it) {
        const int q = it * VQ + lane / VL, cc = lane % VL;
        const uint64_t lq = __shfl_sync(0xffffffffu, lb, q);
        const bool oq = __shfl_sync(0xffffffffu, vdirty, q);
        const uint32_t *r = rowv + (wb + q) * (L + 1) + 4 * cc;
        if (oq) *reinterpret_cast<uint4 *>(val + lq + 4 * cc) = make_uint4(r[0], r[1], r[2], r[3]);
      }
      __syncwarp();
      a_ok += o.ok ? 1u : 0u;
      a_new += o.nnew;
      a_effs += o.effs;
    }
  }
  a_ok = __reduce_add_sync(0xffffffffu, a_ok);         // one shared atomic per warp
  a_new = __reduce_add_sync(0xffffffffu, a_new);
  a_effs = __reduce_add_sync(0xffffffffu, a_effs);
  if ((tid & 31) == 0 && (a_ok | a_new | a_effs)) {
    atomicAdd(&s_stats[0], a_ok);
    atomicAdd(&s_stats[1], a_new);
    atomicAdd(&s_stats[2], a_effs);
  }
  __syncthreads();
  // the rejected new keys, in key order, with their targets: the pending list of level 1
  uint32_t kf[2];
  for (int q = 0; q < 2; ++q) {
    const uint32_t i = tid * 2 + q;
    kf[q] = i < n ? kp[i] : 0u;
  }
  uint32_t kq[2] = {kf[0], kf[1]}, npend = 0;
  sb_block_scan2(kq, wsum, &npend);
  for (int q = 0; q < 2; ++q) {
    const uint32_t i = tid * 2 + q;
    if (kf[q]) {
      pk[kq[q]] = sk[i];
      pv[kq[q]] = si[i];
      pt[kq[q]] = st[i];
    }
  }
  __syncthreads();
  if (tid == 0) {
    c->windows_rewritten += s_stats[0];
    c->sum = s_stats[1];              // new keys (pending after the pre-pass, in the old terms)
    c->nunique = s_stats[2];
    c->sum2 = npend;                  // pending after level 0
    mirror_ctrl(c, c_host, seq);      // the control block, mirrored (zero-copy) for the host
  }
}

// small lazy-delete batch in ONE launch of ceil(n / SD_T) CTAs: every CTA validates
// the whole batch (<= SB_DEL_MAX keys, L2-resident) so that none marks anything unless all keys
// are valid -- no grid barrier -- then marks its own slice (R keys per thread in flight); the
// last CTA to finish (a self-resetting counter) mirrors the control block to the host.  The
// single-CTA version ran the locate chains of 1024 keys on one SM.
constexpr int SD_T = 256;
__global__ void __launch_bounds__(SD_T) k_small_delete(const uint64_t *__restrict__ ik, uint32_t n,
                                                       const uint64_t *__restrict__ key, uint32_t *val, uint32_t *cnt,
                                                       const uint64_t *__restrict__ head, uint32_t nleaves, uint32_t L,
                                                       uint32_t *tmask, uint32_t *deg, uint32_t rb, uint32_t nr,
                                                       uint32_t V, const uint64_t *__restrict__ ro, Ctrl *c,
                                                       Ctrl *c_host, uint32_t seq, float fv) {
  const int tid = threadIdx.x;
  uint32_t e = 0;
  for (uint32_t i = tid; i < n; i += SD_T) {
    const uint64_t k = ik[i];
    const uint32_t src = (uint32_t)(k >> 32), dst = (uint32_t)k;
    if (dst == COL_GUARD) e |= 2u;
    if (src - rb >= nr || dst >= V) e |= 1u;
  }
  e = __syncthreads_or(e) ? (__reduce_or_sync(0xffffffffu, e)) : 0u;
  __shared__ uint32_t s_err;
  if (tid == 0) s_err = 0;
  __syncthreads();
  if (e && (tid & 31) == 0) atomicOr(&s_err, e);
  __syncthreads();
  if (s_err) {                                           // every CTA sees it; CTA 0 reports
    if (blockIdx.x == 0 && tid == 0) {
      c->err = s_err;
      c->nunique = c->sum = c->sum2 = 0;
      mirror_ctrl(c, c_host, seq);
    }
    return;
  }
  {
    const uint32_t i0 = blockIdx.x * SD_T + tid;
    uint64_t k[2];
    bool v[2];
#pragma unroll
    for (int q = 0; q < 2; ++q) {
      const uint32_t i = i0 + q * gridDim.x * SD_T;
      v[q] = i < n;
      k[q] = v[q] ? ik[i] : 0ull;
    }
    uint32_t t[2];
    locate_leaf_rows_r<2>(head, nleaves, ro, rb, L, k, v, t, fv);
    int p[2];
    find_in_leaf_r<2>(key, L, k, v, t, p);
    uint32_t old[2];
#pragma unroll
    for (int q = 0; q < 2; ++q)
      old[q] = p[q] >= 0 ? atomicExch(&val[(uint64_t)t[q] * L + p[q]], VAL_TOMB) : VAL_TOMB;   // duplicates: one accounts it
#pragma unroll
    for (int q = 0; q < 2; ++q)
      if (old[q] != VAL_TOMB) {
        atomicSub(&cnt[t[q]], 1u);
        atomicOr(&tmask[t[q]], 1u << p[q]);
        atomicSub(&deg[(uint32_t)(k[q] >> 32) - rb], 1u);
      }
  }
  __syncthreads();
  if (tid == 0) {
    __threadfence();
    if (atomicAdd((unsigned long long *)&c->done, 1ull) == gridDim.x - 1) {
      c->done = 0;
      c->err = 0;
      c->nunique = c->sum = c->sum2 = 0;
      mirror_ctrl(c, c_host, seq);
    }
  }
}

// the rejected new keys (keep[j] = 1) of the leaf-sorted batch, compacted in leaf order with
// their targets, plus 0..p-1 (the sort of the pending keys permutes it)
__global__ void k_pend_gather(const uint32_t *__restrict__ keep, const uint32_t *__restrict__ pos, uint64_t n,
                              const uint32_t *__restrict__ tix, const uint64_t *__restrict__ tk,
                              const uint64_t *__restrict__ ik, const uint32_t *__restrict__ iv,
                              uint64_t *__restrict__ pk, uint32_t *__restrict__ pv, uint32_t *__restrict__ pt,
                              uint32_t *__restrict__ seq) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < n;
       j += (uint64_t)gridDim.x * blockDim.x) {
    if (!keep[j]) continue;
    const uint32_t d = pos[j], i = tix[j];
    pk[d] = ik[i];
    pv[d] = iv[i];
    pt[d] = (uint32_t)tk[j];
    seq[d] = d;
  }
}

// Pending list in key order without a radix sort: the gather left it in leaf order (leaves
// partition the key space), so only each leaf's own rejected keys -- one group, <= IL_BIG of them,
// distinct (R10 kept the last copy) -- need ordering.  Thread per entry: its rank among the
// entries of its leaf.  Writes the level-1 buffers (pk0, pv0, pt0).
__global__ void k_pend_segsort(const uint64_t *__restrict__ pk1, const uint32_t *__restrict__ pv1,
                               const uint32_t *__restrict__ pt1, uint64_t p, uint64_t *__restrict__ pk0,
                               uint32_t *__restrict__ pv0, uint32_t *__restrict__ pt0) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < p; i += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t t = pt1[i];
    const uint64_t k = pk1[i];
    uint64_t a = i, b = i + 1;
    while (a > 0 && pt1[a - 1] == t) --a;
    while (b < p && pt1[b] == t) ++b;
    uint64_t r = a;
    for (uint64_t j = a; j < b; ++j) r += pk1[j] < k ? 1u : 0u;
    pk0[r] = k;
    pv0[r] = pv1[i];
    pt0[r] = t;
  }
}

// pending list in key order: values and targets follow the sort's permutation
__global__ void k_pend_permute(const uint32_t *__restrict__ perm, uint64_t p, const uint32_t *__restrict__ pv_in,
                               const uint32_t *__restrict__ pt_in, uint32_t *__restrict__ pv, uint32_t *__restrict__ pt) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < p;
       j += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t q = perm[j];
    pv[j] = pv_in[q];
    pt[j] = pt_in[q];
  }
}

// Lazy deletion (R12) in arrival order, R keys per thread interleaved.  Duplicates
// race on the same slot; the exchange on the value lets exactly one account the deletion.
template <int LD_R>
__global__ void __launch_bounds__(256) k_lazy_delete_r(const uint64_t *__restrict__ keys, uint64_t n,
                                                       const uint64_t *__restrict__ key, uint32_t *val,
                                                       uint32_t *__restrict__ cnt, const uint64_t *__restrict__ head,
                                                       uint32_t nleaves, uint32_t L, uint32_t *__restrict__ tmask,
                                                       uint32_t *__restrict__ deg, uint32_t rb, const Ctrl *c,
                                                       const uint64_t *__restrict__ ro, float fv) {
  if (c->err) return;
  const uint64_t nthr = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i0 < n; i0 += nthr * LD_R) {
    uint64_t k[LD_R];
    bool v[LD_R];
#pragma unroll
    for (int q = 0; q < LD_R; ++q) {
      const uint64_t i = i0 + (uint64_t)q * nthr;
      v[q] = i < n;
      k[q] = v[q] ? keys[i] : 0ull;
    }
    uint32_t t[LD_R];
    locate_leaf_rows_r<LD_R>(head, nleaves, ro, rb, L, k, v, t, fv);
    int p[LD_R];
    find_in_leaf_r<LD_R>(key, L, k, v, t, p);
    // one exchange per found key: the copy that swaps a live value for TOMB accounts it
    // (a duplicate, or an already-tombstoned slot, reads TOMB back)
    uint32_t old[LD_R];
#pragma unroll
    for (int q = 0; q < LD_R; ++q)
      old[q] = p[q] >= 0 ? atomicExch(&val[(uint64_t)t[q] * L + p[q]], VAL_TOMB) : VAL_TOMB;
#pragma unroll
    for (int q = 0; q < LD_R; ++q)
      if (old[q] != VAL_TOMB) {
        atomicSub(&cnt[t[q]], 1u);
        atomicOr(&tmask[t[q]], 1u << p[q]);
        atomicSub(&deg[(uint32_t)(k[q] >> 32) - rb], 1u);
      }
  }
}

// Target leaf of every update of the unsorted batch, R keys per thread interleaved
template <int LD_R>
__global__ void __launch_bounds__(256) k_locate_u_r(const uint64_t *__restrict__ ik, uint64_t n,
                                                    const uint64_t *__restrict__ head, uint32_t nleaves, uint32_t L,
                                                    uint32_t rb, const uint64_t *__restrict__ ro,
                                                    uint64_t *__restrict__ tk, uint32_t *__restrict__ tix,
                                                    const Ctrl *c, float fv) {
  if (c->err) return;
  const uint64_t nthr = (uint64_t)gridDim.x * blockDim.x;
  for (uint64_t i0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i0 < n; i0 += nthr * LD_R) {
    uint64_t k[LD_R];
    bool v[LD_R];
#pragma unroll
    for (int q = 0; q < LD_R; ++q) {
      const uint64_t i = i0 + (uint64_t)q * nthr;
      v[q] = i < n;
      k[q] = v[q] ? ik[i] : 0ull;
    }
    uint32_t t[LD_R];
    locate_leaf_rows_r<LD_R>(head, nleaves, ro, rb, L, k, v, t, fv);
#pragma unroll
    for (int q = 0; q < LD_R; ++q) {
      const uint64_t i = i0 + (uint64_t)q * nthr;
      if (v[q]) {
        tk[i] = t[q];
        tix[i] = (uint32_t)i;
      }
    }
  }
}

// Fused level 0 of the level loop (Alg. 4 l.7-15 at the leaves, where nearly every update
// is absorbed).  A warp takes the groups of pending updates (one group per target leaf) that
// start in its 32-item window and hands them to L-lane sub-warps (32/L groups at a time).  A
// sub-warp loads its leaf (lane l = slot l), counts the live entries with a ballot, tests the
// leaf bound max_0 (insert) / min_0 (strict delete) and, on success, merges in registers -- a
// live entry's rank is its live rank plus the updates below it, an update's rank its index
// plus the live entries below it -- and writes the left-packed leaf back (a one-leaf window
// is a single piece of the R7 split).  Rejected groups stay pending for level 1.  Control
// flow is uniform across the warp (everything predicated), so every shuffle is full-mask.
__global__ void __launch_bounds__(256) k_level0(const uint64_t *__restrict__ pk, const uint32_t *__restrict__ pv,
                                                const uint32_t *__restrict__ pt, const uint32_t *__restrict__ p_dev,
                                                uint64_t *key, uint32_t *val, uint32_t *__restrict__ cnt,
                                                uint32_t *__restrict__ tmask, uint64_t *__restrict__ head,
                                                uint64_t *__restrict__ row_offset, uint32_t rb, uint32_t L,
                                                uint32_t bound, int op, uint32_t *__restrict__ keep,
                                                uint2 *__restrict__ dirty, Ctrl *c) {
  if (c->err) return;
  const uint64_t p = *p_dev;                         // pending updates (device-side count)
  const int lane = threadIdx.x & 31;
  const uint32_t nsub = 32 / L, sub = lane / L, sl = lane % L;
  const uint32_t submask = (L == 32 ? 0xffffffffu : ((1u << L) - 1u) << (sub * L));
  const uint32_t below_me = (1u << sl) - 1u;
  const uint64_t nwarps = (uint64_t)gridDim.x * (blockDim.x / 32);
  const bool ins = op == GPMA_INSERT;
  uint32_t accepted = 0;
  for (uint64_t base = ((blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32) * 32; base < p;
       base += nwarps * 32) {
    const uint64_t jl = base + lane;
    const bool first = jl < p && (jl == 0 || pt[jl] != pt[jl - 1]);
    const uint32_t S = __ballot_sync(0xffffffffu, first);
    if (!S) continue;
    const uint32_t nstart = __popc(S);
    // end of the window's last group: warp-cooperative forward scan
    const uint32_t t_last = pt[base + (31 - __clz(S))];
    uint64_t last_end = base + 32;
    while (true) {
      const uint64_t jj = last_end + lane;
      const bool other = jj >= p || pt[jj] != t_last;
      const uint32_t bb = __ballot_sync(0xffffffffu, other);
      if (bb) { last_end += __ffs(bb) - 1; break; }
      last_end += 32;
    }
    if (last_end > p) last_end = p;
    for (uint32_t it = 0; it * nsub < nstart; ++it) {
      const uint32_t gi = it * nsub + sub;
      const bool have = gi < nstart;
      uint64_t j0 = 0, j1 = 0;
      if (have) {
        j0 = base + __fns(S, 0, gi + 1);
        j1 = gi + 1 < nstart ? base + __fns(S, 0, gi + 2) : last_end;
      }
      const uint32_t t = have ? pt[j0] : 0u;
      const uint32_t u = (uint32_t)(j1 - j0);
      const uint64_t lb = (uint64_t)t * L;
      uint64_t ks = KEY_NONE;
      uint32_t vs = 0;
      if (have) {
        ks = key[lb + sl];
        vs = val[lb + sl];
      }
      const bool live = have && ks != KEY_NONE && vs != VAL_TOMB;
      const uint32_t lbits = (__ballot_sync(0xffffffffu, live) & submask) >> (sub * L);
      const uint32_t n = __popc(lbits);
      const bool ok = have && (ins ? (u <= bound && n + u <= bound) : (u <= n && n - u >= bound));
      uint64_t uk = KEY_NONE;
      uint32_t uv = 0;
      if (ok && sl < u) {
        uk = pk[j0 + sl];
        uv = pv[j0 + sl];
      }
      // merged ranks: one round per update of the sub-warp (u <= max_0 when accepted; most
      // accepted leaves take a single update), the leaf side by one ballot per round
      uint32_t below_u = 0, below_l = 0;
      bool drop = false;
      const uint32_t umax = __reduce_max_sync(0xffffffffu, ok ? u : 0u);
      for (uint32_t i = 0; i < umax; ++i) {
        const bool vi = ok && i < u;                    // uniform within the sub-warp
        const uint64_t ui = __shfl_sync(0xffffffffu, uk, i, L);
        below_u += vi && ui < ks;
        const uint32_t bl = __popc((__ballot_sync(0xffffffffu, vi && live && ks < ui) & submask) >> (sub * L));
        if (sl == i) below_l = bl;
        drop |= !ins && live && vi && ui == ks;
      }
      const uint32_t N = ins ? n + u : n - u;
      const uint32_t live_rank = __popc(lbits & below_me);
      const uint32_t lpos = ins ? live_rank + below_u : live_rank - below_u;
      const uint32_t upos = sl + below_l;
      // new first key (held by the lane whose entry lands at 0) and the old one
      const bool l0 = live && !drop && lpos == 0;
      const bool u0 = ins && ok && sl < u && upos == 0;
      const uint32_t b0 = ((__ballot_sync(0xffffffffu, l0 || u0) & submask) >> (sub * L));
      const uint64_t h_new = __shfl_sync(0xffffffffu, l0 ? ks : uk, b0 ? __ffs(b0) - 1 : 0, L);
      const uint64_t h_old = __shfl_sync(0xffffffffu, ks, 0, L);
      __syncwarp();
      if (ok) {
        if (live && !drop) {
          key[lb + lpos] = ks;
          val[lb + lpos] = vs;
          if (is_guard_key(ks)) row_offset[(ks >> 32) - rb + 1] = lb + lpos;
        }
        if (ins && sl < u) {
          key[lb + upos] = uk;
          val[lb + upos] = uv;
        }
      }
      __syncwarp();
      if (ok && sl >= N) {
        key[lb + sl] = KEY_NONE;
        val[lb + sl] = 0;
      }
      if (have)
        for (uint64_t j = j0 + sl; j < j1; j += L) keep[j] = ok ? 0u : 1u;
      if (ok && sl == 0) {
        cnt[t] = N;
        tmask[t] = 0u;
        if (h_new != h_old && N) {
          head[t] = h_new;
          // empty leaves to the left carry this head (R9): leave them to the final fix-up
          if (t > 0 && key[lb - L] == KEY_NONE) {
            const uint64_t d = atomicAdd((unsigned long long *)&c->ndirty, 1ull);
            dirty[d] = make_uint2(t, 1u);
          }
        }
        if (!N) {   // an emptied leaf (strict delete with min_0 = 0): the fix-up recomputes it
          const uint64_t d = atomicAdd((unsigned long long *)&c->ndirty, 1ull);
          dirty[d] = make_uint2(t, 1u);
        }
        ++accepted;
      }
    }
  }
  accepted = __reduce_add_sync(0xffffffffu, accepted);
  if (lane == 0 && accepted) atomicAdd((unsigned long long *)&c->windows_rewritten, (unsigned long long)accepted);
}

__global__ void k_compact_pending(const uint32_t *__restrict__ keep, const uint32_t *__restrict__ pos,
                                  uint64_t n, const uint64_t *__restrict__ ik,
                                  const uint32_t *__restrict__ iv, const uint32_t *__restrict__ it,
                                  uint64_t *__restrict__ ok, uint32_t *__restrict__ ov,
                                  uint32_t *__restrict__ ot, const Ctrl *c) {
  if (c->err) return;
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    if (keep[i]) {
      uint32_t d = pos[i];
      ok[d] = ik[i];
      ov[d] = iv ? iv[i] : 0u;                      // (a delete batch is sorted keys-only)
      ot[d] = it[i];
    }
  }
}

// ------------------------------------------------------------------ level step
struct Lvl {
  const uint64_t *pk;
  const uint32_t *pv;
  const uint32_t *pt;
  uint64_t p;          // pending entering this level (host-known)
  uint32_t lvl;        // tree level i
  uint32_t L;
  uint32_t *hf, *widx, *wfirst, *acc, *aidx, *alist, *keep, *kpos;
  uint64_t *nw, *woff, *lpre;
  uint64_t *wk;        // scratch: merged windows, dense
  uint32_t *wv;
  uint64_t tmin, tmax;
  int op;
  int force;           // resize: accept the single root window unconditionally
  uint32_t rb;         // first owned row (row offsets are local)
  uint64_t nleaves;    // leaves of the store (offset of the guard counts after the masks)
  const uint32_t *lcnt; // small levels: leaf live counts read directly instead of the prefix lpre
  const uint32_t *sup;  // (nullable) windows the batch truly accepts, heap-indexed bits (superseded)
};

// A window (level l, index w) is superseded when a window above it is truly accepted (its test
// passes while updates of its chain are still pending -- k_lvl_root_reach marks them): that
// rewrite re-lays out all of it, so a lower rewrite inside it changes nothing and is skipped
// (its updates stay pending and are merged there).  Bits are heap-indexed: (l, w) -> (nl >> l) + w,
// the parent of id is id >> 1.
__device__ __forceinline__ bool lvl_superseded(const uint32_t *sup, uint64_t nl, uint32_t l, uint64_t w) {
  uint64_t id = (nl >> l) + w;
  for (id >>= 1; id >= 2; id >>= 1)                     // (id 1, the root, is never marked)
    if ((__ldg(sup + (id >> 5)) >> (id & 31)) & 1u) return true;
  return false;
}

__global__ void k_lvl_flags(Lvl a) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < a.p;
       j += (uint64_t)gridDim.x * blockDim.x)
    a.hf[j] = (j == 0 || (a.pt[j] >> a.lvl) != (a.pt[j - 1] >> a.lvl)) ? 1u : 0u;
}

__global__ void k_lvl_first(Lvl a) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < a.p;
       j += (uint64_t)gridDim.x * blockDim.x) {
    if (a.hf[j]) a.wfirst[a.widx[j]] = (uint32_t)j;
    if (j == 0) a.wfirst[a.widx[a.p]] = (uint32_t)a.p;
  }
}

// CountSegment + CountUpdatesInSegment + density test (Alg. 4 l.23-25).
// TPW threads per window sum the per-leaf live counts of the window.
template <int TPW>
__global__ void k_lvl_count(Lvl a, const uint32_t *__restrict__ cnt) {
  __shared__ uint64_t red[TB / 32];
  const uint32_t q = a.widx[a.p];
  const uint64_t groups_per_grid = (uint64_t)gridDim.x * (blockDim.x / TPW);
  const uint64_t g0 = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / TPW;
  const int r = threadIdx.x % TPW;
  const uint64_t nleaf_w = 1ull << a.lvl;
  // the loop trip count must be uniform inside a group
  for (uint64_t w = g0; w < a.p; w += groups_per_grid) {
    uint64_t n = 0;
    bool real = w < q;
    uint64_t leaf0 = 0;
    if (real) {
      leaf0 = ((uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)) << a.lvl;
      for (uint64_t l = r; l < nleaf_w; l += TPW) n += cnt[leaf0 + l];
    }
    if (TPW >= 32) {
      for (int o = 16; o; o >>= 1) n += __shfl_xor_sync(0xffffffffu, n, o);
      if (TPW > 32) {
        if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = n;
        __syncthreads();
        if (threadIdx.x == 0) {
          uint64_t s = 0;
          for (int k = 0; k < TPW / 32; ++k) s += red[k];
          red[0] = s;
        }
        __syncthreads();
        n = red[0];
        __syncthreads();
      }
    }
    if (r == 0) {
      if (!real) {
        a.acc[w] = 0;
        a.nw[w] = 0;
      } else {
        uint64_t u = a.wfirst[w + 1] - a.wfirst[w];
        bool ok;
        if (a.force) ok = true;
        else if (a.op == GPMA_INSERT) ok = n + u <= a.tmax;
        else ok = n >= u && n - u >= a.tmin;
        if (ok && !a.force && a.sup && lvl_superseded(a.sup, a.nleaves, a.lvl, leaf0 >> a.lvl)) ok = false;
        a.acc[w] = ok ? 1u : 0u;
        a.nw[w] = ok ? (a.op == GPMA_INSERT ? n + u : n - u) : 0;
      }
    }
  }
}

// High levels (few, huge windows): the window counts with every SM busy -- CTA (c, w) sums
// chunk c of window w's leaf counts into nw[w] (zeroed first); k_lvl_accept then applies the
// density test (Alg. 4 l.23-25, R5).  One CTA per window (k_lvl_count<TB>) left a 2^23-leaf
// root window to a single SM: 8.4 of a 34 ms resizing batch.
__global__ void __launch_bounds__(TB) k_lvl_count_wide(Lvl a, const uint32_t *__restrict__ cnt,
                                                        uint32_t chunk_leaves) {
  __shared__ uint64_t red[TB / 32];
  const uint32_t q = a.widx[a.p];
  const uint64_t w = blockIdx.y;
  if (w >= q) return;
  const uint64_t leaf0 = ((uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)) << a.lvl;
  const uint64_t c0 = (uint64_t)blockIdx.x * chunk_leaves;
  uint64_t n = 0;
  for (uint64_t l = c0 + threadIdx.x; l < c0 + chunk_leaves; l += TB) n += __ldg(cnt + leaf0 + l);
  for (int o = 16; o; o >>= 1) n += __shfl_xor_sync(0xffffffffu, n, o);
  if ((threadIdx.x & 31) == 0) red[threadIdx.x >> 5] = n;
  __syncthreads();
  if (threadIdx.x == 0) {
    uint64_t t = 0;
    for (int k = 0; k < TB / 32; ++k) t += red[k];
    if (t) atomicAdd((unsigned long long *)(a.nw + w), (unsigned long long)t);
  }
}

__global__ void k_lvl_accept(Lvl a) {
  const uint32_t q = a.widx[a.p];
  for (uint64_t w = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; w < a.p;
       w += (uint64_t)gridDim.x * blockDim.x) {
    if (w >= q) {
      a.acc[w] = 0;
      a.nw[w] = 0;
      continue;
    }
    const uint64_t n = a.nw[w];
    const uint64_t u = a.wfirst[w + 1] - a.wfirst[w];
    bool ok;
    if (a.force) ok = true;
    else if (a.op == GPMA_INSERT) ok = n + u <= a.tmax;
    else ok = n >= u && n - u >= a.tmin;
    if (ok && !a.force && a.sup && lvl_superseded(a.sup, a.nleaves, a.lvl, (uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)))
      ok = false;
    a.acc[w] = ok ? 1u : 0u;
    a.nw[w] = ok ? (a.op == GPMA_INSERT ? n + u : n - u) : 0;
  }
}

__global__ void k_lvl_alist(Lvl a) {
  for (uint64_t w = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; w < a.p;
       w += (uint64_t)gridDim.x * blockDim.x)
    if (a.acc[w]) a.alist[a.aidx[w]] = (uint32_t)w;
}

// live counts of the leaves of the accepted windows, flattened (then scanned)
__global__ void k_lvl_leafcnt(Lvl a, const uint32_t *__restrict__ cnt, uint64_t bound) {
  const uint32_t nacc = a.aidx[a.p];
  const uint64_t mask = (1ull << a.lvl) - 1;
  for (uint64_t g = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; g < bound;
       g += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t ai = g >> a.lvl;
    uint64_t v = 0;
    if (ai < nacc) {
      uint32_t w = a.alist[ai];
      uint64_t leaf0 = ((uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)) << a.lvl;
      v = cnt[leaf0 + (g & mask)];
    }
    a.lpre[g] = v;
  }
}

__device__ __forceinline__ uint64_t lower_bound_u64(const uint64_t *__restrict__ x, uint64_t lo,
                                                    uint64_t hi, uint64_t k) {
  while (lo < hi) {
    uint64_t mid = (lo + hi) >> 1;
    if (x[mid] < k) lo = mid + 1;
    else hi = mid;
  }
  return lo;
}

// Gather the live entries of every accepted window into the dense scratch list at
// their merged rank (Merge, Alg. 4 l.26).  Tombstones are dropped (R12).  Threads
// map to slots; a leaf never straddles a warp (L | 32), so ballots rank inside it.
__global__ void k_lvl_gather(Lvl a, const uint64_t *__restrict__ key, const uint32_t *__restrict__ val,
                             uint64_t bound_r) {
  const uint32_t nacc = a.aidx[a.p];
  const uint64_t wslots = (uint64_t)a.L << a.lvl;
  const uint32_t lgw = (uint32_t)(__ffs(a.L) - 1) + a.lvl;        // wslots is a power of two
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint32_t leafmask = (a.L == 32 ? 0xffffffffu : ((1u << a.L) - 1u) << (lane & ~(a.L - 1)));
  // only the accepted windows' slots (rounded to whole warps: the ballot below needs them)
  const uint64_t lim = min((uint64_t)bound_r, (uint64_t)((((uint64_t)nacc << lgw) + 31) & ~(uint64_t)31));
  for (uint64_t g = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; g < lim;
       g += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t ai = g >> lgw;
    bool valid = ai < nacc;
    uint64_t k = KEY_NONE, s = 0;
    uint32_t v = 0, w = 0;
    if (valid) {
      w = a.alist[ai];
      uint64_t seg = a.pt[a.wfirst[w]] >> a.lvl;
      s = seg * wslots + (g & (wslots - 1));
      k = key[s];
      v = val[s];
    }
    bool live = valid && k != KEY_NONE && v != VAL_TOMB;
    uint32_t bal = __ballot_sync(0xffffffffu, live);
    if (live) {
      uint64_t off = g & (wslots - 1);
      uint64_t lidx = leaf_div(off, a.L);
      uint64_t rl = __popc(bal & leafmask & lt);
      if (a.lvl) {
        if (a.lcnt) {                                  // <= 15 earlier leaves of a small window
          const uint64_t leaf0 = ((uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)) << a.lvl;
          for (uint64_t l = 0; l < lidx; ++l) rl += a.lcnt[leaf0 + l];
        } else {
          rl += a.lpre[(ai << a.lvl) + lidx] - a.lpre[ai << a.lvl];
        }
      }
      uint64_t ub = a.wfirst[w], ue = a.wfirst[w + 1];
      uint64_t c = lower_bound_u64(a.pk, ub, ue, k) - ub;
      uint64_t r;
      bool drop = false;
      if (a.op == GPMA_INSERT) {
        r = rl + c;
      } else {
        drop = (ub + c < ue) && a.pk[ub + c] == k;
        r = rl - c;
      }
      if (!drop) {
        uint64_t d = a.woff[w] + r;
        a.wk[d] = k;
        a.wv[d] = v;
      }
    }
  }
}

// The same gather for windows of >= GB_CHUNK slots (high levels, the root of a resize): a CTA
// takes one 4096-slot chunk of a window, finds the key range its occupied slots span, and stages
// the window's pending keys of that range (a contiguous run of the sorted list, found by two
// binary searches) in shared memory, so each live slot's rank among the pending keys is a search
// of a few shared-memory entries instead of ~log2(pending) dependent global probes (merge-path
// split of the window merge, Alg. 4 l.26).
constexpr int GB_T = 256, GB_I = 16, GB_CHUNK = GB_T * GB_I, GB_SP = 4096;
// CTAs in the big-window gather grid per SM (GPMA_GB_PER_SM; 4 resident): 16 short contiguous
// runs per SM balance the tail best (4 / 8 / 16: 2.35 / 2.31 / 2.23 ms for the configs[3] halving)
static int gb_per_sm() {
  const char *e = getenv("GPMA_GB_PER_SM");
  return e ? std::max(1, atoi(e)) : 16;
}

// first index in [lo, hi) with a[i] >= x (hi if none), all 32 lanes of a warp: 32 probes per
// round narrow the range 32-fold (4 rounds for 10^6 keys instead of 20 dependent probes)
__device__ __forceinline__ uint64_t warp_lower_bound_u64(const uint64_t *__restrict__ a, uint64_t lo, uint64_t hi,
                                                         uint64_t x) {
  const int lane = threadIdx.x & 31;
  while (hi - lo > 32) {
    const uint64_t step = (hi - lo + 31) / 32;
    const uint64_t idx = lo + (uint64_t)lane * step;
    const bool ge = idx >= hi || a[idx] >= x;            // (past the range counts as >= x)
    const uint32_t m = __ballot_sync(0xffffffffu, ge);
    if (m & 1u) return lo;                               // a[lo] >= x
    if (m == 0) {                                        // every probe < x: past the last one
      lo = lo + 31 * step + 1;
    } else {
      const int f = __ffs(m) - 1;                        // answer in (probe f-1, probe f]
      const uint64_t pf = lo + (uint64_t)f * step;
      lo = lo + (uint64_t)(f - 1) * step + 1;
      hi = min(hi, pf);
    }
  }
  const uint64_t idx = lo + lane;
  const bool ge = idx >= hi || a[idx] >= x;
  const uint32_t m = __ballot_sync(0xffffffffu, ge);
  return m ? min(hi, lo + (uint64_t)(__ffs(m) - 1)) : hi;
}
__global__ void __launch_bounds__(GB_T, 4) k_lvl_gather_big(Lvl a, const uint64_t *__restrict__ key,
                                                          const uint32_t *__restrict__ val, uint64_t nchunks) {
  __shared__ uint64_t sp[GB_SP];
  __shared__ uint64_t slp[GB_CHUNK / 4];                // the chunk's leaf prefixes (L >= 4)
  __shared__ uint64_t red_min[GB_T / 32], red_max[GB_T / 32];
  __shared__ uint64_t s_pa, s_pb, s_lbase;
  const uint32_t nacc = a.aidx[a.p];
  const uint32_t lgw = (uint32_t)(__ffs(a.L) - 1) + a.lvl;       // window slots = 2^lgw
  const uint64_t cpw = (1ull << lgw) / GB_CHUNK;                  // chunks per window
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  const uint32_t lt = (1u << lane) - 1u;
  const uint32_t leafmask = (a.L == 32 ? 0xffffffffu : ((1u << a.L) - 1u) << (lane & ~(a.L - 1)));
  // a CTA walks a contiguous run of chunks: the next chunk's pending run starts at or after the
  // previous one's end (keys ascend with the slot), so its searches begin there (usually one probe)
  const uint64_t cpc = (nchunks + gridDim.x - 1) / gridDim.x;
  const uint64_t c1 = min(nchunks, (blockIdx.x + 1) * cpc);
  uint64_t prev = 0;
  uint32_t prev_w = 0xffffffffu;
  for (uint64_t ch = blockIdx.x * cpc; ch < c1; ++ch) {   // block-uniform
    const uint64_t ai = ch / cpw;
    if (ai >= nacc) break;
    const uint32_t w = a.alist[ai];
    const uint64_t seg = a.pt[a.wfirst[w]] >> a.lvl;
    const uint64_t off0 = (ch % cpw) * GB_CHUNK;                  // chunk offset in the window
    const uint64_t s0 = seg * (1ull << lgw) + off0;
    uint64_t k[GB_I];
    uint32_t v[GB_I];
    uint64_t kmin = KEY_NONE, kmax = 0;
    bool anyocc = false;
    {                                                    // leaf prefixes: issued with the slot loads
      const uint64_t lp0 = (ai << a.lvl) + leaf_div(off0, a.L);
      const uint32_t nlc = GB_CHUNK / a.L;
      for (uint32_t j = threadIdx.x; j < nlc; j += GB_T) slp[j] = a.lpre[lp0 + j];
      if (threadIdx.x == 0) s_lbase = a.lpre[ai << a.lvl];
    }
#pragma unroll
    for (int i = 0; i < GB_I; ++i) {
      const uint64_t s = s0 + (uint64_t)i * GB_T + threadIdx.x;
      k[i] = key[s];
      v[i] = val[s];
      if (k[i] != KEY_NONE) {
        kmin = min(kmin, k[i]);
        kmax = max(kmax, k[i]);
        anyocc = true;
      }
    }
    for (int o = 16; o; o >>= 1) {
      kmin = min(kmin, __shfl_xor_sync(0xffffffffu, kmin, o));
      kmax = max(kmax, __shfl_xor_sync(0xffffffffu, kmax, o));
    }
    anyocc = __any_sync(0xffffffffu, anyocc);
    if (lane == 0) {
      red_min[warp] = kmin;
      red_max[warp] = anyocc ? kmax : 0;
    }
    __syncthreads();
    const uint64_t ub = a.wfirst[w], ue = a.wfirst[w + 1];
    const uint64_t lo0 = w == prev_w ? prev : ub;
    if (warp < 2) {                                      // the chunk's pending run: warp 0 finds its
      uint64_t mn = KEY_NONE, mx = 0;                    // start, warp 1 its end (concurrently)
      for (int q = 0; q < GB_T / 32; ++q) {
        mn = min(mn, red_min[q]);
        mx = max(mx, red_max[q]);
      }
      uint64_t r = lo0;
      if (mn != KEY_NONE) {
        const uint64_t x = warp == 0 ? mn : mx + 1;
        const uint64_t idx = lo0 + lane;
        const uint64_t pv = idx < ue ? a.pk[idx] : KEY_NONE;
        const uint32_t m = __ballot_sync(0xffffffffu, idx >= ue || pv >= x);
        r = m ? min(ue, lo0 + (uint64_t)(__ffs(m) - 1)) : warp_lower_bound_u64(a.pk, lo0 + 32, ue, x);
        if (warp == 1) sp[lane] = pv;                    // pk[lo0 .. lo0 + 32): the usual whole run
      }
      if (lane == 0) (warp == 0 ? s_pa : s_pb) = r;
    }
    __syncthreads();
    const uint64_t pa = s_pa, pb = s_pb;
    uint64_t base = lo0;                                 // sp[j - base] = pk[j] for j in [pa, pb)
    bool staged = pb - lo0 <= 32;
    if (!staged && pb - pa <= (uint64_t)GB_SP) {        // (overwrites the probe values)
      for (uint64_t j = pa + threadIdx.x; j < pb; j += GB_T) sp[j - pa] = a.pk[j];
      base = pa;
      staged = true;
      __syncthreads();
    }
    uint64_t cmn = KEY_NONE;
    for (int q = 0; q < GB_T / 32; ++q) cmn = min(cmn, red_min[q]);
    if (cmn != KEY_NONE) {                               // an occupied chunk moves the run start
      prev = pb;
      prev_w = w;
    }
#pragma unroll
    for (int i = 0; i < GB_I; ++i) {
      const bool live = k[i] != KEY_NONE && v[i] != VAL_TOMB;
      const uint32_t bal = __ballot_sync(0xffffffffu, live);
      if (!live) continue;
      const uint64_t rl = __popc(bal & leafmask & lt) + (slp[leaf_div((uint64_t)i * GB_T + threadIdx.x, a.L)] - s_lbase);
      uint64_t c;                                        // pending keys < k[i] in the window
      if (staged) {
        uint64_t lo = pa - base, hi = pb - base;
        while (lo < hi) {
          const uint64_t mid = (lo + hi) >> 1;
          if (sp[mid] < k[i]) lo = mid + 1;
          else hi = mid;
        }
        c = base - ub + lo;
      } else {
        c = lower_bound_u64(a.pk, pa, pb, k[i]) - ub;
      }
      uint64_t r;
      bool drop = false;
      if (a.op == GPMA_INSERT) {
        r = rl + c;
      } else {                                           // (pk[pb] > every key of the chunk)
        drop = ub + c < pb && (staged ? sp[ub + c - base] : a.pk[ub + c]) == k[i];
        r = rl - c;
      }
      if (!drop) {
        const uint64_t d = a.woff[w] + r;
        a.wk[d] = k[i];
        a.wv[d] = v[i];
      }
    }
    __syncthreads();                                     // sp / red reused by the next chunk
  }
}

// Place the pending insertions of accepted windows at their merged rank.
__global__ void k_lvl_place(Lvl a, const uint64_t *__restrict__ key, const uint32_t *__restrict__ val) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < a.p;
       j += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t w = a.widx[j] + a.hf[j] - 1;
    if (!a.acc[w]) continue;
    uint64_t ai = a.aidx[w];
    uint32_t t = a.pt[j];
    uint64_t k = a.pk[j];
    uint64_t seg = t >> a.lvl;
    uint64_t lidx = t - (seg << a.lvl);
    uint64_t rl = 0;
    if (a.lvl) {
      if (a.lcnt) {                                    // small window: sum the earlier leaves
        for (uint64_t l = 0; l < lidx; ++l) rl += a.lcnt[(seg << a.lvl) + l];
      } else {
        rl = a.lpre[(ai << a.lvl) + lidx] - a.lpre[ai << a.lvl];
      }
    }
    uint64_t base = (uint64_t)t * a.L;
    for (uint32_t p = 0; p < a.L; ++p) {
      uint64_t x = key[base + p];
      if (x == KEY_NONE || x > k) break;
      if (val[base + p] != VAL_TOMB) ++rl;
    }
    uint64_t d = a.woff[w] + (j - a.wfirst[w]) + rl;
    a.wk[d] = k;
    a.wv[d] = a.pv[j];
  }
}

// Re-dispatch evenly (Alg. 4 l.27, R7): leaf l of a window with Lc leaves and N
// entries receives entries [floor(l N / Lc), floor((l+1) N / Lc)), left-packed.
// Guards moved here update the row offsets (R8).
__global__ void k_lvl_redistribute(Lvl a, uint64_t *__restrict__ key, uint32_t *__restrict__ val,
                                   uint32_t *__restrict__ cnt, uint32_t *__restrict__ tmask,
                                   uint64_t *__restrict__ row_offset, uint64_t bound,
                                   uint2 *__restrict__ dirty, uint64_t dirty_base) {
  // 4 consecutive slots of one leaf per thread (L >= 4), stored as 16-B vectors; leaf bounds by
  // shifts (Lc = 2^lvl leaves per window)
  const uint32_t nacc = a.aidx[a.p];
  const uint64_t wslots = (uint64_t)a.L << a.lvl;
  const uint32_t lgL = (uint32_t)(__ffs(a.L) - 1);
  const uint32_t lgw = lgL + a.lvl;                              // wslots is a power of two
  const uint64_t lim = min(bound, (uint64_t)nacc << lgw) / 4;    // the accepted windows' slots only
  for (uint64_t g4 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; g4 < lim;
       g4 += (uint64_t)gridDim.x * blockDim.x) {
    const uint64_t g = g4 * 4;
    const uint64_t ai = g >> lgw;
    if (ai >= nacc) continue;
    const uint32_t w = a.alist[ai];
    const uint64_t N = a.nw[w];
    const uint64_t leaf0 = ((uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)) << a.lvl;
    const uint64_t off = g & (wslots - 1);
    const uint64_t l = off >> lgL, p = off & (a.L - 1);
    const uint64_t lo = (l * N) >> a.lvl, hi = ((l + 1) * N) >> a.lvl, m = hi - lo;
    const uint64_t s = leaf0 * a.L + off;
    const uint64_t e0 = a.woff[w] + lo + p;
    uint64_t k[4];
    uint32_t v[4];
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      if (p + q < m) {
        k[q] = a.wk[e0 + q];
        v[q] = a.wv[e0 + q];
        if (is_guard_key(k[q])) row_offset[(k[q] >> 32) - a.rb + 1] = s + q;
      } else {
        k[q] = KEY_NONE;
        v[q] = 0;
      }
    }
    *reinterpret_cast<ulonglong2 *>(key + s) = make_ulonglong2(k[0], k[1]);
    *reinterpret_cast<ulonglong2 *>(key + s + 2) = make_ulonglong2(k[2], k[3]);
    *reinterpret_cast<uint4 *>(val + s) = make_uint4(v[0], v[1], v[2], v[3]);
    if (p == 0) {
      cnt[leaf0 + l] = (uint32_t)m;
      tmask[leaf0 + l] = 0u;                          // tombstones are dropped by a rewrite
      uint32_t gc = 0;
      for (uint64_t e = lo; e < hi; ++e) gc += is_guard_key(a.wk[a.woff[w] + e]);
      tmask[a.nleaves + leaf0 + l] = gc;              // guards per leaf (third section)
    }
    if (off == 0) dirty[dirty_base + ai] = make_uint2((uint32_t)leaf0, (uint32_t)(1ull << a.lvl));
  }
}

// Small levels (windows of <= 16 leaves, <= 512 slots): gather + placement + even
// re-dispatch of one accepted window in one CTA, the merged list staged in shared memory
// instead of the HBM scratch (Alg. 4 l.26-27, R7) -- the three kernels above fused.
constexpr int LM_T = 256, LM_MAXS = 512;
__global__ void __launch_bounds__(LM_T) k_lvl_merge_small(Lvl a, uint64_t *__restrict__ key, uint32_t *__restrict__ val,
                                                          uint32_t *__restrict__ cnt, uint32_t *__restrict__ tmask,
                                                          uint64_t *__restrict__ row_offset, uint2 *__restrict__ dirty,
                                                          uint64_t dirty_base) {
  __shared__ uint64_t mk[LM_MAXS];
  __shared__ uint32_t mv[LM_MAXS];
  __shared__ uint32_t lpre[17];
  const uint32_t nacc = a.aidx[a.p];
  const uint32_t ai = blockIdx.x;
  if (ai >= nacc) return;                              // uniform: the whole CTA leaves
  const uint32_t w = a.alist[ai];
  const uint32_t Lc = 1u << a.lvl;
  const uint32_t ws = a.L << a.lvl;
  const uint64_t leaf0 = ((uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)) << a.lvl;
  const uint64_t N = a.nw[w];
  const uint64_t ub = a.wfirst[w], ue = a.wfirst[w + 1];
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint32_t leafmask = (a.L == 32 ? 0xffffffffu : ((1u << a.L) - 1u) << (lane & ~(a.L - 1)));
  if (threadIdx.x == 0) {                              // live entries before each leaf
    uint32_t acc = 0;
    for (uint32_t l = 0; l < Lc; ++l) {
      lpre[l] = acc;
      acc += cnt[leaf0 + l];
    }
    lpre[Lc] = acc;
  }
  __syncthreads();
  for (uint32_t o0 = 0; o0 < ws; o0 += LM_T) {         // gather the live entries (whole warps)
    const uint32_t off = o0 + threadIdx.x;
    const bool in = off < ws;
    uint64_t k = KEY_NONE;
    uint32_t v = 0;
    if (in) {
      k = key[leaf0 * a.L + off];
      v = val[leaf0 * a.L + off];
    }
    const bool live = in && k != KEY_NONE && v != VAL_TOMB;
    const uint32_t bal = __ballot_sync(0xffffffffu, live);
    if (live) {
      const uint64_t rl = __popc(bal & leafmask & lt) + lpre[leaf_div(off, a.L)];
      const uint64_t c = lower_bound_u64(a.pk, ub, ue, k) - ub;
      bool drop = false;
      uint64_t r;
      if (a.op == GPMA_INSERT) {
        r = rl + c;
      } else {
        drop = (ub + c < ue) && a.pk[ub + c] == k;
        r = rl - c;
      }
      if (!drop) {
        mk[r] = k;
        mv[r] = v;
      }
    }
  }
  if (a.op == GPMA_INSERT) {                           // place the window's insertions
    for (uint64_t j = ub + threadIdx.x; j < ue; j += LM_T) {
      const uint64_t k = a.pk[j];
      const uint32_t t = a.pt[j];
      uint64_t rl = lpre[t - leaf0];
      const uint64_t base = (uint64_t)t * a.L;
      for (uint32_t q = 0; q < a.L; ++q) {
        const uint64_t x = key[base + q];
        if (x == KEY_NONE || x > k) break;
        if (val[base + q] != VAL_TOMB) ++rl;
      }
      const uint64_t r = (j - ub) + rl;
      mk[r] = k;
      mv[r] = a.pv[j];
    }
  }
  __syncthreads();                                     // every read of the window is done
  for (uint32_t off = threadIdx.x; off < ws; off += LM_T) {   // re-dispatch evenly (R7)
    const uint64_t l = leaf_div(off, a.L), q = leaf_mod(off, a.L);
    const uint64_t lo = l * N / Lc, hi = (l + 1) * N / Lc;
    const uint64_t sl = leaf0 * a.L + off;
    if (q < hi - lo) {
      const uint64_t k = mk[lo + q];
      key[sl] = k;
      val[sl] = mv[lo + q];
      if (is_guard_key(k)) row_offset[(k >> 32) - a.rb + 1] = sl;
    } else {
      key[sl] = KEY_NONE;
      val[sl] = 0;
    }
    if (q == 0) {
      cnt[leaf0 + l] = (uint32_t)(hi - lo);
      tmask[leaf0 + l] = 0u;                          // tombstones are dropped by a rewrite
      uint32_t gc = 0;
      for (uint64_t e = lo; e < hi; ++e) gc += is_guard_key(mk[e]);
      tmask[a.nleaves + leaf0 + l] = gc;              // guards per leaf (third section)
    }
  }
  if (threadIdx.x == 0) dirty[dirty_base + ai] = make_uint2((uint32_t)leaf0, Lc);
}

__global__ void k_lvl_keep(Lvl a) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < a.p;
       j += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t w = a.widx[j] + a.hf[j] - 1;
    a.keep[j] = a.acc[w] ? 0u : 1u;
  }
}

// ---- small levels (p <= 4096 pending, windows of <= 64 leaves): one CTA runs the
// segment / count / accept front (UniqueSegments, CountSegment, density test, the accepted
// list: 7 launches) and another the keep / compaction-offset / summary back (3 launches).
// Above level 0 the pending lists are small and every launch is a few us of pure overhead.
constexpr int LS_T = 1024, LS_I = 4;
constexpr uint64_t LS_MAXP = (uint64_t)LS_T * LS_I;
constexpr uint32_t LS_MAXLVL = 4;                     // windows of <= 16 leaves: counted in-thread

// exclusive scan of 4 consecutive items per thread over the CTA; returns the total
__device__ __forceinline__ uint64_t ls_scan4(uint64_t v[LS_I], uint64_t *wsum) {
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint64_t ex[LS_I];
  uint64_t t = 0;
#pragma unroll
  for (int i = 0; i < LS_I; ++i) {
    ex[i] = t;
    t += v[i];
  }
  uint64_t x = t;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const uint64_t y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  if (lane == 31) wsum[warp] = x;
  __syncthreads();
  if (warp == 0) {
    uint64_t w = wsum[lane];
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint64_t y = __shfl_up_sync(0xffffffffu, w, o);
      if (lane >= o) w += y;
    }
    wsum[lane] = w;
  }
  __syncthreads();
  const uint64_t base = (warp ? wsum[warp - 1] : 0) + x - t;
  const uint64_t total = wsum[31];
  __syncthreads();                                     // wsum is reused by the next scan
#pragma unroll
  for (int i = 0; i < LS_I; ++i) v[i] = base + ex[i];
  return total;
}

__global__ void __launch_bounds__(LS_T) k_lvl_front_small(Lvl a, const uint32_t *__restrict__ cnt) {
  __shared__ uint64_t wsum[32];
  const uint64_t p = a.p;
  const uint64_t j0 = (uint64_t)threadIdx.x * LS_I;
  uint64_t f[LS_I];
#pragma unroll
  for (int i = 0; i < LS_I; ++i) {                     // window-head flags (l.18-21: RLE)
    const uint64_t j = j0 + i;
    f[i] = (j < p && (j == 0 || (a.pt[j] >> a.lvl) != (a.pt[j - 1] >> a.lvl))) ? 1u : 0u;
    if (j < p) a.hf[j] = (uint32_t)f[i];
  }
  uint64_t e[LS_I] = {f[0], f[1], f[2], f[3]};
  const uint64_t q = ls_scan4(e, wsum);                // windows
#pragma unroll
  for (int i = 0; i < LS_I; ++i) {
    const uint64_t j = j0 + i;
    if (j < p) {
      a.widx[j] = (uint32_t)e[i];
      if (f[i]) a.wfirst[e[i]] = (uint32_t)j;
    }
  }
  if (threadIdx.x == 0) {
    a.widx[p] = (uint32_t)q;
    a.wfirst[q] = (uint32_t)p;
  }
  __syncthreads();
  uint64_t ac[LS_I], nw[LS_I];
#pragma unroll
  for (int i = 0; i < LS_I; ++i) {                     // count + density test (l.23-25, R5)
    const uint64_t w = j0 + i;
    ac[i] = nw[i] = 0;
    if (w < q) {
      const uint64_t leaf0 = ((uint64_t)(a.pt[a.wfirst[w]] >> a.lvl)) << a.lvl;
      uint64_t n = 0;
#pragma unroll
      for (uint32_t l = 0; l < (1u << LS_MAXLVL); ++l)   // independent loads, all in flight
        if (l < (1u << a.lvl)) n += cnt[leaf0 + l];
      const uint64_t u = a.wfirst[w + 1] - a.wfirst[w];
      bool ok;
      if (a.force) ok = true;
      else if (a.op == GPMA_INSERT) ok = n + u <= a.tmax;
      else ok = n >= u && n - u >= a.tmin;
      if (ok && !a.force && a.sup && lvl_superseded(a.sup, a.nleaves, a.lvl, leaf0 >> a.lvl)) ok = false;
      ac[i] = ok ? 1u : 0u;
      nw[i] = ok ? (a.op == GPMA_INSERT ? n + u : n - u) : 0;
    }
    if (w < p) {
      a.acc[w] = (uint32_t)ac[i];
      a.nw[w] = nw[i];
    }
  }
  uint64_t ai[LS_I] = {ac[0], ac[1], ac[2], ac[3]};
  const uint64_t nacc = ls_scan4(ai, wsum);
  const uint64_t tot = ls_scan4(nw, wsum);
#pragma unroll
  for (int i = 0; i < LS_I; ++i) {
    const uint64_t w = j0 + i;
    if (w < p) {
      a.aidx[w] = (uint32_t)ai[i];
      a.woff[w] = nw[i];
      if (ac[i]) a.alist[ai[i]] = (uint32_t)w;
    }
  }
  if (threadIdx.x == 0) {
    a.aidx[p] = (uint32_t)nacc;
    a.woff[p] = tot;
  }
}

__global__ void __launch_bounds__(LS_T) k_lvl_back_small(Lvl a, Ctrl *c) {
  __shared__ uint64_t wsum[32];
  const uint64_t p = a.p;
  const uint64_t j0 = (uint64_t)threadIdx.x * LS_I;
  uint64_t k[LS_I];
#pragma unroll
  for (int i = 0; i < LS_I; ++i) {                     // promote the rejected (l.12-15)
    const uint64_t j = j0 + i;
    k[i] = 0;
    if (j < p) {
      const uint32_t w = a.widx[j] + a.hf[j] - 1;
      k[i] = a.acc[w] ? 0u : 1u;
      a.keep[j] = (uint32_t)k[i];
    }
  }
  const uint64_t tot = ls_scan4(k, wsum);
#pragma unroll
  for (int i = 0; i < LS_I; ++i)
    if (j0 + i < p) a.kpos[j0 + i] = (uint32_t)k[i];
  if (threadIdx.x == 0) {
    a.kpos[p] = (uint32_t)tot;
    c->sum = (uint64_t)a.widx[p] | ((uint64_t)a.aidx[p] << 32);
    c->sum2 = tot;
  }
}

__global__ void k_lvl_summary(Lvl a, Ctrl *c) {
  // sum  = unique windows | accepted windows << 32 ; sum2 = pending after this level
  c->sum = (uint64_t)a.widx[a.p] | ((uint64_t)a.aidx[a.p] << 32);
  c->sum2 = a.kpos[a.p];
}

// ---- device-resident level loop (Alg. 4 l.4-15 above the leaves) ----------------------------
// One cooperative kernel runs levels 1, 2, ... on the device while the windows fit a CTA's
// shared memory (<= CL_MAXS slots, TryInsert+ at block scale): per level, the
// segments (UniqueSegments = RLE + a grid-wide scan, l.18-21), a warp per window counts and
// tests it (CountSegment + density, l.23-25), a CTA per accepted window merges and re-dispatches
// it in shared memory (l.26-27, R7), the rest is promoted by a second grid-wide scan (l.12-15) --
// grid-wide barriers between the phases instead of a host round trip per level.  It stops at the
// first level whose windows are larger; the host continues from there (the root resize).
constexpr int CL_T = 512, CL_I = 16;
constexpr uint32_t CL_MAXS = 4096;                   // slots of the largest window (48 KiB of keys + values)

struct CoopState {
  uint64_t p;                  // pending entering the level
  uint32_t cur, lvl, done, q;  // pending buffer, level, stop flag, windows of the level
  uint64_t windows, slots;     // rewritten by this kernel
  uint32_t top;                // highest level that ran
};

struct CoopArgs {
  uint64_t *pk[2];
  uint32_t *pv[2], *pt[2];
  uint32_t *hf, *widx, *wfirst, *acc, *keep, *kpos;
  uint64_t *nw;
  uint64_t *ctot;              // [gridDim] chunk totals of the grid-wide scans
  uint64_t *key;
  uint32_t *val, *cnt, *tmask;
  uint64_t *row_offset;
  uint2 *dirty;
  uint64_t nleaves;
  uint32_t L, h, rb;
  int op;
  int warp_merge;              // small windows merged by a warp (GPMA_LVL_WARP, default on)
  uint64_t tmin[48], tmax[48];
  CoopState *st;
  Ctrl *c;
};

// exclusive scan of CL_I consecutive items per thread over the CTA; returns the total
__device__ __forceinline__ uint64_t cl_scan(uint64_t (&v)[CL_I], uint64_t *wsum) {
  const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
  uint64_t ex[CL_I];
  uint64_t t = 0;
#pragma unroll
  for (int i = 0; i < CL_I; ++i) {
    ex[i] = t;
    t += v[i];
  }
  uint64_t x = t;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const uint64_t y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  if (lane == 31) wsum[warp] = x;
  __syncthreads();
  if (warp == 0) {
    uint64_t w = lane < CL_T / 32 ? wsum[lane] : 0;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint64_t y = __shfl_up_sync(0xffffffffu, w, o);
      if (lane >= o) w += y;
    }
    if (lane < CL_T / 32) wsum[lane] = w;
  }
  __syncthreads();
  const uint64_t base = (warp ? wsum[warp - 1] : 0) + x - t;
  const uint64_t total = wsum[CL_T / 32 - 1];
  __syncthreads();
#pragma unroll
  for (int i = 0; i < CL_I; ++i) v[i] = base + ex[i];
  return total;
}

// Grid-wide exclusive scan of the 0/1 flags f(j), j < p (every CTA takes a contiguous chunk;
// chunk scans, one barrier, the CTA totals' prefix, one barrier): out[j] = the prefix, returns the
// total on every CTA.  flag_out (optional) receives the flags.
template <class F>
__device__ uint64_t cl_grid_scan(cooperative_groups::grid_group &grid, uint64_t p, const F &f, uint32_t *out,
                                 uint32_t *flag_out, uint64_t *ctot, uint64_t *wsum) {
  const uint64_t per = (p + gridDim.x - 1) / gridDim.x;
  const uint64_t b0 = min(p, (uint64_t)blockIdx.x * per), b1 = min(p, b0 + per);
  uint64_t carry = 0;
  for (uint64_t t0 = b0; t0 < b1; t0 += (uint64_t)CL_T * CL_I) {       // block-uniform
    uint64_t v[CL_I], fl[CL_I];
#pragma unroll
    for (int i = 0; i < CL_I; ++i) {
      const uint64_t j = t0 + (uint64_t)threadIdx.x * CL_I + i;
      fl[i] = j < b1 ? f(j) : 0u;
      v[i] = fl[i];
    }
    const uint64_t tot = cl_scan(v, wsum);
#pragma unroll
    for (int i = 0; i < CL_I; ++i) {
      const uint64_t j = t0 + (uint64_t)threadIdx.x * CL_I + i;
      if (j < b1) {
        out[j] = (uint32_t)(carry + v[i]);
        if (flag_out) flag_out[j] = (uint32_t)fl[i];
      }
    }
    carry += tot;
  }
  if (threadIdx.x == 0) ctot[blockIdx.x] = carry;
  grid.sync();
  uint64_t pre = 0, all = 0;
  for (uint32_t k = threadIdx.x; k < gridDim.x; k += CL_T) {
    const uint64_t x = ctot[k];
    all += x;
    if (k < blockIdx.x) pre += x;
  }
  for (int o = 16; o; o >>= 1) {
    pre += __shfl_xor_sync(0xffffffffu, pre, o);
    all += __shfl_xor_sync(0xffffffffu, all, o);
  }
  __shared__ uint64_t s_pre[CL_T / 32], s_all[CL_T / 32];
  if ((threadIdx.x & 31) == 0) {
    s_pre[threadIdx.x >> 5] = pre;
    s_all[threadIdx.x >> 5] = all;
  }
  __syncthreads();
  pre = 0;
  all = 0;
  for (int k = 0; k < CL_T / 32; ++k) {
    pre += s_pre[k];
    all += s_all[k];
  }
  __syncthreads();
  if (pre)
    for (uint64_t j = b0 + threadIdx.x; j < b1; j += CL_T) out[j] += (uint32_t)pre;
  return all;
}

// the segments of level lvl over the pending list of buffer cur: hf, widx, wfirst; returns q
__device__ uint64_t cl_segments(cooperative_groups::grid_group &grid, const CoopArgs &a, uint64_t p, uint32_t cur,
                                uint32_t lvl, uint64_t *wsum) {
  const uint32_t *pt = a.pt[cur];
  const auto f = [&](uint64_t j) -> uint64_t {
    return (j == 0 || (pt[j] >> lvl) != (pt[j - 1] >> lvl)) ? 1u : 0u;
  };
  const uint64_t q = cl_grid_scan(grid, p, f, a.widx, a.hf, a.ctot, wsum);
  grid.sync();                                           // widx / hf complete
  for (uint64_t j = blockIdx.x * (uint64_t)CL_T + threadIdx.x; j < p; j += (uint64_t)gridDim.x * CL_T)
    if (a.hf[j]) a.wfirst[a.widx[j]] = (uint32_t)j;
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    a.widx[p] = (uint32_t)q;
    a.wfirst[q] = (uint32_t)p;
  }
  return q;
}

// promote the rejected updates of the level to the other buffer (l.12-15); returns the count
__device__ uint64_t cl_promote(cooperative_groups::grid_group &grid, const CoopArgs &a, uint64_t p, uint32_t cur,
                               uint64_t *wsum) {
  const auto f = [&](uint64_t j) -> uint64_t { return a.acc[a.widx[j] + a.hf[j] - 1] ? 0u : 1u; };
  const uint64_t pn = cl_grid_scan(grid, p, f, a.kpos, nullptr, a.ctot, wsum);
  grid.sync();                                           // kpos complete
  for (uint64_t j = blockIdx.x * (uint64_t)CL_T + threadIdx.x; j < p; j += (uint64_t)gridDim.x * CL_T)
    if (!a.acc[a.widx[j] + a.hf[j] - 1]) {
      const uint32_t d = a.kpos[j];
      a.pk[cur ^ 1][d] = a.pk[cur][j];
      a.pv[cur ^ 1][d] = a.pv[cur][j];
      a.pt[cur ^ 1][d] = a.pt[cur][j];
    }
  return pn;
}

// one accepted window merged and re-dispatched in shared memory (CTA-wide, Alg. 4 l.26-27)
__device__ void cl_merge_window(const CoopArgs &a, uint32_t cur, uint32_t lvl, uint32_t w, uint64_t *mk, uint32_t *mv,
                                uint32_t *lpre) {
  const uint32_t L = a.L;
  const uint64_t *pk = a.pk[cur];
  const uint32_t *pv = a.pv[cur], *pt = a.pt[cur];
  const uint32_t Lc = 1u << lvl, ws = L << lvl;
  const uint64_t leaf0 = ((uint64_t)(pt[a.wfirst[w]] >> lvl)) << lvl;
  const uint64_t N = a.nw[w];
  const uint64_t ub = a.wfirst[w], ue = a.wfirst[w + 1];
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint32_t leafmask = (L == 32 ? 0xffffffffu : ((1u << L) - 1u) << (lane & ~(L - 1)));
  // live entries before each leaf of the window (Lc <= CL_MAXS / 4)
  if (threadIdx.x < 32) {
    uint32_t carry = 0;
    for (uint32_t l0 = 0; l0 < Lc; l0 += 32) {
      const uint32_t l = l0 + lane;
      const uint32_t c0 = l < Lc ? a.cnt[leaf0 + l] : 0u;
      uint32_t x = c0;
#pragma unroll
      for (int o = 1; o < 32; o <<= 1) {
        const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
        if (lane >= o) x += y;
      }
      if (l < Lc) lpre[l] = carry + x - c0;
      carry += __shfl_sync(0xffffffffu, x, 31);
    }
    if (lane == 0) lpre[Lc] = carry;
  }
  __syncthreads();
  for (uint32_t o0 = 0; o0 < ws; o0 += CL_T) {           // gather the live entries (whole warps)
    const uint32_t off = o0 + threadIdx.x;
    const bool in = off < ws;
    uint64_t k = KEY_NONE;
    uint32_t v = 0;
    if (in) {
      k = a.key[leaf0 * L + off];
      v = a.val[leaf0 * L + off];
    }
    const bool live = in && k != KEY_NONE && v != VAL_TOMB;
    const uint32_t bal = __ballot_sync(0xffffffffu, live);
    if (live) {
      const uint64_t rl = __popc(bal & leafmask & lt) + lpre[leaf_div(off, L)];
      const uint64_t cc = lower_bound_u64(pk, ub, ue, k) - ub;
      bool drop = false;
      uint64_t r;
      if (a.op == GPMA_INSERT) {
        r = rl + cc;
      } else {
        drop = (ub + cc < ue) && pk[ub + cc] == k;
        r = rl - cc;
      }
      if (!drop) {
        mk[r] = k;
        mv[r] = v;
      }
    }
  }
  if (a.op == GPMA_INSERT) {                             // place the window's insertions
    for (uint64_t j = ub + threadIdx.x; j < ue; j += CL_T) {
      const uint64_t k = pk[j];
      const uint32_t t = pt[j];
      uint64_t rl = lpre[t - leaf0];
      const uint64_t base = (uint64_t)t * L;
      for (uint32_t q = 0; q < L; ++q) {
        const uint64_t x = a.key[base + q];
        if (x == KEY_NONE || x > k) break;
        if (a.val[base + q] != VAL_TOMB) ++rl;
      }
      const uint64_t r = (j - ub) + rl;
      mk[r] = k;
      mv[r] = pv[j];
    }
  }
  __syncthreads();                                       // every read of the window is done
  for (uint32_t off = threadIdx.x; off < ws; off += CL_T) {   // re-dispatch evenly (R7)
    const uint64_t l = leaf_div(off, L), q = leaf_mod(off, L);
    const uint64_t lo = l * N / Lc, hi = (l + 1) * N / Lc;
    const uint64_t sl = leaf0 * L + off;
    if (q < hi - lo) {
      const uint64_t k = mk[lo + q];
      a.key[sl] = k;
      a.val[sl] = mv[lo + q];
      if (is_guard_key(k)) a.row_offset[(k >> 32) - a.rb + 1] = sl;
    } else {
      a.key[sl] = KEY_NONE;
      a.val[sl] = 0;
    }
    if (q == 0) {
      a.cnt[leaf0 + l] = (uint32_t)(hi - lo);
      a.tmask[leaf0 + l] = 0u;                           // tombstones are dropped by a rewrite
      uint32_t gc = 0;
      for (uint64_t e = lo; e < hi; ++e) gc += is_guard_key(mk[e]);
      a.tmask[a.nleaves + leaf0 + l] = gc;               // guards per leaf (third section)
    }
  }
  if (threadIdx.x == 0) {
    const uint64_t d = atomicAdd((unsigned long long *)&a.c->ndirty, 1ull);
    a.dirty[d] = make_uint2((uint32_t)leaf0, Lc);
  }
  __syncthreads();                                       // the smem list is reused by the next window
}

// One accepted SMALL window (<= CL_WMAX slots: levels 1-4 at L = 16) merged and re-dispatched
// by ONE WARP in its private shared-memory list: a CTA per 32-slot window (the block path above)
// left 15 of 16 warps idle and made the level-1 step of a 1M batch with 10^4 rejected keys the
// longest part of the insert.
constexpr uint32_t CL_WMAX = 256;
__device__ void cl_merge_window_warp(const CoopArgs &a, uint32_t cur, uint32_t lvl, uint32_t w, uint64_t *mk,
                                     uint32_t *mv) {
  const uint32_t L = a.L;
  const uint64_t *pk = a.pk[cur];
  const uint32_t *pv = a.pv[cur], *pt = a.pt[cur];
  const uint32_t Lc = 1u << lvl, ws = L << lvl;
  const uint64_t leaf0 = ((uint64_t)(pt[a.wfirst[w]] >> lvl)) << lvl;
  const uint64_t N = a.nw[w];
  const uint64_t ub = a.wfirst[w], ue = a.wfirst[w + 1];
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint32_t leafmask = (L == 32 ? 0xffffffffu : ((1u << L) - 1u) << (lane & ~(L - 1)));
  // live entries before each leaf (Lc <= 32 leaves: one lane each, a warp scan)
  const uint32_t c0 = (uint32_t)lane < Lc ? a.cnt[leaf0 + lane] : 0u;
  uint32_t x = c0;
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  const uint32_t lpre_me = x - c0;                       // lane l: live entries before leaf l
  for (uint32_t o0 = 0; o0 < ws; o0 += 32) {             // gather the live entries
    const uint32_t off = o0 + lane;
    uint64_t k = KEY_NONE;
    uint32_t v = 0;
    if (off < ws) {
      k = a.key[leaf0 * L + off];
      v = a.val[leaf0 * L + off];
    }
    const bool live = off < ws && k != KEY_NONE && v != VAL_TOMB;
    const uint32_t bal = __ballot_sync(0xffffffffu, live);
    const uint32_t lidx = off / L;
    const uint32_t lp = __shfl_sync(0xffffffffu, lpre_me, (int)(lidx & 31));
    if (live) {
      const uint64_t rl = __popc(bal & leafmask & lt) + lp;
      const uint64_t cc = lower_bound_u64(pk, ub, ue, k) - ub;
      bool drop = false;
      uint64_t r;
      if (a.op == GPMA_INSERT) {
        r = rl + cc;
      } else {
        drop = (ub + cc < ue) && pk[ub + cc] == k;
        r = rl - cc;
      }
      if (!drop) {
        mk[r] = k;
        mv[r] = v;
      }
    }
  }
  if (a.op == GPMA_INSERT) {                             // place the window's insertions
    for (uint64_t j = ub + lane; j < ue; j += 32) {
      const uint64_t k = pk[j];
      const uint32_t t = pt[j];
      uint64_t rl = 0;
      {
        // live entries of the window's leaves before t: the prefix held by lane (t - leaf0)
        const uint32_t li = (uint32_t)(t - leaf0);
        for (uint32_t l = 0; l < li; ++l) rl += a.cnt[leaf0 + l];
      }
      const uint64_t base = (uint64_t)t * L;
      for (uint32_t q = 0; q < L; ++q) {
        const uint64_t xk = a.key[base + q];
        if (xk == KEY_NONE || xk > k) break;
        if (a.val[base + q] != VAL_TOMB) ++rl;
      }
      const uint64_t r = (j - ub) + rl;
      mk[r] = k;
      mv[r] = pv[j];
    }
  }
  __syncwarp();                                          // every read of the window is done
  for (uint32_t off = lane; off < ws; off += 32) {       // re-dispatch evenly (R7)
    const uint64_t l = leaf_div(off, L), q = leaf_mod(off, L);
    const uint64_t lo = l * N / Lc, hi = (l + 1) * N / Lc;
    const uint64_t sl = leaf0 * L + off;
    if (q < hi - lo) {
      const uint64_t k = mk[lo + q];
      a.key[sl] = k;
      a.val[sl] = mv[lo + q];
      if (is_guard_key(k)) a.row_offset[(k >> 32) - a.rb + 1] = sl;
    } else {
      a.key[sl] = KEY_NONE;
      a.val[sl] = 0;
    }
    if (q == 0) {
      a.cnt[leaf0 + l] = (uint32_t)(hi - lo);
      a.tmask[leaf0 + l] = 0u;
      uint32_t gc = 0;
      for (uint64_t e = lo; e < hi; ++e) gc += is_guard_key(mk[e]);
      a.tmask[a.nleaves + leaf0 + l] = gc;
    }
  }
  if (lane == 0) {
    const uint64_t d = atomicAdd((unsigned long long *)&a.c->ndirty, 1ull);
    a.dirty[d] = make_uint2((uint32_t)leaf0, Lc);
  }
  __syncwarp();                                          // the warp's list is reused by its next window
}

__global__ void __launch_bounds__(CL_T) k_levels_coop(CoopArgs a) {
  extern __shared__ __align__(16) unsigned char cl_smem[];
  uint64_t *mk = reinterpret_cast<uint64_t *>(cl_smem);
  uint32_t *mv = reinterpret_cast<uint32_t *>(mk + CL_MAXS);
  uint32_t *lpre = mv + CL_MAXS;                         // [CL_MAXS / 4 + 1] (L >= 4)
  __shared__ uint64_t wsum[CL_T / 32];
  cooperative_groups::grid_group grid = cooperative_groups::this_grid();
  CoopState &S = *a.st;
  // every CTA follows the same state: (p, cur, lvl) are recomputed identically everywhere
  uint64_t p = S.p;
  uint32_t cur = S.cur, lvl = S.lvl;
  uint64_t wins = 0, slots = 0;
  uint32_t top = lvl;
  while (p > 0 && lvl <= a.h && ((uint64_t)a.L << lvl) <= CL_MAXS) {
    const uint64_t q = cl_segments(grid, a, p, cur, lvl, wsum);
    grid.sync();
    const uint32_t *pt = a.pt[cur];
    // CountSegment + CountUpdatesInSegment + density test: a warp per window
    {
      const int lane = threadIdx.x & 31;
      const uint64_t nwarps = (uint64_t)gridDim.x * (CL_T / 32);
      const uint64_t Lc = 1ull << lvl;
      for (uint64_t w = (blockIdx.x * (uint64_t)CL_T + threadIdx.x) / 32; w < q; w += nwarps) {
        const uint64_t leaf0 = ((uint64_t)(pt[a.wfirst[w]] >> lvl)) << lvl;
        uint64_t n = 0;
        for (uint64_t l = lane; l < Lc; l += 32) n += a.cnt[leaf0 + l];
        for (int o = 16; o; o >>= 1) n += __shfl_xor_sync(0xffffffffu, n, o);
        if (lane == 0) {
          const uint64_t u = a.wfirst[w + 1] - a.wfirst[w];
          const bool ok = a.op == GPMA_INSERT ? n + u <= a.tmax[lvl] : (n >= u && n - u >= a.tmin[lvl]);
          a.acc[w] = ok ? 1u : 0u;
          a.nw[w] = ok ? (a.op == GPMA_INSERT ? n + u : n - u) : 0;
        }
      }
    }
    grid.sync();
    // Merge + re-dispatch evenly: a warp per accepted small window, a CTA per larger one
    if (((uint64_t)a.L << lvl) <= CL_WMAX && a.L <= 32 && lvl <= 5 && a.warp_merge) {
      const uint32_t wi = threadIdx.x >> 5;
      uint64_t *wk_ = mk + (uint64_t)wi * CL_WMAX;
      uint32_t *wv_ = reinterpret_cast<uint32_t *>(mk + (uint64_t)(CL_T / 32) * CL_WMAX) + (uint64_t)wi * CL_WMAX;
      const uint64_t nwarps = (uint64_t)gridDim.x * (CL_T / 32);
      for (uint64_t w = (blockIdx.x * (uint64_t)CL_T + threadIdx.x) / 32; w < q; w += nwarps) {
        if (!a.acc[w]) continue;
        cl_merge_window_warp(a, cur, lvl, (uint32_t)w, wk_, wv_);
        if ((threadIdx.x & 31) == 0) {
          ++wins;
          slots += (uint64_t)a.L << lvl;
        }
      }
    } else {
      for (uint64_t w = blockIdx.x; w < q; w += gridDim.x) {
        if (!a.acc[w]) continue;
        cl_merge_window(a, cur, lvl, (uint32_t)w, mk, mv, lpre);
        if (threadIdx.x == 0) {
          ++wins;
          slots += (uint64_t)a.L << lvl;
        }
      }
    }
    grid.sync();
    const uint64_t pn = cl_promote(grid, a, p, cur, wsum);
    grid.sync();                                         // the next buffer is complete
    top = lvl;
    p = pn;
    if (pn) cur ^= 1u;
    ++lvl;
  }
  if (wins) {
    atomicAdd((unsigned long long *)&S.windows, (unsigned long long)wins);
    atomicAdd((unsigned long long *)&S.slots, (unsigned long long)slots);
  }
  if (blockIdx.x == 0 && threadIdx.x == 0) {
    S.p = p;
    S.cur = cur;
    S.lvl = lvl;
    S.top = top;
    S.done = 1;
  }
}

// Whole-array even layout of a dense sorted list (create, resize; R7 over all leaves): a thread
// writes 4 consecutive slots of one leaf with 16-B stores (two key pairs, one value quad).
// (head != nullptr: also the locate heads, valid when N >= nleaves -- then no leaf is empty and
// head[l] is the leaf's first key; the caller recomputes them otherwise)
__global__ void k_layout_even(const uint64_t *__restrict__ wk, const uint32_t *__restrict__ wv,
                              uint64_t N, uint64_t *__restrict__ key, uint32_t *__restrict__ val,
                              uint32_t *__restrict__ cnt, uint64_t *__restrict__ row_offset,
                              uint32_t L, uint64_t nleaves, uint32_t rb, uint64_t *__restrict__ head) {
  uint32_t *tmask = cnt + nleaves;
  const uint64_t cap = nleaves * L;
  const int lg = __ffsll((long long)nleaves) - 1;       // nleaves: a power of two
  for (uint64_t s = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) * 4; s < cap;
       s += (uint64_t)gridDim.x * blockDim.x * 4) {
    const uint64_t l = leaf_div(s, L), p = leaf_mod(s, L);
    const uint64_t lo = (l * N) >> lg, hi = ((l + 1) * N) >> lg, m = hi - lo;
    uint64_t k[4];
    uint32_t v[4];
#pragma unroll
    for (int q = 0; q < 4; ++q) {
      if (p + q < m) {
        k[q] = wk[lo + p + q];
        v[q] = wv[lo + p + q];
        if (is_guard_key(k[q])) row_offset[(k[q] >> 32) - rb + 1] = s + q;
      } else {
        k[q] = KEY_NONE;
        v[q] = 0;
      }
    }
    *reinterpret_cast<ulonglong2 *>(key + s) = make_ulonglong2(k[0], k[1]);
    *reinterpret_cast<ulonglong2 *>(key + s + 2) = make_ulonglong2(k[2], k[3]);
    *reinterpret_cast<uint4 *>(val + s) = make_uint4(v[0], v[1], v[2], v[3]);
    if (p == 0) {
      cnt[l] = (uint32_t)m;
      tmask[l] = 0u;
      uint32_t gc = 0;
      for (uint64_t e = lo; e < hi; ++e) gc += is_guard_key(wk[e]);
      tmask[nleaves + l] = gc;
      if (head) head[l] = k[0];
    }
  }
}

// ------------------------------------------------------------------ locate index
__device__ __forceinline__ uint64_t next_head(const uint64_t *__restrict__ key, uint32_t L,
                                              uint64_t nleaves, uint64_t l) {
  for (; l < nleaves; ++l) {
    uint64_t k = key[l * L];
    if (k != KEY_NONE) return k;
  }
  return KEY_NONE;
}

// head[l] = first key of the first non-empty leaf >= l (KEY_NONE if none): a pure
// function of the layout, so concurrent writers agree.
__global__ void k_heads_all(const uint64_t *__restrict__ key, uint64_t *__restrict__ head, uint32_t L,
                            uint64_t nleaves) {
  for (uint64_t l = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; l < nleaves;
       l += (uint64_t)gridDim.x * blockDim.x)
    head[l] = next_head(key, L, nleaves, l);
}

// Fix the heads of rewritten windows and of the run of empty leaves left of them.
// Windows of >= HD_BIG leaves (levels >= 11 at L = 16, the root): a warp per window left a
// 2^24-leaf root rewrite to one warp -- 350 ms for one configs[3] strict-delete batch -- so those
// are fixed up by k_heads_span, a CTA per HD_BIG-leaf chunk of each big window.
constexpr uint32_t HD_BIG = 2048;
__global__ void k_heads_span(const uint64_t *__restrict__ key, uint64_t *__restrict__ head, uint32_t L,
                             uint64_t nleaves, const uint2 *__restrict__ dirty) {
  const uint2 wd = dirty[blockIdx.y];
  const uint64_t l0 = (uint64_t)wd.x + (uint64_t)blockIdx.x * HD_BIG;
  const uint64_t l1 = min(l0 + HD_BIG, (uint64_t)wd.x + wd.y);
  for (uint64_t l = l0 + threadIdx.x; l < l1; l += blockDim.x) head[l] = next_head(key, L, nleaves, l);
  if (blockIdx.x == 0 && threadIdx.x == 0) {             // empty leaves to the left carry the head
    uint64_t hv = next_head(key, L, nleaves, wd.x);
    for (int64_t m = (int64_t)wd.x - 1; m >= 0 && key[(uint64_t)m * L] == KEY_NONE; --m) head[m] = hv;
  }
}

__global__ void k_heads_dirty(const uint64_t *__restrict__ key, uint64_t *__restrict__ head,
                              uint32_t L, uint64_t nleaves, const uint2 *__restrict__ dirty,
                              uint64_t ndirty) {
  const int lane = threadIdx.x & 31;
  const uint64_t warps = (uint64_t)gridDim.x * (blockDim.x / 32);
  for (uint64_t d = (blockIdx.x * (uint64_t)blockDim.x + threadIdx.x) / 32; d < ndirty; d += warps) {
    uint2 wd = dirty[d];
    if (wd.y >= HD_BIG) continue;                        // (k_heads_span: every SM on a big window)
    for (uint64_t l = wd.x + lane; l < (uint64_t)wd.x + wd.y; l += 32)
      head[l] = next_head(key, L, nleaves, l);
    if (lane == 0) {
      uint64_t hv = next_head(key, L, nleaves, wd.x);
      for (int64_t m = (int64_t)wd.x - 1; m >= 0 && key[(uint64_t)m * L] == KEY_NONE; --m) head[m] = hv;
    }
  }
}

__global__ void k_sum_cnt(const uint32_t *__restrict__ cnt, uint64_t nleaves, Ctrl *c) {
  uint64_t s = 0;
  for (uint64_t l = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; l < nleaves;
       l += (uint64_t)gridDim.x * blockDim.x)
    s += cnt[l];
  for (int o = 16; o; o >>= 1) s += __shfl_xor_sync(0xffffffffu, s, o);
  if ((threadIdx.x & 31) == 0 && s) atomicAdd((unsigned long long *)&c->sum, (unsigned long long)s);
}

__global__ void k_count_slots(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val,
                              uint64_t cap, Ctrl *c) {
  uint64_t e = 0, t = 0;
  for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < cap;
       s += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t k = key[s];
    if (k == KEY_NONE || is_guard_key(k)) continue;
    if (val[s] == VAL_TOMB) ++t;
    else ++e;
  }
  for (int o = 16; o; o >>= 1) {
    e += __shfl_xor_sync(0xffffffffu, e, o);
    t += __shfl_xor_sync(0xffffffffu, t, o);
  }
  if ((threadIdx.x & 31) == 0) {
    if (e) atomicAdd((unsigned long long *)&c->sum, (unsigned long long)e);
    if (t) atomicAdd((unsigned long long *)&c->sum2, (unsigned long long)t);
  }
}

// create: merge sorted unique edges with the V guards into a dense list (R1).
// Edge j with source u lands at j + u; guard u at (#edges with src <= u) + u.
__global__ void k_place_edges(const uint64_t *__restrict__ sk, const uint32_t *__restrict__ sv,
                              const uint32_t *__restrict__ pos, const uint32_t *__restrict__ keep,
                              uint64_t n, uint64_t *__restrict__ wk, uint32_t *__restrict__ wv, uint32_t rb) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x) {
    if (!keep[i]) continue;
    uint64_t k = sk[i];
    uint64_t d = (uint64_t)pos[i] + ((k >> 32) - rb);   // guards of the owned rows before it
    wk[d] = k;
    wv[d] = sv[i];
  }
}

__global__ void k_place_guards(uint32_t rb, uint32_t nr, const uint64_t *__restrict__ ek, uint64_t m,
                               uint64_t *__restrict__ wk, uint32_t *__restrict__ wv) {
  for (uint64_t u = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; u < nr;
       u += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t gk = ((u + rb) << 32) | COL_GUARD;
    // number of edges with key < guard key, searched in the dense edge list ek[0..m)
    uint64_t lo = 0, hi = m;
    while (lo < hi) {
      uint64_t mid = (lo + hi) >> 1;
      if (ek[mid] < gk) lo = mid + 1;
      else hi = mid;
    }
    wk[lo + u] = gk;
    wv[lo + u] = 0;
  }
}

__global__ void k_unique_last(const uint64_t *__restrict__ sk, uint64_t n, uint32_t *__restrict__ keep) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x)
    keep[i] = (i + 1 == n || sk[i + 1] != sk[i]) ? 1u : 0u;
}

__global__ void k_compact_kv(const uint32_t *__restrict__ keep, const uint32_t *__restrict__ pos,
                             uint64_t n, const uint64_t *__restrict__ ik, const uint32_t *__restrict__ iv,
                             uint64_t *__restrict__ ok, uint32_t *__restrict__ ov) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < n;
       i += (uint64_t)gridDim.x * blockDim.x)
    if (keep[i]) {
      ok[pos[i]] = ik[i];
      ov[pos[i]] = iv[i];
    }
}

__global__ void k_raw_counts(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val,
                             uint32_t *__restrict__ cnt, uint64_t *__restrict__ row_offset, uint32_t L,
                             uint64_t nleaves, uint32_t rb, uint32_t nr) {
  for (uint64_t l = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; l < nleaves;
       l += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t c = 0, m = 0, gc = 0;
    for (uint32_t p = 0; p < L; ++p) {
      uint64_t s = l * L + p;
      uint64_t k = key[s];
      if (k == KEY_NONE) continue;
      gc += is_guard_key(k);
      if (val[s] != VAL_TOMB) ++c;
      else m |= 1u << p;
      if (is_guard_key(k) && (uint32_t)(k >> 32) - rb < nr) row_offset[(k >> 32) - rb + 1] = s;
    }
    cnt[l] = c;
    cnt[nleaves + l] = m;
    cnt[2 * nleaves + l] = gc;
  }
}

// ------------------------------------------------------------------ host driver
static gpma_status read_ctrl(gpma *g, cudaStream_t s) {
  GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  return GPMA_OK;
}

static gpma_status zero_ctrl(gpma *g, cudaStream_t s) {
  GP_CHECK(g, fill_zero(g, g->ctrl_d, sizeof(Ctrl), s));
  return GPMA_OK;
}

gpma_status recompute_heads(gpma *g, cudaStream_t s) {
  uint64_t nl = g->cap / g->L;
  GP_LAUNCH(g, k_heads_all, grid_for(nl), TB, 0, s, g->key, g->head, g->L, nl);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status count_slots(gpma *g, uint64_t *live_edges, uint64_t *tombs, cudaStream_t s) {
  gpma_status st = zero_ctrl(g, s);
  if (st) return st;
  GP_LAUNCH(g, k_count_slots, grid_for(g->cap), TB, 0, s, g->key, g->val, g->cap, g->ctrl_d);
  if ((st = read_ctrl(g, s))) return st;
  *live_edges = g->ctrl_h->sum;
  *tombs = g->ctrl_h->sum2;
  return GPMA_OK;
}

// GPMA_SPARE=0 frees the old store arrays at a resize instead of keeping them as a spare set
static bool spare_on() {
  const char *e = getenv("GPMA_SPARE");
  return !e || atoi(e) != 0;
}

static void set_geometry(gpma *g, uint64_t cap) {
  g->cap = cap;
  g->h = ilog2(cap / g->L);
  level_bounds(g->L, g->h, g->rho0, g->rhoh, g->tau0, g->tauh, g->tmin, g->tmax);
}

// The store arrays of the previous capacity are kept as a spare set across a resize, so the
// dual resize (a halving after a doubling, a doubling after a halving) takes them back instead
// of allocating -- and mapping -- GBs (round-1 resizing steps varied 16 ms - 1.1 s).
static void spare_stash(gpma *g, uint64_t cap, uint64_t *k, uint32_t *v, uint32_t *c, uint64_t *hd, cudaStream_t s) {
  if (g->spare.key) {
    dev_free(g, g->spare.key, s);
    dev_free(g, g->spare.val, s);
    dev_free(g, g->spare.cnt, s);
    dev_free(g, g->spare.head, s);
  }
  g->spare.cap = cap;
  g->spare.key = k;
  g->spare.val = v;
  g->spare.cnt = c;
  g->spare.head = hd;
}

void spare_release(gpma *g, cudaStream_t s) { spare_stash(g, 0, nullptr, nullptr, nullptr, nullptr, s); }

static gpma_status alloc_store(gpma *g, uint64_t cap, uint64_t **k, uint32_t **v, uint32_t **c,
                               uint64_t **hd, cudaStream_t s) {
  uint64_t nl = cap / g->L;
  if (g->spare.key && g->spare.cap == cap && spare_on()) {
    *k = g->spare.key;
    *v = g->spare.val;
    *c = g->spare.cnt;
    *hd = g->spare.head;
    g->spare = gpma::SpareStore{};
    return GPMA_OK;
  }
  *k = nullptr; *v = nullptr; *c = nullptr; *hd = nullptr;
  cudaError_t e1 = dev_alloc(g, (void **)k, cap * 8, s);
  cudaError_t e2 = dev_alloc(g, (void **)v, cap * 4, s);
  cudaError_t e3 = dev_alloc(g, (void **)c, nl * 12, s);  // live counts, tombstone masks, guards
  cudaError_t e4 = dev_alloc(g, (void **)hd, ((nl + 7) & ~(uint64_t)7) * 8, s);   // (whole 64-B lines)
  if ((e1 || e2 || e3 || e4) && g->spare.key) {          // out of memory: give the spare set back first
    dev_free(g, *k, s);
    dev_free(g, *v, s);
    dev_free(g, *c, s);
    dev_free(g, *hd, s);
    spare_release(g, s);
    e1 = dev_alloc(g, (void **)k, cap * 8, s);
    e2 = dev_alloc(g, (void **)v, cap * 4, s);
    e3 = dev_alloc(g, (void **)c, nl * 12, s);
    e4 = dev_alloc(g, (void **)hd, ((nl + 7) & ~(uint64_t)7) * 8, s);
  }
  if (e1 || e2 || e3 || e4) {
    cudaGetLastError();
    dev_free(g, *k, s);
    dev_free(g, *v, s);
    dev_free(g, *c, s);
    dev_free(g, *hd, s);
    *k = nullptr; *v = nullptr; *c = nullptr; *hd = nullptr;
    g->err = "out of device memory allocating the store";
    return GPMA_ERR_OOM;
  }
  return GPMA_OK;
}

// dense sorted list (wk, wv)[0..N) -> whole array of `cap` slots
gpma_status build_from_sorted(gpma *g, const uint64_t *wk, const uint32_t *wv, uint64_t N,
                              cudaStream_t s) {
  uint64_t nl = g->cap / g->L;
  GP_LAUNCH(g, k_layout_even, grid_for(g->cap / 4), TB, 0, s, wk, wv, N, g->key, g->val, g->cnt,
            g->row_offset, g->L, nl, g->rb, N >= nl ? g->head : nullptr);
  GP_CHECK(g, cudaGetLastError());
  if (N < nl) {
    gpma_status st = recompute_heads(g, s);
    if (st) return st;
  }
  return recompute_degrees(g, s);
}

gpma_status load_raw(gpma *g, const uint64_t *keys, const uint32_t *vals, cudaStream_t s) {
  GP_CHECK(g, stage_in(g, g->key, keys, g->cap * 8, s));
  GP_CHECK(g, stage_in(g, g->val, vals, g->cap * 4, s));
  uint64_t nl = g->cap / g->L;
  GP_LAUNCH(g, k_raw_counts, grid_for(nl), TB, 0, s, g->key, g->val, g->cnt, g->row_offset, g->L, nl,
            g->rb, g->nr);
  GP_CHECK(g, cudaGetLastError());
  gpma_status st = recompute_heads(g, s);
  if (st) return st;
  return recompute_degrees(g, s);
}

// Sort a batch (Alg. 4 l.2) in place: (keys, vals) is library scratch (the staged copy of the
// caller's batch), clobbered by the ping-pong with b_sk[1]/b_sv[1]; vals == nullptr sorts the
// keys only.  Duplicates stay (stable: the last copy of a key is the last of its run, R10).
struct Sorted {
  uint64_t *k = nullptr;
  uint32_t *v = nullptr;
  uint64_t *ok = nullptr;      // the other buffer of the pair (free scratch after the sort)
  uint32_t *ov = nullptr;
};

static gpma_status sort_batch(gpma *g, uint64_t *keys, uint32_t *vals, uint64_t n, Sorted *out, cudaStream_t s) {
  GP_CHECK(g, ensure(g, g->b_sk[1], n * 8, s));
  if (vals) GP_CHECK(g, ensure(g, g->b_sv[1], n * 4, s));
  uint64_t *k1 = (uint64_t *)g->b_sk[1].p;
  uint32_t *v1 = vals ? (uint32_t *)g->b_sv[1].p : nullptr;
  int sh[8];
  const int ns = key_shifts(g->V, sh);
  int which = 0;
  GP_CHECK(g, radix_sort_pairs(g, keys, vals, k1, v1, n, sh, ns, s, &which));
  out->k = which ? k1 : keys;
  out->v = which ? v1 : vals;
  out->ok = which ? keys : k1;
  out->ov = which ? vals : v1;
  return GPMA_OK;
}

static gpma_status validate(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n,
                            bool check_vals, cudaStream_t s) {
  gpma_status st = zero_ctrl(g, s);
  if (st) return st;
  GP_LAUNCH(g, k_validate, grid_for(n), TB, 0, s, keys, vals, n, g->V, g->rb, g->nr, check_vals ? 1 : 0,
            g->ctrl_d);
  if ((st = read_ctrl(g, s))) return st;
  if (g->ctrl_h->err & 2u) return GPMA_ERR_RESERVED;
  if (g->ctrl_h->err & 1u) return GPMA_ERR_RANGE;
  return GPMA_OK;
}

// Validate a caller's batch slice against the GLOBAL vertex range (multi-GPU routing runs
// before the owner is known): ctrl.err gets the bits, no read-back (the caller reduces them).
gpma_status validate_slice(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, bool check_vals,
                           cudaStream_t s) {
  gpma_status st = zero_ctrl(g, s);
  if (st) return st;
  if (n) GP_LAUNCH(g, k_validate, grid_for(n), TB, 0, s, keys, vals, n, g->V, 0u, g->V, check_vals ? 1 : 0, g->ctrl_d);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

gpma_status create_from_batch(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n,
                              uint64_t cap_override, uint32_t leaf_override, cudaStream_t s) {
  gpma_status st;
  uint64_t m = 0;
  const uint64_t *ek = nullptr;
  const uint32_t *ev = nullptr;
  if (n) {
    // stage + validate on device
    GP_CHECK(g, ensure(g, g->b_stage[0], n * 8, s));
    GP_CHECK(g, ensure(g, g->b_stage[1], n * 4, s));
    GP_CHECK(g, stage_in(g, g->b_stage[0].p, keys, n * 8, s));
    GP_CHECK(g, stage_in(g, g->b_stage[1].p, vals, n * 4, s));
    if ((st = validate(g, (uint64_t *)g->b_stage[0].p, (uint32_t *)g->b_stage[1].p, n, true, s)))
      return st;
    Sorted srt;
    if ((st = sort_batch(g, (uint64_t *)g->b_stage[0].p, (uint32_t *)g->b_stage[1].p, n, &srt, s))) return st;
    uint64_t *sk = srt.k;
    uint32_t *sv = srt.v;
    GP_CHECK(g, ensure(g, g->b_keep, (n + 1) * 4, s));
    GP_CHECK(g, ensure(g, g->b_pos, (n + 1) * 4, s));
    uint32_t *keep = (uint32_t *)g->b_keep.p, *pos = (uint32_t *)g->b_pos.p;
    GP_LAUNCH(g, k_unique_last, grid_for(n), TB, 0, s, sk, n, keep);
    GP_CHECK(g, scan_u32(g, keep, pos, n, s));
    uint32_t mh = 0;
    GP_CHECK(g, readback(g, &g->ctrl_h->sum, pos + n, 4, s));
    GP_CHECK(g, cudaStreamSynchronize(s));
    mh = (uint32_t)(g->ctrl_h->sum & 0xFFFFFFFFu);
    m = mh;
    // dense unique edges into the other buffer
    uint64_t *uk = srt.ok;
    uint32_t *uv = srt.ov;
    GP_LAUNCH(g, k_compact_kv, grid_for(n), TB, 0, s, keep, pos, n, sk, sv, uk, uv);
    ek = uk;
    ev = uv;
  }
  const uint64_t E = m + g->nr;
  uint64_t cap;
  if (cap_override) {
    cap = cap_override;
    g->L = leaf_override ? leaf_override : leaf_rule(cap);
  } else {
    cap = 8;
    while (E > cap * g->init_bp / 10000) cap *= 2;
    g->L = leaf_override ? leaf_override : leaf_rule(cap);
    if (cap < 2ull * g->L) cap = 2ull * g->L;
  }
  if (cap < 2ull * g->L || (cap & (cap - 1))) {
    g->err = "capacity must be a power of two >= 2L";
    return GPMA_ERR_INVALID_ARG;
  }
  set_geometry(g, cap);
  if ((st = alloc_store(g, cap, &g->key, &g->val, &g->cnt, &g->head, s))) return st;
  GP_CHECK(g, dev_alloc(g, (void **)&g->row_offset, ((uint64_t)g->nr + 1) * 8, s));
  GP_CHECK(g, fill_zero(g, g->row_offset, ((uint64_t)g->nr + 1) * 8, s));
  GP_CHECK(g, dev_alloc(g, (void **)&g->deg, (uint64_t)g->nr * 4 + 4, s));
  if (E > g->tmax[g->h] && !cap_override) {
    g->err = "initial graph exceeds the root bound";
    return GPMA_ERR_INVALID_ARG;
  }
  // dense merged list (edges + guards) in the window scratch
  GP_CHECK(g, ensure(g, g->b_wk, std::max<uint64_t>(E, 1) * 8, s));
  GP_CHECK(g, ensure(g, g->b_wv, std::max<uint64_t>(E, 1) * 4, s));
  uint64_t *wk = (uint64_t *)g->b_wk.p;
  uint32_t *wv = (uint32_t *)g->b_wv.p;
  if (m) {
    // positions: edge with unique rank j (pos) and source u goes to j + u
    uint32_t *keep = (uint32_t *)g->b_keep.p, *pos = (uint32_t *)g->b_pos.p;
    // recompute from the dense list: keep = 1, pos = j
    // (the dense list ek is sorted & unique; place directly)
    GP_LAUNCH(g, k_unique_last, grid_for(m), TB, 0, s, ek, m, keep);  // all ones (unique)
    GP_CHECK(g, scan_u32(g, keep, pos, m, s));
    GP_LAUNCH(g, k_place_edges, grid_for(m), TB, 0, s, ek, ev, pos, keep, m, wk, wv, g->rb);
  }
  GP_LAUNCH(g, k_place_guards, grid_for(g->nr), TB, 0, s, g->rb, g->nr, ek, m, wk, wv);
  GP_CHECK(g, cudaGetLastError());
  g->rows_indexed = true;      // one guard per owned row from here on (R1)
  return build_from_sorted(g, wk, wv, E, s);
}

// ---- one GPMA+ round (level `lvl`), generic device-scale implementation
struct LevelOut {
  uint64_t q, nacc, p_new;
};

// single-CTA front / back of small levels (GPMA_LVL_SMALL=0 disables; read per call)
static int lvl_small_on() {      // 0 off, 1 front/back only, 2 (default) + fused window merge
  const char *e = getenv("GPMA_LVL_SMALL");
  return e ? atoi(e) : 2;
}

// GPMA_GATHER_BIG=0: windows of >= 4096 slots gathered by the per-slot global search instead
static bool gather_big_on() {
  const char *e = getenv("GPMA_GATHER_BIG");
  return !e || atoi(e) != 0;
}

// head fix-up of the windows rewritten by a batch's level loop: a warp per small window, a CTA
// per HD_BIG-leaf chunk of every big one (recorded by level_step in g->big_dirty)
static gpma_status fix_heads(gpma *g, uint64_t ndirty, cudaStream_t s) {
  const uint64_t nl = g->cap / g->L;
  const uint2 *dirty = (const uint2 *)g->b_dirty.p;
  GP_LAUNCH(g, k_heads_dirty, grid_for(ndirty * 32), TB, 0, s, g->key, g->head, g->L, nl, dirty, ndirty);
  for (const auto &b : g->big_dirty) {
    g->last.last_big_head_windows += b[1];
    for (uint64_t y0 = 0; y0 < b[1]; y0 += 65535) {
      const unsigned ny = (unsigned)std::min<uint64_t>(65535, b[1] - y0);
      GP_LAUNCH(g, k_heads_span, dim3((unsigned)(b[2] / HD_BIG), ny), TB, 0, s, g->key, g->head, g->L, nl,
                dirty + b[0] + y0);
    }
  }
  g->big_dirty.clear();
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

static gpma_status level_step(gpma *g, Lvl &a, int cur, LevelOut *out, uint64_t *dirty_base,
                              cudaStream_t s, bool resize_target, uint64_t new_cap, uint64_t *nk,
                              uint32_t *nv, uint32_t *ncnt, uint64_t *nhead = nullptr) {
  const uint64_t p = a.p;
  const uint64_t nleaves = g->cap / g->L;
  const uint64_t wins_bound = std::min<uint64_t>(p, nleaves >> a.lvl);
  const uint64_t wslots = (uint64_t)g->L << a.lvl;
  const unsigned gp = grid_for(p);
  const bool small = p <= LS_MAXP && a.lvl <= LS_MAXLVL && lvl_small_on();
  if (small) {
    GP_LAUNCH(g, k_lvl_front_small, 1, LS_T, 0, s, a, g->cnt);
  } else {
  if (gstart_fused()) {                                  // UniqueSegments (l.18-21) in one pass
    const uint64_t nt = std::max<uint64_t>(1, (p + GS_TILE - 1) / GS_TILE);
    DevBuf &sb = tl_scan ? *tl_scan : g->b_scan;
    GP_CHECK(g, ensure(g, sb, (nt + 1) * sizeof(unsigned long long), s));
    GP_CHECK(g, fill_zero(g, sb.p, (nt + 1) * sizeof(unsigned long long), s));
    GP_LAUNCH(g, k_group_starts<uint32_t>, (unsigned)nt, GS_T, 0, s, a.pt, p, a.lvl, a.wfirst, (uint32_t *)nullptr,
              a.hf, a.widx, (unsigned long long *)sb.p, g->ctrl_d);
  } else {
    GP_LAUNCH(g, k_lvl_flags, gp, TB, 0, s, a);
    GP_CHECK(g, scan_u32(g, a.hf, a.widx, p, s));
    GP_LAUNCH(g, k_lvl_first, gp, TB, 0, s, a);
  }
  if (a.lvl <= 4) GP_LAUNCH(g, k_lvl_count<1>, grid_for(p), TB, 0, s, a, g->cnt);
  else if (a.lvl <= 11) GP_LAUNCH(g, k_lvl_count<32>, grid_for(p * 32), TB, 0, s, a, g->cnt);
  else {
    const uint64_t nleaf_w = 1ull << a.lvl;
    const uint32_t chunk = (uint32_t)std::min<uint64_t>(nleaf_w, 16384);
    GP_CHECK(g, fill_zero(g, a.nw, p * 8, s));
    GP_LAUNCH(g, k_lvl_count_wide, dim3((unsigned)(nleaf_w / chunk), (unsigned)wins_bound), TB, 0, s, a, g->cnt,
              chunk);
    GP_LAUNCH(g, k_lvl_accept, gp, TB, 0, s, a);
  }
  GP_CHECK(g, scan_u32(g, a.acc, a.aidx, p, s));
  GP_CHECK(g, scan_u64(g, a.nw, a.woff, p, s));
  GP_LAUNCH(g, k_lvl_alist, gp, TB, 0, s, a);
  }
  const bool merge_small = small && !resize_target && wslots <= (uint64_t)LM_MAXS && lvl_small_on() > 1;
  if (merge_small) {
    GP_LAUNCH(g, k_lvl_merge_small, (unsigned)wins_bound, LM_T, 0, s, a, g->key, g->val, g->cnt, tmask_of(g),
              g->row_offset, (uint2 *)g->b_dirty.p, *dirty_base);
  } else {
    // Windows of >= GB_CHUNK slots (the host-driven high levels): read the number of accepted
    // windows first -- a root-bound batch (every level rejects) then skips the merge kernels,
    // and the scratch is sized by the accepted windows, not by every window holding pending
    // updates (which had allocated up to half the store's bytes at level h-1 for nothing).
    uint64_t nacc_h = wins_bound;
    if (!a.force && !small && wslots >= (uint64_t)GB_CHUNK) {
      GP_CHECK(g, readback(g, g->pin, a.aidx + p, 4, s));
      GP_CHECK(g, cudaStreamSynchronize(s));
      uint32_t na;
      memcpy(&na, g->pin, 4);
      nacc_h = na;
    }
    if (nacc_h == 0) goto merged;
  {
    // scratch: sum of merged window sizes <= accepted windows * wslots (and <= cap + p)
    uint64_t need = a.force ? (g->root_need ? g->root_need : g->cap + p) : nacc_h * wslots;
    GP_CHECK(g, ensure(g, g->b_wk, need * 8, s));
    GP_CHECK(g, ensure(g, g->b_wv, need * 4, s));
    a.wk = (uint64_t *)g->b_wk.p;
    a.wv = (uint32_t *)g->b_wv.p;
    a.lcnt = nullptr;
    if (small && a.lvl) {
      a.lcnt = g->cnt;                                   // the gather sums its window's leaves itself
    } else if (a.lvl) {
      uint64_t lb = wins_bound << a.lvl;
      GP_CHECK(g, ensure(g, g->b_lpre, (lb + 1) * 8, s));
      a.lpre = (uint64_t *)g->b_lpre.p;
      GP_LAUNCH(g, k_lvl_leafcnt, grid_for(lb), TB, 0, s, a, g->cnt, lb);
      GP_CHECK(g, scan_u64(g, a.lpre, a.lpre, lb, s));
    }
    uint64_t bslots = (a.force ? wins_bound : nacc_h) * wslots;
    uint64_t bslots_r = (bslots + 31) & ~31ull;
    if (a.lvl && wslots >= (uint64_t)GB_CHUNK && gather_big_on()) {
      const uint64_t nch = bslots / GB_CHUNK;
      GP_LAUNCH(g, k_lvl_gather_big, (unsigned)std::min<uint64_t>(nch, (uint64_t)num_sms() * gb_per_sm()), GB_T, 0, s, a, g->key,
                g->val, nch);
    } else {
      GP_LAUNCH(g, k_lvl_gather, grid_for(bslots_r), TB, 0, s, a, g->key, g->val, bslots_r);
    }
    if (a.op == GPMA_INSERT) GP_LAUNCH(g, k_lvl_place, gp, TB, 0, s, a, g->key, g->val);
    if (!resize_target) {
      GP_LAUNCH(g, k_lvl_redistribute, grid_for(bslots / 4), TB, 0, s, a, g->key, g->val, g->cnt, tmask_of(g),
                g->row_offset, bslots, (uint2 *)g->b_dirty.p, *dirty_base);
    } else {
      // the single root window, laid out over the whole new array
      uint64_t N;
      GP_CHECK(g, readback(g, &g->ctrl_h->sum, a.nw, 8, s));
      GP_CHECK(g, cudaStreamSynchronize(s));
      N = g->ctrl_h->sum;
      uint64_t nl_new = new_cap / g->L;
      g->root_heads_done = nhead && N >= nl_new;
      GP_LAUNCH(g, k_layout_even, grid_for(new_cap / 4), TB, 0, s, a.wk, a.wv, N, nk, nv, ncnt,
                g->row_offset, g->L, nl_new, g->rb, g->root_heads_done ? nhead : nullptr);
    }
  }
  }
merged:
  if (small) {
    GP_LAUNCH(g, k_lvl_back_small, 1, LS_T, 0, s, a, g->ctrl_d);
  } else {
    GP_LAUNCH(g, k_lvl_keep, gp, TB, 0, s, a);
    GP_CHECK(g, scan_u32(g, a.keep, a.kpos, p, s));
    GP_LAUNCH(g, k_lvl_summary, 1, 1, 0, s, a, g->ctrl_d);
  }
  if (g->trace_on) {
    // copy segment starts / offsets / flags of this level (debug only)
    std::vector<uint32_t> wf(p + 1), ac(p + 1), pt(p), wi(p + 1);
    GP_CHECK(g, cudaMemcpyAsync(wf.data(), a.wfirst, (p + 1) * 4, cudaMemcpyDeviceToHost, s));
    GP_CHECK(g, cudaMemcpyAsync(ac.data(), a.acc, p * 4, cudaMemcpyDeviceToHost, s));
    GP_CHECK(g, cudaMemcpyAsync(pt.data(), a.pt, p * 4, cudaMemcpyDeviceToHost, s));
    GP_CHECK(g, cudaMemcpyAsync(wi.data(), a.widx, (p + 1) * 4, cudaMemcpyDeviceToHost, s));
    GP_CHECK(g, cudaStreamSynchronize(s));
    uint32_t q = wi[p];
    for (uint32_t w = 0; w < q; ++w) {
      uint64_t start = ((uint64_t)(pt[wf[w]] >> a.lvl) << a.lvl) * g->L;
      g->trace.insert(g->trace.end(), {a.lvl, start, wf[w], ac[w]});
    }
    g->trace.insert(g->trace.end(), {a.lvl, KEY_NONE, wf[q], 2});
  }
  gpma_status st = read_ctrl(g, s);
  if (st) return st;
  out->q = g->ctrl_h->sum & 0xFFFFFFFFull;
  out->nacc = g->ctrl_h->sum >> 32;
  out->p_new = g->ctrl_h->sum2;
  if (out->nacc && ((uint64_t)1 << a.lvl) >= HD_BIG && !resize_target)
    g->big_dirty.push_back({*dirty_base, out->nacc, (uint64_t)1 << a.lvl});
  *dirty_base += out->nacc;
  // compact the pending list into the other buffer
  if (out->p_new && !resize_target) {
    GP_LAUNCH(g, k_compact_pending, grid_for(p), TB, 0, s, a.keep, a.kpos, p, a.pk, a.pv, a.pt,
              (uint64_t *)g->b_pk[cur ^ 1].p, (uint32_t *)g->b_pv[cur ^ 1].p,
              (uint32_t *)g->b_pt[cur ^ 1].p, g->ctrl_d);
  }
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

static gpma_status level_buffers(gpma *g, uint64_t n, cudaStream_t s) {
  size_t b4 = (n + 2) * 4, b8 = (n + 2) * 8;
  GP_CHECK(g, ensure(g, g->b_hf, b4, s));
  GP_CHECK(g, ensure(g, g->b_widx, b4, s));
  GP_CHECK(g, ensure(g, g->b_wfirst, b4, s));
  GP_CHECK(g, ensure(g, g->b_acc, b4, s));
  GP_CHECK(g, ensure(g, g->b_aidx, b4, s));
  GP_CHECK(g, ensure(g, g->b_alist, b4, s));
  GP_CHECK(g, ensure(g, g->b_keep2, b4, s));
  GP_CHECK(g, ensure(g, g->b_kpos, b4, s));
  GP_CHECK(g, ensure(g, g->b_nw, b8, s));
  GP_CHECK(g, ensure(g, g->b_woff, b8, s));
  GP_CHECK(g, ensure(g, g->b_dirty, (n + 2) * sizeof(uint2), s));
  for (int i = 0; i < 2; ++i) {
    GP_CHECK(g, ensure(g, g->b_pk[i], b8, s));
    GP_CHECK(g, ensure(g, g->b_pv[i], b4, s));
    GP_CHECK(g, ensure(g, g->b_pt[i], b4, s));
  }
  return GPMA_OK;
}

static Lvl make_lvl(gpma *g, int cur, uint64_t p, uint32_t lvl, int op) {
  Lvl a{};
  a.pk = (const uint64_t *)g->b_pk[cur].p;
  a.pv = (const uint32_t *)g->b_pv[cur].p;
  a.pt = (const uint32_t *)g->b_pt[cur].p;
  a.p = p;
  a.lvl = lvl;
  a.L = g->L;
  a.hf = (uint32_t *)g->b_hf.p;
  a.widx = (uint32_t *)g->b_widx.p;
  a.wfirst = (uint32_t *)g->b_wfirst.p;
  a.acc = (uint32_t *)g->b_acc.p;
  a.aidx = (uint32_t *)g->b_aidx.p;
  a.alist = (uint32_t *)g->b_alist.p;
  a.keep = (uint32_t *)g->b_keep2.p;
  a.kpos = (uint32_t *)g->b_kpos.p;
  a.nw = (uint64_t *)g->b_nw.p;
  a.woff = (uint64_t *)g->b_woff.p;
  a.lpre = (uint64_t *)g->b_lpre.p;
  a.tmin = lvl < g->tmin.size() ? g->tmin[lvl] : 0;
  a.tmax = lvl < g->tmax.size() ? g->tmax[lvl] : 0;
  a.op = op;
  a.force = 0;
  a.rb = g->rb;
  a.nleaves = g->cap / g->L;
  a.sup = g->sup_on ? (const uint32_t *)g->b_sup.p : nullptr;
  return a;
}

// Root resize (Alg. 4 l.16-17; R14): double until the live entries plus the pending
// insertions fit max_h of the new capacity; halve (strict deletes) while below min_h
// and cap > 2L.  Everything is laid out evenly over the new array.
// GPMA_TRACE_ALLOC=1: phase times of a root resize on stderr (the stream synchronised at each
// stamp -- diagnostics only)
static thread_local std::chrono::steady_clock::time_point tl_call_start;
struct ResizeTrace {
  bool on;
  cudaStream_t s;
  std::chrono::steady_clock::time_point t;
  explicit ResizeTrace(cudaStream_t s_) : s(s_) {
    const char *e = getenv("GPMA_TRACE_ALLOC");
    on = e && atoi(e) != 0;
    if (on) {
      cudaStreamSynchronize(s);
      t = std::chrono::steady_clock::now();
      fprintf(stderr, "[gpma] resize %-12s %.3f ms\n", "levels<root",
              std::chrono::duration<double, std::milli>(t - tl_call_start).count());
    }
  }
  void stamp(const char *what) {
    if (!on) return;
    cudaStreamSynchronize(s);
    const auto n = std::chrono::steady_clock::now();
    fprintf(stderr, "[gpma] resize %-12s %.3f ms\n", what, std::chrono::duration<double, std::milli>(n - t).count());
    t = n;
  }
};

static gpma_status resize(gpma *g, int cur, uint64_t p, int op, cudaStream_t s, uint64_t *dirty_base) {
  Nvtx nvtx_("update: root resize");
  ResizeTrace tr(s);
  gpma_status st;
  uint64_t nl = g->cap / g->L;
  if ((st = zero_ctrl(g, s))) return st;
  GP_LAUNCH(g, k_sum_cnt, grid_for(nl), TB, 0, s, g->cnt, nl, g->ctrl_d);
  if ((st = read_ctrl(g, s))) return st;
  const uint64_t ntot = g->ctrl_h->sum;
  const uint64_t N = op == GPMA_INSERT ? ntot + p : ntot - p;
  uint64_t cap = g->cap;
  std::vector<uint64_t> mn, mx;
  if (op == GPMA_INSERT) {
    for (;;) {
      uint32_t hh = ilog2(cap / g->L);
      level_bounds(g->L, hh, g->rho0, g->rhoh, g->tau0, g->tauh, mn, mx);
      if (N <= mx[hh]) break;
      cap *= 2;
    }
  } else {
    for (;;) {
      uint32_t hh = ilog2(cap / g->L);
      level_bounds(g->L, hh, g->rho0, g->rhoh, g->tau0, g->tauh, mn, mx);
      if (!(cap > 2ull * g->L && N < mn[hh])) break;
      level_bounds(g->L, hh - 1, g->rho0, g->rhoh, g->tau0, g->tauh, mn, mx);
      if (N > mx[hh - 1]) break;
      cap /= 2;
    }
  }
  uint64_t *nk = g->key;
  uint32_t *nv = g->val, *ncnt = g->cnt;
  uint64_t *nhead = g->head;
  tr.stamp("count");
  if (cap != g->cap) {
    if ((st = alloc_store(g, cap, &nk, &nv, &ncnt, &nhead, s))) return st;
  }
  tr.stamp("alloc_store");
  Lvl a = make_lvl(g, cur, p, g->h, op);
  a.force = 1;
  LevelOut lo{};
  g->root_need = ntot + p;                 // the dense root list: live entries + the pending
  g->root_heads_done = false;
  st = level_step(g, a, cur, &lo, dirty_base, s, true, cap, nk, nv, ncnt, nhead);
  g->root_need = 0;
  if (st) return st;
  tr.stamp("root_merge");
  if (cap != g->cap) {
    if (spare_on()) {
      spare_stash(g, g->cap, g->key, g->val, g->cnt, g->head, s);
    } else {
      dev_free(g, g->key, s);
      dev_free(g, g->val, s);
      dev_free(g, g->cnt, s);
      dev_free(g, g->head, s);
    }
    g->key = nk;
    g->val = nv;
    g->cnt = ncnt;
    g->head = nhead;
    g->resizes++;
    g->last.last_resized = 1;
  }
  tr.stamp("free/stash");
  set_geometry(g, cap);
  g->last.last_slots_rewritten += cap;
  g->last.last_windows_rewritten += 1;
  st = g->root_heads_done ? GPMA_OK : recompute_heads(g, s);   // (heads written by the layout)
  tr.stamp("heads");
  return st;
}

// ---- the device-resident level loop from the host
__global__ void k_coop_init(CoopState *st, uint64_t p, uint32_t cur, uint32_t lvl, Ctrl *c, uint64_t ndirty) {
  st->p = p;
  st->cur = cur;
  st->lvl = lvl;
  st->done = 0;
  st->q = 0;
  st->windows = 0;
  st->slots = 0;
  st->top = lvl;
  c->ndirty = ndirty;
}

// GPMA_LVL_COOP=0 disables the device-resident level loop (read per call)
// GPMA_COOP_MAXP: the largest pending count the device level loop takes (read per call);
// larger climbs go level by level from the host, whose steps spread a level's windows over
// every SM at once (the cooperative kernel's warps merge their share of windows one after the
// other: barrier-bound at ~0.6M pending)
static bool coop_eligible(gpma *g, uint64_t p, uint32_t lvl) {
  const char *e = getenv("GPMA_LVL_COOP");
  if (e && atoi(e) == 0) return false;
  uint64_t maxp = 1ull << 18;                   // (measured: configs[3] resizing steps 6.5 / 9.7 / 11.8 -> 6.0 / 9.1 / 10.7 ms)
  if (const char *m = getenv("GPMA_COOP_MAXP")) maxp = (uint64_t)atoll(m);
  return p <= maxp && ((uint64_t)g->L << lvl) <= CL_MAXS && g->h < 48;
}

static gpma_status coop_levels(gpma *g, int &cur, uint64_t &p, uint32_t &lvl, uint64_t *dirty_base, int op,
                               cudaStream_t s) {
  constexpr size_t smem = (size_t)CL_MAXS * 12 + (CL_MAXS / 4 + 4) * 4;
  static int blocks_per_sm = [] {
    cudaFuncSetAttribute(k_levels_coop, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    int b = 0;
    cudaOccupancyMaxActiveBlocksPerMultiprocessor(&b, k_levels_coop, CL_T, smem);
    return b > 0 ? b : 1;
  }();
  GP_CHECK(g, ensure(g, g->b_misc2, sizeof(CoopState) + 64 + (size_t)8 * 64 * 1024, s));
  CoopArgs a{};
  for (int i = 0; i < 2; ++i) {
    a.pk[i] = (uint64_t *)g->b_pk[i].p;
    a.pv[i] = (uint32_t *)g->b_pv[i].p;
    a.pt[i] = (uint32_t *)g->b_pt[i].p;
  }
  a.hf = (uint32_t *)g->b_hf.p;
  a.widx = (uint32_t *)g->b_widx.p;
  a.wfirst = (uint32_t *)g->b_wfirst.p;
  a.acc = (uint32_t *)g->b_acc.p;
  a.keep = (uint32_t *)g->b_keep2.p;
  a.kpos = (uint32_t *)g->b_kpos.p;
  a.nw = (uint64_t *)g->b_nw.p;
  a.key = g->key;
  a.val = g->val;
  a.cnt = g->cnt;
  a.tmask = tmask_of(g);
  a.row_offset = g->row_offset;
  a.dirty = (uint2 *)g->b_dirty.p;
  a.nleaves = g->cap / g->L;
  a.L = g->L;
  a.h = g->h;
  a.rb = g->rb;
  a.op = op;
  {
    const char *e = getenv("GPMA_LVL_WARP");          // read per call (tests flip it)
    a.warp_merge = e ? atoi(e) : 1;
  }
  for (uint32_t i = 0; i <= g->h; ++i) {
    a.tmin[i] = g->tmin[i];
    a.tmax[i] = g->tmax[i];
  }
  a.st = (CoopState *)g->b_misc2.p;
  a.ctot = (uint64_t *)((char *)g->b_misc2.p + ((sizeof(CoopState) + 63) & ~(size_t)63));
  a.c = g->ctrl_d;
  GP_LAUNCH(g, k_coop_init, 1, 1, 0, s, a.st, p, (uint32_t)cur, lvl, g->ctrl_d, *dirty_base);
  // CTAs per SM (GPMA_COOP_CTAS, default 2): every level costs ~8 grid barriers, whose arrival
  // count serialises on one word; measured 1 / 2 / 4 per SM: configs[2] insert 0.560 / 0.569 /
  // 0.569 ms, configs[3] grow insert 1.56 / 1.31 / 1.33 ms
  static const int per_sm = [] {
    const char *e = getenv("GPMA_COOP_CTAS");
    return e ? std::max(1, atoi(e)) : 2;
  }();
  const int grid = std::max(1, std::min(blocks_per_sm, per_sm) * num_sms());
  void *args[] = {&a};
  g->launches++;
  GP_CHECK(g, cudaLaunchCooperativeKernel((void *)k_levels_coop, grid, CL_T, args, smem, s));
  static_assert(sizeof(CoopState) <= 192, "pinned scratch");
  GP_CHECK(g, readback(g, g->pin, a.st, sizeof(CoopState), s));
  GP_CHECK(g, readback(g, &g->ctrl_h->ndirty, &g->ctrl_d->ndirty, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  CoopState S;
  memcpy(&S, g->pin, sizeof S);
  g->last.last_slots_rewritten += S.slots;
  g->last.last_windows_rewritten += S.windows;
  if (S.top > g->last.last_top_level) g->last.last_top_level = S.top;
  *dirty_base = g->ctrl_h->ndirty;
  cur = (int)S.cur;
  p = S.p;
  lvl = S.lvl;
  return GPMA_OK;
}

// ---- GPMA lock-based insertion (Alg. 1) -----------------------------------------------
__global__ void k_count_leaf_live(const uint32_t *__restrict__ cnt, uint64_t nl, uint64_t *__restrict__ out) {
  for (uint64_t l = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; l < nl;
       l += (uint64_t)gridDim.x * blockDim.x)
    out[l] = cnt[l];
}

__global__ void k_relocate(const uint64_t *__restrict__ pk, uint64_t p, const uint64_t *__restrict__ head,
                           uint32_t nleaves, uint32_t *__restrict__ pt) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < p;
       j += (uint64_t)gridDim.x * blockDim.x)
    pt[j] = locate_leaf(head, nleaves, pk[j]);
}

// Lock arbitration at level `lvl` (R28): among the insertions that reach one segment, the
// contender that climbed from the highest child segment (child = leaf >> (lvl-1)) wins, and
// among contenders of one child -- always the case at the leaves -- the smallest key: the
// first contender of the segment's last child run (Ex. 2: 1 beats 4, 48 beats 35).
// pt is sorted, so that run ends where the segment ends: a binary search for the end of j's
// child run decides it.
__global__ void k_lock_winner(const uint32_t *__restrict__ pt, uint64_t p, uint32_t lvl, uint32_t *__restrict__ win) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < p;
       j += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t sh = lvl ? lvl - 1 : 0;
    const uint32_t c = pt[j] >> sh;
    uint32_t w = 0;
    if (j == 0 || (pt[j - 1] >> sh) != c) {            // first contender of its child run
      if (lvl == 0) {
        w = 1;
      } else {
        uint64_t lo = j + 1, hi = p;                   // first index past the child run
        while (lo < hi) {
          const uint64_t mid = (lo + hi) >> 1;
          if ((pt[mid] >> sh) == c) lo = mid + 1;
          else hi = mid;
        }
        w = (lo == p || (pt[lo] >> lvl) != (pt[j] >> lvl)) ? 1u : 0u;
      }
    }
    win[j] = w;
  }
}

// split at one level by the winner flags (hf) and their exclusive scan (widx): the winner of
// every segment keeps going (winner list), the others abort to the next round (loser list,
// appended at `na`)
__global__ void k_lock_split(const uint64_t *__restrict__ pk, const uint32_t *__restrict__ pv,
                             const uint32_t *__restrict__ pt, const uint32_t *__restrict__ hf,
                             const uint32_t *__restrict__ widx, uint64_t p, uint64_t *__restrict__ wk,
                             uint32_t *__restrict__ wv, uint32_t *__restrict__ wt, uint64_t *__restrict__ ak,
                             uint32_t *__restrict__ av, uint64_t na) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < p;
       j += (uint64_t)gridDim.x * blockDim.x) {
    if (hf[j]) {
      const uint32_t d = widx[j];
      wk[d] = pk[j];
      wv[d] = pv[j];
      wt[d] = pt[j];
    } else {
      const uint64_t d = na + j - widx[j];
      ak[d] = pk[j];
      av[d] = pv[j];
    }
  }
}

__global__ void k_append_kv(const uint64_t *__restrict__ k, const uint32_t *__restrict__ v, uint64_t n,
                            uint64_t *__restrict__ ak, uint32_t *__restrict__ av, uint64_t na) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < n;
       j += (uint64_t)gridDim.x * blockDim.x) {
    ak[na + j] = k[j];
    av[na + j] = v[j];
  }
}

// dense list of every live entry (guards included, tombstones dropped), in key order
__global__ void k_gather_live(const uint64_t *__restrict__ key, const uint32_t *__restrict__ val, uint32_t L,
                              uint64_t cap, const uint64_t *__restrict__ lbase, uint64_t *__restrict__ wk,
                              uint32_t *__restrict__ wv) {
  const int lane = threadIdx.x & 31;
  const uint32_t lt = (1u << lane) - 1u;
  const uint32_t leafmask = (L == 32 ? 0xffffffffu : ((1u << L) - 1u) << (lane & ~(L - 1)));
  const uint64_t capr = (cap + 31) & ~31ull;
  for (uint64_t s = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; s < capr;
       s += (uint64_t)gridDim.x * blockDim.x) {
    uint64_t k = KEY_NONE;
    uint32_t v = 0;
    if (s < cap) {
      k = key[s];
      v = val[s];
    }
    const bool live = s < cap && k != KEY_NONE && v != VAL_TOMB;
    const uint32_t bal = __ballot_sync(0xffffffffu, live);
    if (live) {
      const uint64_t d = lbase[leaf_div(s, L)] + __popc(bal & leafmask & lt);
      wk[d] = k;
      wv[d] = v;
    }
  }
}

// Alg. 1 l.20: double the space of the root segment -- all live entries re-dispatched evenly
// over twice the capacity (R7); the insertion that reached the root retries.
static gpma_status double_root(gpma *g, cudaStream_t s) {
  gpma_status st;
  const uint64_t nl = g->cap / g->L, cap2 = g->cap * 2;
  GP_CHECK(g, ensure(g, g->b_lpre, (nl + 1) * 8, s));
  uint64_t *lb = (uint64_t *)g->b_lpre.p;
  GP_LAUNCH(g, k_count_leaf_live, grid_for(nl), TB, 0, s, g->cnt, nl, lb);
  GP_CHECK(g, scan_u64(g, lb, lb, nl, s));
  GP_CHECK(g, readback(g, &g->ctrl_h->sum, lb + nl, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  const uint64_t N = g->ctrl_h->sum;
  GP_CHECK(g, ensure(g, g->b_wk, std::max<uint64_t>(N, 1) * 8, s));
  GP_CHECK(g, ensure(g, g->b_wv, std::max<uint64_t>(N, 1) * 4, s));
  GP_LAUNCH(g, k_gather_live, grid_for(g->cap), TB, 0, s, g->key, g->val, g->L, g->cap, lb,
            (uint64_t *)g->b_wk.p, (uint32_t *)g->b_wv.p);
  uint64_t *nk;
  uint32_t *nv, *ncnt;
  uint64_t *nhead;
  if ((st = alloc_store(g, cap2, &nk, &nv, &ncnt, &nhead, s))) return st;
  const bool heads_done = N >= cap2 / g->L;
  GP_LAUNCH(g, k_layout_even, grid_for(cap2 / 4), TB, 0, s, (const uint64_t *)g->b_wk.p, (const uint32_t *)g->b_wv.p,
            N, nk, nv, ncnt, g->row_offset, g->L, cap2 / g->L, g->rb, heads_done ? nhead : nullptr);
  if (spare_on()) {
    spare_stash(g, g->cap, g->key, g->val, g->cnt, g->head, s);
  } else {
    dev_free(g, g->key, s);
    dev_free(g, g->val, s);
    dev_free(g, g->cnt, s);
    dev_free(g, g->head, s);
  }
  g->key = nk;
  g->val = nv;
  g->cnt = ncnt;
  g->head = nhead;
  g->resizes++;
  g->last.last_resized = 1;
  set_geometry(g, cap2);
  g->last.last_slots_rewritten += cap2;
  g->last.last_windows_rewritten += 1;
  return heads_done ? GPMA_OK : recompute_heads(g, s);
}

__global__ void k_upd_summary(const uint32_t *__restrict__ pos, const uint32_t *__restrict__ kpos, uint64_t n,
                              Ctrl *c) {
  if (pos) c->sum = pos[n];                          // pending after the pre-pass (else counted)
  c->sum2 = kpos ? kpos[n] : 0;                      // pending after level 0
}

// GPMA concurrent insertion (Alg. 1): rounds of level-synchronous climbs with one
// lock per segment.  Lock arbitration is deterministic (R28, k_lock_winner) -- the others
// abort to the next round -- so the layout is reproducible (the oracle follows the same rule).  Winners test count + 1 <= max_i and are
// merged by the generic level step; a winner that reaches the root doubles it (l.20).
static gpma_status gpma_lock_insert(gpma *g, uint64_t p, cudaStream_t s) {
  gpma_status st;
  GP_CHECK(g, ensure(g, g->b_stage[2], (p + 1) * 8, s));
  GP_CHECK(g, ensure(g, g->b_stage[3], (p + 1) * 4, s));
  uint64_t *ak = (uint64_t *)g->b_stage[2].p;
  uint32_t *av = (uint32_t *)g->b_stage[3].p;
  uint64_t rounds = 0;
  while (p > 0) {
    ++rounds;
    int cur = 0;
    const uint64_t nl = g->cap / g->L;
    GP_LAUNCH(g, k_relocate, grid_for(p), TB, 0, s, (const uint64_t *)g->b_pk[0].p, p, g->head, (uint32_t)nl,
              (uint32_t *)g->b_pt[0].p);
    uint64_t na = 0, nw = p, dirty_base = 0;
    for (uint32_t lvl = 0; lvl <= g->h && nw > 0; ++lvl) {   // the root is tested too (R6)
      Lvl a = make_lvl(g, cur, nw, lvl, GPMA_INSERT);
      GP_LAUNCH(g, k_lock_winner, grid_for(nw), TB, 0, s, a.pt, nw, lvl, a.hf);
      GP_CHECK(g, scan_u32(g, a.hf, a.widx, nw, s));
      GP_LAUNCH(g, k_lock_split, grid_for(nw), TB, 0, s, a.pk, a.pv, a.pt, a.hf, a.widx, nw,
                (uint64_t *)g->b_pk[cur ^ 1].p, (uint32_t *)g->b_pv[cur ^ 1].p, (uint32_t *)g->b_pt[cur ^ 1].p, ak,
                av, na);
      GP_CHECK(g, readback(g, &g->ctrl_h->sum, a.widx + nw, 4, s));
      GP_CHECK(g, cudaStreamSynchronize(s));
      const uint64_t q = (uint32_t)g->ctrl_h->sum;      // lock winners at this level
      na += nw - q;
      cur ^= 1;
      nw = q;
      Lvl b = make_lvl(g, cur, nw, lvl, GPMA_INSERT);
      LevelOut lo{};
      if ((st = level_step(g, b, cur, &lo, &dirty_base, s, false, 0, nullptr, nullptr, nullptr))) return st;
      g->last.last_slots_rewritten += lo.nacc * ((uint64_t)g->L << lvl);
      g->last.last_windows_rewritten += lo.nacc;
      if (lvl > g->last.last_top_level) g->last.last_top_level = lvl;
      if (lo.p_new) cur ^= 1;
      nw = lo.p_new;
    }
    if (nw > 0) {                                       // the root could not take it: double, retry
      GP_LAUNCH(g, k_append_kv, grid_for(nw), TB, 0, s, (const uint64_t *)g->b_pk[cur].p,
                (const uint32_t *)g->b_pv[cur].p, nw, ak, av, na);
      na += nw;
      g->last.last_top_level = g->h + 1;
      if ((st = double_root(g, s))) return st;
    } else if (dirty_base) {
      if ((st = fix_heads(g, dirty_base, s))) return st;
    }
    if (na) {                                           // the aborted insertions, sorted again
      Sorted srt;
      if ((st = sort_batch(g, ak, av, na, &srt, s))) return st;
      GP_CHECK(g, cudaMemcpyAsync(g->b_pk[0].p, srt.k, na * 8, cudaMemcpyDeviceToDevice, s));
      GP_CHECK(g, cudaMemcpyAsync(g->b_pv[0].p, srt.v, na * 4, cudaMemcpyDeviceToDevice, s));
    }
    p = na;
  }
  g->last.last_rounds = rounds;
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

static gpma_status status_of(gpma *g) {
  if (g->ctrl_h->err & 2u) return GPMA_ERR_RESERVED;
  if (g->ctrl_h->err & 1u) return GPMA_ERR_RANGE;
  return GPMA_OK;
}

// Strategy switches (read per call; every one is parity-tested): GPMA_DEL_SORT=0 marks lazy
// deletes unsorted (k_lazy_delete), GPMA_INS_FUSED=0 runs the separate insert pre-pass +
// k_level0 instead of the fused k_ins_leaf.
static bool env_on(const char *name) {
  const char *e = getenv(name);
  return !e || atoi(e) != 0;
}

enum { PATH_LAZY_UNSORTED = 0, PATH_LAZY_SORTED, PATH_INS_FUSED, PATH_INS_LEAF, PATH_GENERIC, PATH_INS_SMALL };

// GPMA_INS_THREAD=0: the fused insert leaf step by L-lane sub-warps (k_ins_leaf) instead of a
// thread per leaf group (k_ins_leaf_t, L <= 16)
static int ins_thread_mode() { return env_on("GPMA_INS_THREAD") ? 1 : 0; }

// GPMA_DEL_SORT=1: lazy deletes sorted by key first (k_del_mark) instead of marked in arrival
// order (k_lazy_delete, default: at 1 key per ~16 leaves a sort shares no sector, it only costs);
// GPMA_INS_LEAFSORT=0: inserts sorted by key (k_locate + k_ins_leaf[_t]) instead of located first
// and sorted by target leaf (k_locate_u + k_ins_leaf_u, default).
static int prefix_path(gpma *g, int op) {
  if (op == GPMA_DELETE && g->mode == GPMA_DELETE_LAZY) {
    const char *e = getenv("GPMA_DEL_SORT");
    return (e && atoi(e) != 0) ? PATH_LAZY_SORTED : PATH_LAZY_UNSORTED;
  }
  if (op == GPMA_INSERT && g->algorithm == 0 && !g->trace_on && env_on("GPMA_INS_FUSED"))
    return (g->L <= 16 && env_on("GPMA_INS_LEAFSORT")) ? PATH_INS_LEAF : PATH_INS_FUSED;
  return PATH_GENERIC;
}

// GPMA_ILP = keys per thread of the random-probe kernels (lazy delete, locate): 1, 2 or 4
static int ilp_r() {
  const char *e = getenv("GPMA_ILP");
  return e ? atoi(e) : 2;
}

static int leaf_shifts(uint64_t nleaves, int *sh) {
  const uint32_t bits = nleaves <= 1 ? 1 : ilog2(nleaves - 1) + 1;
  int n = 0;
  for (uint32_t b = 0; b < bits; b += 8) sh[n++] = (int)b;
  return n;
}

// The prefix of one batch, up to and including the read-back of the control block (no host
// synchronisation inside): validate, then
//  * lazy delete: sort the keys, mark the last copy of each (k_del_mark);
//  * insert: sort, locate + group heads (k_locate), scan, group starts, the fused pre-pass +
//    level 0 (k_ins_leaf), scan of the pending flags;
//  * otherwise (strict deletes, GPMA lock-based inserts, traced batches): sort -> pre-pass ->
//    compact -> level 0 (k_level0) unless traced -> summary.
// *srt = the sorted batch.
// 1/V for the interpolation step of the row search (GPMA_INTERP=0: plain binary search; read per
// call).  Every located key has dst < V.
static float interp_fv(gpma *g) {
  const char *e = getenv("GPMA_INTERP");
  if (e && atoi(e) == 0) return 0.f;
  return 1.0f / (float)std::max<uint32_t>(g->V, 1u);
}

static gpma_status upd_prefix(gpma *g, uint64_t *ik, uint32_t *iv, uint64_t n, int op, Sorted *srt,
                              cudaStream_t s) {
  gpma_status st;
  if ((st = zero_ctrl(g, s))) return st;
  GP_LAUNCH(g, k_validate, grid_for(n), TB, 0, s, ik, iv, n, g->V, g->rb, g->nr, op == GPMA_INSERT ? 1 : 0,
            g->ctrl_d);
  const uint64_t nl = g->cap / g->L;
  const uint64_t *ro = g->rows_indexed ? g->row_offset : nullptr;
  const int path = prefix_path(g, op);
  if (path == PATH_LAZY_UNSORTED) {
    const int R = ilp_r();
    if (R >= 4)
      GP_LAUNCH(g, k_lazy_delete_r<4>, grid_for((n + 3) / 4), TB, 0, s, ik, n, g->key, g->val, g->cnt, g->head,
                (uint32_t)nl, g->L, tmask_of(g), g->deg, g->rb, g->ctrl_d, ro, interp_fv(g));
    else if (R == 2)
      GP_LAUNCH(g, k_lazy_delete_r<2>, grid_for((n + 1) / 2), TB, 0, s, ik, n, g->key, g->val, g->cnt, g->head,
                (uint32_t)nl, g->L, tmask_of(g), g->deg, g->rb, g->ctrl_d, ro, interp_fv(g));
    else
      GP_LAUNCH(g, k_lazy_delete, grid_for(n), TB, 0, s, ik, n, g->key, g->val, g->cnt, g->head, (uint32_t)nl, g->L,
                tmask_of(g), g->deg, g->rb, g->ctrl_d, ro);
    GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
    return GPMA_OK;
  }
  if (path == PATH_INS_LEAF) {
    GP_CHECK(g, ensure(g, g->b_keep, (n + 1) * 4, s));
    GP_CHECK(g, ensure(g, g->b_pos, (n + 1) * 4, s));
    if ((st = level_buffers(g, n, s))) return st;
    uint32_t *keep = (uint32_t *)g->b_keep.p, *pos = (uint32_t *)g->b_pos.p;
    uint32_t *keep2 = (uint32_t *)g->b_keep2.p, *kpos = (uint32_t *)g->b_kpos.p;
    GP_CHECK(g, ensure(g, g->b_sk[0], n * 8, s));
    GP_CHECK(g, ensure(g, g->b_sv[0], n * 4, s));
    GP_CHECK(g, ensure(g, g->b_sk[1], n * 8, s));
    GP_CHECK(g, ensure(g, g->b_sv[1], n * 4, s));
    uint64_t *tk0 = (uint64_t *)g->b_sk[0].p, *tk1 = (uint64_t *)g->b_sk[1].p;
    uint32_t *tx0 = (uint32_t *)g->b_sv[0].p, *tx1 = (uint32_t *)g->b_sv[1].p;
    const int R = ilp_r();
    if (R >= 4)
      GP_LAUNCH(g, k_locate_u_r<4>, grid_for((n + 3) / 4), TB, 0, s, ik, n, g->head, (uint32_t)nl, g->L, g->rb, ro, tk0,
                tx0, g->ctrl_d, interp_fv(g));
    else if (R == 2)
      GP_LAUNCH(g, k_locate_u_r<2>, grid_for((n + 1) / 2), TB, 0, s, ik, n, g->head, (uint32_t)nl, g->L, g->rb, ro, tk0,
                tx0, g->ctrl_d, interp_fv(g));
    else
      GP_LAUNCH(g, k_locate_u, grid_for(n), TB, 0, s, ik, n, g->head, (uint32_t)nl, g->L, g->rb, ro, tk0, tx0, g->ctrl_d);
    int sh[8], which = 0;
    const int ns = leaf_shifts(nl, sh);
    GP_CHECK(g, radix_sort_pairs(g, tk0, tx0, tk1, tx1, n, sh, ns, s, &which));
    const uint64_t *tk = which ? tk1 : tk0;
    const uint32_t *tix = which ? tx1 : tx0;
    srt->k = (uint64_t *)tk;
    srt->v = (uint32_t *)tix;
    uint32_t *gid = kpos, *gstart = (uint32_t *)g->b_wfirst.p;
    if (gstart_fused()) {
      if ((st = group_starts(g, tk, n, gstart, gid + n, s))) return st;
    } else {
      uint32_t *hf = keep2;
      GP_LAUNCH(g, k_gflags, grid_for(n), TB, 0, s, tk, n, hf, g->ctrl_d);
      GP_CHECK(g, scan_u32(g, hf, gid, n, s));
      GP_LAUNCH(g, k_gstart, grid_for(n), TB, 0, s, hf, gid, n, gstart, g->ctrl_d);
    }
    const uint32_t bound = (uint32_t)g->tmax[0];
    uint2 *dirty = (uint2 *)g->b_dirty.p;
    GP_CHECK(g, ensure(g, g->b_tgt, (n + 1) * 4, s));
    uint32_t *bigf = (uint32_t *)g->b_tgt.p;
    if (g->L == 16)
      GP_LAUNCH(g, k_ins_leaf_u<16>, grid_for(n, ILU_T), ILU_T, 0, s, ik, iv, tk, tix, gstart, gid + n, g->key, g->val, g->cnt,
                tmask_of(g), g->head, g->row_offset, g->deg, g->rb, bound, keep, bigf, dirty, g->ctrl_d);
    else if (g->L == 8)
      GP_LAUNCH(g, k_ins_leaf_u<8>, grid_for(n, ILU_T), ILU_T, 0, s, ik, iv, tk, tix, gstart, gid + n, g->key, g->val, g->cnt,
                tmask_of(g), g->head, g->row_offset, g->deg, g->rb, bound, keep, bigf, dirty, g->ctrl_d);
    else
      GP_LAUNCH(g, k_ins_leaf_u<4>, grid_for(n, ILU_T), ILU_T, 0, s, ik, iv, tk, tix, gstart, gid + n, g->key, g->val, g->cnt,
                tmask_of(g), g->head, g->row_offset, g->deg, g->rb, bound, keep, bigf, dirty, g->ctrl_d);
    GP_CHECK(g, scan_u32(g, keep, pos, n, s));
    GP_LAUNCH(g, k_upd_summary, 1, 1, 0, s, (const uint32_t *)nullptr, pos, n, g->ctrl_d);
    GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
    return GPMA_OK;
  }
  if ((st = sort_batch(g, ik, op == GPMA_INSERT ? iv : nullptr, n, srt, s))) return st;
  const uint64_t *sk = srt->k;
  const uint32_t *sv = srt->v;
  if (path == PATH_LAZY_SORTED) {
    GP_LAUNCH(g, k_del_mark, grid_for((n + 31) / 32 * 32), 256, 0, s, sk, n, g->key, g->val, g->cnt, g->head,
              (uint32_t)nl, g->L, tmask_of(g), g->deg, g->rb, g->ctrl_d, ro);
    GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
    return GPMA_OK;
  }
  GP_CHECK(g, ensure(g, g->b_keep, (n + 1) * 4, s));
  GP_CHECK(g, ensure(g, g->b_pos, (n + 1) * 4, s));
  GP_CHECK(g, ensure(g, g->b_tgt, (n + 1) * 4, s));
  if ((st = level_buffers(g, n, s))) return st;
  uint32_t *keep = (uint32_t *)g->b_keep.p, *pos = (uint32_t *)g->b_pos.p, *tgt = (uint32_t *)g->b_tgt.p;
  uint32_t *keep2 = (uint32_t *)g->b_keep2.p, *kpos = (uint32_t *)g->b_kpos.p;
  if (path == PATH_INS_FUSED) {
    uint32_t *hf = keep2, *gid = kpos, *gstart = (uint32_t *)g->b_wfirst.p;
    GP_LAUNCH(g, k_locate, grid_for(n, LOC_T), LOC_T, 0, s, sk, n, g->head, (uint32_t)nl, g->L, g->rb, ro, tgt, hf,
              g->ctrl_d);
    GP_CHECK(g, scan_u32(g, hf, gid, n, s));
    GP_LAUNCH(g, k_gstart, grid_for(n), TB, 0, s, hf, gid, n, gstart, g->ctrl_d);
    const uint32_t bound = (uint32_t)g->tmax[0];
    uint2 *dirty = (uint2 *)g->b_dirty.p;
    const int per_thread = ins_thread_mode();
    if (per_thread && g->L == 16)
      GP_LAUNCH(g, k_ins_leaf_t<16>, grid_for(n), 256, 0, s, sk, sv, tgt, gstart, gid + n, g->key, g->val, g->cnt,
                tmask_of(g), g->head, g->row_offset, g->deg, g->rb, bound, keep, dirty, g->ctrl_d);
    else if (per_thread && g->L == 8)
      GP_LAUNCH(g, k_ins_leaf_t<8>, grid_for(n), 256, 0, s, sk, sv, tgt, gstart, gid + n, g->key, g->val, g->cnt,
                tmask_of(g), g->head, g->row_offset, g->deg, g->rb, bound, keep, dirty, g->ctrl_d);
    else if (per_thread && g->L == 4)
      GP_LAUNCH(g, k_ins_leaf_t<4>, grid_for(n), 256, 0, s, sk, sv, tgt, gstart, gid + n, g->key, g->val, g->cnt,
                tmask_of(g), g->head, g->row_offset, g->deg, g->rb, bound, keep, dirty, g->ctrl_d);
    else
      GP_LAUNCH(g, k_ins_leaf, grid_for((n + 31) / 32 * 32, IL_T), IL_T, 0, s, sk, sv, tgt, gstart, gid + n, g->key,
                g->val, g->cnt, tmask_of(g), g->head, g->row_offset, g->deg, g->rb, g->L, bound, keep, dirty,
                g->ctrl_d);
    GP_CHECK(g, scan_u32(g, keep, pos, n, s));
    GP_LAUNCH(g, k_upd_summary, 1, 1, 0, s, (const uint32_t *)nullptr, pos, n, g->ctrl_d);
    GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
    return GPMA_OK;
  }
  GP_LAUNCH(g, k_prepass, (unsigned)((n + TB - 1) / TB), TB, 0, s, sk, sv, n, g->key, g->val, g->cnt, g->head,
            (uint32_t)nl, g->L, op, (int)g->mode, keep, tgt, g->ctrl_d, tmask_of(g), g->deg, g->rb, ro);
  GP_CHECK(g, scan_u32(g, keep, pos, n, s));
  GP_LAUNCH(g, k_compact_pending, grid_for(n), TB, 0, s, keep, pos, n, sk, sv, tgt, (uint64_t *)g->b_pk[0].p,
            (uint32_t *)g->b_pv[0].p, (uint32_t *)g->b_pt[0].p, g->ctrl_d);
  const bool lock = op == GPMA_INSERT && g->algorithm == 1;   // GPMA (Alg. 1) instead of GPMA+
  const bool fused = !g->trace_on && !lock;   // the per-level trace needs the generic level-0 step
  if (fused) {
    // level 0 fused: one warp per leaf group, sized by n, counts read on the device
    GP_CHECK(g, fill_zero(g, keep2, (n + 1) * 4, s));
    const uint32_t bound = (uint32_t)(op == GPMA_INSERT ? g->tmax[0] : g->tmin[0]);
    GP_LAUNCH(g, k_level0, grid_for((n + 31) / 32 * 32), 256, 0, s, (const uint64_t *)g->b_pk[0].p,
              (const uint32_t *)g->b_pv[0].p, (const uint32_t *)g->b_pt[0].p, pos + n, g->key, g->val, g->cnt,
              tmask_of(g), g->head, g->row_offset, g->rb, g->L, bound, op, keep2, (uint2 *)g->b_dirty.p,
              g->ctrl_d);
    GP_CHECK(g, scan_u32(g, keep2, kpos, n, s));
  }
  GP_LAUNCH(g, k_upd_summary, 1, 1, 0, s, pos, fused ? kpos : nullptr, n, g->ctrl_d);
  GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
  return GPMA_OK;
}

// GPMA_SMALL=0 disables the one-kernel small-batch path; GPMA_SMALL=<n> sets the largest batch it
// takes (inserts <= min(n, 2048), lazy deletes <= min(n, 4096)).  Default: every batch up to those
// maxima -- measured (configs[1], tools/r02_small_sweep2.sh): insert call 46 vs 66 us at 1000 keys
// and 68 vs 75 at 2000 against the multi-kernel path, lazy delete 27 vs 33 at both.  Read per call.
static bool small_batch_path(gpma *g, uint64_t n, int op, int path) {
  uint64_t lim_ins = SB_MAX, lim_del = SB_DEL_MAX;
  if (const char *e = getenv("GPMA_SMALL")) {
    const uint64_t lim = (uint64_t)atoll(e);
    lim_ins = std::min<uint64_t>(lim, SB_MAX);
    lim_del = std::min<uint64_t>(lim, SB_DEL_MAX);
  }
  if (path == PATH_LAZY_UNSORTED || path == PATH_LAZY_SORTED) return n <= lim_del;
  if (path == PATH_INS_LEAF || path == PATH_INS_FUSED)
    return n <= lim_ins && (g->L == 4 || g->L == 8 || g->L == 16);
  return false;
}

static uint32_t next_seq(gpma *g) {
  if (++g->ctrl_seq == 0) g->ctrl_seq = 1;            // 0: what the mirror copies before the number
  return g->ctrl_seq;
}

// Wait for the one-kernel call's control block: spin on its sequence number in pinned memory
// (GPMA_SPIN=0: cudaStreamSynchronize).  The stream is polled now and then, so a failed kernel
// (which never writes the number) surfaces its error instead of hanging the host.
static cudaError_t wait_ctrl(gpma *g, cudaStream_t s) {
  static const bool spin = [] {
    const char *e = getenv("GPMA_SPIN");
    return !e || atoi(e) != 0;
  }();
  if (spin) {
    const volatile uint32_t *q = &g->ctrl_h->seq;
    for (uint64_t it = 1;; ++it) {
      if (*q == g->ctrl_seq) {
        std::atomic_thread_fence(std::memory_order_acquire);
        return cudaSuccess;
      }
      if ((it & 4095) == 0) {
        const cudaError_t e = cudaStreamQuery(s);
        if (e == cudaSuccess) break;                     // done without the number: let sync decide
        if (e != cudaErrorNotReady) return e;
      }
    }
  }
  return cudaStreamSynchronize(s);
}

static gpma_status run_small(gpma *g, uint64_t *ik, uint32_t *iv, uint64_t n, int op, cudaStream_t s) {
  const uint64_t nl = g->cap / g->L;
  const uint64_t *ro = g->rows_indexed ? g->row_offset : nullptr;
  if (op == GPMA_DELETE) {
    GP_LAUNCH(g, k_small_delete, (unsigned)std::max<uint64_t>(1, (n + 2 * SD_T - 1) / (2 * SD_T)), SD_T, 0, s, ik,
              (uint32_t)n, g->key, g->val, g->cnt, g->head, (uint32_t)nl, g->L,
              tmask_of(g), g->deg, g->rb, g->nr, g->V, ro, g->ctrl_d, g->ctrl_h, next_seq(g), interp_fv(g));
    GP_CHECK(g, cudaGetLastError());
    return GPMA_OK;
  }
  gpma_status st;
  if ((st = level_buffers(g, n, s))) return st;
  static const bool attr = [] {
    cudaFuncSetAttribute(k_small_insert<16>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sb_smem_bytes(16));
    cudaFuncSetAttribute(k_small_insert<8>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sb_smem_bytes(8));
    cudaFuncSetAttribute(k_small_insert<4>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)sb_smem_bytes(4));
    return true;
  }();
  (void)attr;
  const uint32_t bound = (uint32_t)g->tmax[0];
  uint64_t *pk = (uint64_t *)g->b_pk[0].p;
  uint32_t *pv = (uint32_t *)g->b_pv[0].p, *pt = (uint32_t *)g->b_pt[0].p;
  uint2 *dirty = (uint2 *)g->b_dirty.p;
#define GP_SMALL_INS(LL)                                                                                         \
  GP_LAUNCH(g, k_small_insert<LL>, 1, SB_T, sb_smem_bytes(LL), s, ik, iv, (uint32_t)n, g->key, g->val, g->cnt,   \
            tmask_of(g), g->head, g->row_offset, g->deg, (uint32_t)nl, g->rb, g->nr, g->V, bound, ro, pk, pv, pt, \
            dirty, g->ctrl_d, g->ctrl_h, seq, pbd, interp_fv(g))
  const uint32_t seq = next_seq(g);
  auto bits = [](uint64_t x) { uint32_t b = 1; while ((1ull << b) < x) ++b; return b; };
  const uint32_t pbd0 = bits(g->V);
  const uint32_t pbd = bits(g->nr) + pbd0 + 11 <= 64 ? pbd0 : 0u;   // packed sort keys fit
  if (g->L == 16) GP_SMALL_INS(16);
  else if (g->L == 8) GP_SMALL_INS(8);
  else GP_SMALL_INS(4);
#undef GP_SMALL_INS
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// everything the prefix bakes into its launches
static std::vector<uint64_t> upd_signature(gpma *g, uint64_t n, int op) {
  std::vector<uint64_t> v = {n, (uint64_t)op, (uint64_t)prefix_path(g, op), g->mode, g->algorithm, g->V, g->rb,
                             g->nr, g->cap, g->L, g->h,
                             g->tmax.empty() ? 0 : g->tmax[0], g->tmin.empty() ? 0 : g->tmin[0],
                             (uint64_t)g->rows_indexed, (uint64_t)g->trace_on,
                             (uint64_t)(uintptr_t)g->key, (uint64_t)(uintptr_t)g->val, (uint64_t)(uintptr_t)g->cnt,
                             (uint64_t)(uintptr_t)g->deg, (uint64_t)(uintptr_t)g->head,
                             (uint64_t)(uintptr_t)g->row_offset, (uint64_t)(uintptr_t)g->ctrl_d,
                             (uint64_t)(uintptr_t)g->ctrl_h, (uint64_t)(uintptr_t)tl_scan};
  const DevBuf *bufs[] = {&g->b_sk[0], &g->b_sk[1], &g->b_sv[0], &g->b_sv[1], &g->b_keep, &g->b_pos, &g->b_tgt,
                          &g->b_pk[0], &g->b_pk[1], &g->b_pv[0], &g->b_pv[1], &g->b_pt[0], &g->b_pt[1],
                          &g->b_hf, &g->b_widx, &g->b_wfirst, &g->b_acc, &g->b_aidx, &g->b_alist, &g->b_nw,
                          &g->b_woff, &g->b_keep2, &g->b_kpos, &g->b_lpre, &g->b_wk, &g->b_wv, &g->b_dirty,
                          &g->b_scan, &g->b_hist, &g->b_stage[0], &g->b_stage[1], &g->b_stage[2],
                          &g->b_stage[3], &g->b_misc, &g->b_misc2, &g->b_misc3, &g->b_sup};
  for (const DevBuf *b : bufs) {
    v.push_back((uint64_t)(uintptr_t)b->p);
    v.push_back(b->bytes);
  }
  return v;
}

// GPMA_UPD_GRAPH=0 disables graph replay (read per call)
// The per-launch profiler cannot see inside a replayed graph: replay stays on unless the filter
// names a kernel of the replayed prefix ("*" or one of them), so profiling an analytics kernel
// (bench.py's roofline) times the same update path as an unprofiled run.
static bool prof_sees_prefix(const std::string &f) {
  if (f.empty()) return false;
  if (f == "*") return true;
  static const char *pre[] = {"k_validate", "k_lazy", "k_prepass", "k_level0", "k_os_", "k_small_sort",
                              "k_scan", "k_compact", "k_upd", "k_zero", "k_copy", "k_readback", "k_locate",
                              "k_del", "k_gflags", "k_gstart", "k_ins_leaf", "k_pend"};
  for (const char *p : pre)
    if (f.find(p) != std::string::npos) return true;
  return false;
}

static bool upd_graph_on(gpma *g) {
  if (g->graphs_off || g->trace_on || prof_sees_prefix(g->prof_filter)) return false;
  const char *e = getenv("GPMA_UPD_GRAPH");
  return !e || atoi(e) != 0;
}

// Run the prefix: replay the cached graph when the signature matches; capture it on the second
// run of an unchanged shape (the first run sized every buffer, so the capture allocates
// nothing); plain launches otherwise.
static gpma_status run_prefix(gpma *g, uint64_t *ik, uint32_t *iv, uint64_t n, int op, Sorted *srt,
                              cudaStream_t s) {
  if (!s || !upd_graph_on(g)) return upd_prefix(g, ik, iv, n, op, srt, s);   // (no capture on the legacy stream)
  UpdGraph &G = g->ugraph[op == GPMA_INSERT ? 0 : 1];
  std::vector<uint64_t> sig = upd_signature(g, n, op);
  if (G.exec && G.sig == sig) {
    GP_CHECK(g, cudaGraphLaunch(G.exec, s));
    g->launches += G.nlaunch;
    srt->k = (uint64_t *)G.srt[0];
    srt->v = (uint32_t *)G.srt[1];
    srt->ok = (uint64_t *)G.srt[2];
    srt->ov = (uint32_t *)G.srt[3];
    return GPMA_OK;
  }
  if (G.seen != sig) {
    gpma_status st = upd_prefix(g, ik, iv, n, op, srt, s);
    G.seen = upd_signature(g, n, op);
    return st;
  }
  cudaGraph_t graph = nullptr;
  const uint64_t l0 = g->launches;
  GP_CHECK(g, cudaStreamBeginCapture(s, cudaStreamCaptureModeRelaxed));
  gpma_status st = upd_prefix(g, ik, iv, n, op, srt, s);
  cudaError_t e = cudaStreamEndCapture(s, &graph);
  if (st) return st;
  cudaGraphExec_t exec = nullptr;
  if (e == cudaSuccess && upd_signature(g, n, op) == sig) e = cudaGraphInstantiate(&exec, graph, 0);
  else if (e == cudaSuccess) e = cudaErrorNotSupported;   // the capture allocated: never replay it
  if (graph) cudaGraphDestroy(graph);
  if (e != cudaSuccess) {                 // fall back for good; run the prefix plainly now
    cudaGetLastError();
    g->graphs_off = true;
    g->launches = l0;
    return upd_prefix(g, ik, iv, n, op, srt, s);
  }
  if (G.exec) cudaGraphExecDestroy(G.exec);
  G.exec = exec;
  G.sig = sig;
  G.nlaunch = g->launches - l0;
  G.srt[0] = srt->k;
  G.srt[1] = srt->v;
  G.srt[2] = srt->ok;
  G.srt[3] = srt->ov;
  GP_CHECK(g, cudaGraphLaunch(exec, s));
  return GPMA_OK;
}

// One batch.  Validation runs on the device and every mutating kernel bails out when it
// flagged the batch, so the common insert path (sort -> pre-pass -> fused level 0) needs a
// single host round trip; the generic levels >= 1 and the resize follow only when level 0
// leaves updates pending.
static gpma_status update_after_prefix(gpma *g, const uint64_t *ik, const uint32_t *iv, uint64_t n, int op, int path,
                                       const Sorted &srt, cudaStream_t s);

static bool is_device_ptr(const void *p) {
  if (!p) return false;
  cudaPointerAttributes a{};
  if (cudaPointerGetAttributes(&a, p) != cudaSuccess) {
    cudaGetLastError();
    return false;
  }
  return a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged;
}

gpma_status update_batch(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, int op,
                         cudaStream_t s) {
  gpma_status st;
  g->last = gpma_stats_t{};
  g->trace.clear();
  if (n == 0) return GPMA_OK;
  tl_call_start = std::chrono::steady_clock::now();
  int path = prefix_path(g, op);
  Sorted srt;
  Nvtx nvtx_(op == GPMA_INSERT ? "update: insert prefix" : "update: delete prefix");
  if (small_batch_path(g, n, op, path) && is_device_ptr(keys) && (op != GPMA_INSERT || is_device_ptr(vals))) {
    // the one-kernel small batch only reads the batch: no staging copy of a device batch
    if ((st = run_small(g, const_cast<uint64_t *>(keys), const_cast<uint32_t *>(vals), n, op, s))) return st;
    path = path == PATH_INS_LEAF || path == PATH_INS_FUSED ? PATH_INS_SMALL : path;
    GP_CHECK(g, wait_ctrl(g, s));
    if (path == PATH_LAZY_UNSORTED || path == PATH_LAZY_SORTED) {
      g->last.last_unique = n;
      return status_of(g);
    }
    return update_after_prefix(g, keys, vals, n, op, path, srt, s);
  }
  // GPMA_DIRECT=1: large device batches on the paths that only READ the batch (leaf-keyed insert,
  // unsorted lazy delete) skip the staging copy and the graph (which needs the stable staged
  // address).  Measured off by default: 25 configs[2] slides, insert 0.586 (direct) vs 0.561 ms
  // (staged + graph-replayed prefix: the short kernels of the prefix wait on host launches
  // otherwise), delete 0.258 vs 0.255 ms.
  const char *de = n >= (1u << 16) ? getenv("GPMA_DIRECT") : nullptr;   // (read per large call)
  const bool direct_on = de && atoi(de) != 0;
  if (direct_on && n >= (1u << 16) && (path == PATH_INS_LEAF || path == PATH_LAZY_UNSORTED) && is_device_ptr(keys) &&
      (op != GPMA_INSERT || is_device_ptr(vals))) {
    uint64_t *dk = const_cast<uint64_t *>(keys);
    uint32_t *dv = const_cast<uint32_t *>(vals);
    if ((st = upd_prefix(g, dk, dv, n, op, &srt, s))) return st;
    GP_CHECK(g, cudaStreamSynchronize(s));           // the one host round trip of the batch
    if (path == PATH_LAZY_UNSORTED) {
      g->last.last_unique = n;
      return status_of(g);
    }
    return update_after_prefix(g, dk, dv, n, op, path, srt, s);
  }
  GP_CHECK(g, ensure(g, g->b_stage[0], n * 8, s));
  GP_CHECK(g, ensure(g, g->b_stage[1], n * 4, s));
  uint64_t *ik = (uint64_t *)g->b_stage[0].p;
  uint32_t *iv = (uint32_t *)g->b_stage[1].p;
  GP_CHECK(g, stage_in(g, ik, keys, n * 8, s));
  if (op == GPMA_INSERT) GP_CHECK(g, stage_in(g, iv, vals, n * 4, s));
  const bool small = small_batch_path(g, n, op, path);
  if (small) {
    if ((st = run_small(g, ik, iv, n, op, s))) return st;
    path = path == PATH_INS_LEAF || path == PATH_INS_FUSED ? PATH_INS_SMALL : path;
  } else if ((st = run_prefix(g, ik, iv, n, op, &srt, s))) {
    return st;
  }
  GP_CHECK(g, small ? wait_ctrl(g, s) : cudaStreamSynchronize(s));   // the one host round trip of the batch
  if (path == PATH_LAZY_UNSORTED || path == PATH_LAZY_SORTED) {
    g->last.last_unique = n;   // (lazy deletes are idempotent; the sorted path marks each key once)
    return status_of(g);
  }
  return update_after_prefix(g, ik, iv, n, op, path, srt, s);
}

__global__ void k_big_gather(const uint32_t *__restrict__ bigf, const uint32_t *__restrict__ bpos, uint64_t n,
                             const uint32_t *__restrict__ tix, const uint64_t *__restrict__ ik,
                             const uint32_t *__restrict__ iv, uint64_t *__restrict__ bk, uint32_t *__restrict__ bv) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < n; j += (uint64_t)gridDim.x * blockDim.x)
    if (bigf[j]) {
      const uint32_t i = tix[j];
      bk[bpos[j]] = ik[i];
      bv[bpos[j]] = iv[i];
    }
}

__global__ void k_iota(uint32_t *__restrict__ out, uint64_t n, uint32_t base) {
  for (uint64_t j = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; j < n; j += (uint64_t)gridDim.x * blockDim.x)
    out[j] = base + (uint32_t)j;
}

// Level 0 for the updates of oversized leaf groups (flagged by k_ins_leaf_u in b_tgt): compact,
// sort by key (stable: copies adjacent, the last wins, R10), locate, group, merge with the
// sub-warp leaf kernel (any group size); the rejected keys are appended to the pending list at
// (pk, pv, pt, seq) with sequence numbers from seq0.  The control block keeps accumulating.
static gpma_status big_groups(gpma *g, const uint64_t *ik, const uint32_t *iv, uint64_t n, const Sorted &srt,
                              uint64_t nbig, uint64_t *pk, uint32_t *pv, uint32_t *pt, uint32_t *seq, uint64_t seq0,
                              uint64_t *p2, cudaStream_t s) {
  const uint64_t nl = g->cap / g->L;
  const uint64_t *ro = g->rows_indexed ? g->row_offset : nullptr;
  uint32_t *bigf = (uint32_t *)g->b_tgt.p, *bpos = (uint32_t *)g->b_kpos.p;
  GP_CHECK(g, scan_u32(g, bigf, bpos, n, s));
  GP_CHECK(g, ensure(g, g->b_stage[2], nbig * 8 + 16, s));
  GP_CHECK(g, ensure(g, g->b_stage[3], nbig * 4 + 16, s));
  uint64_t *bk = (uint64_t *)g->b_stage[2].p;
  uint32_t *bv = (uint32_t *)g->b_stage[3].p;
  GP_LAUNCH(g, k_big_gather, grid_for(n), TB, 0, s, bigf, bpos, n, (const uint32_t *)srt.v, ik, iv, bk, bv);
  Sorted s2;
  gpma_status st = sort_batch(g, bk, bv, nbig, &s2, s);
  if (st) return st;
  uint32_t *tgt = bigf, *hf = (uint32_t *)g->b_acc.p, *gid = bpos, *gstart = (uint32_t *)g->b_wfirst.p;
  uint32_t *keep = (uint32_t *)g->b_keep.p, *pos = (uint32_t *)g->b_pos.p;
  GP_LAUNCH(g, k_locate, grid_for(nbig, LOC_T), LOC_T, 0, s, s2.k, nbig, g->head, (uint32_t)nl, g->L, g->rb, ro, tgt, hf,
            g->ctrl_d);
  GP_CHECK(g, scan_u32(g, hf, gid, nbig, s));
  GP_LAUNCH(g, k_gstart, grid_for(nbig), TB, 0, s, hf, gid, nbig, gstart, g->ctrl_d);
  GP_LAUNCH(g, k_ins_leaf, grid_for((nbig + 31) / 32 * 32, IL_T), IL_T, 0, s, s2.k, s2.v, tgt, gstart, gid + nbig,
            g->key, g->val, g->cnt, tmask_of(g), g->head, g->row_offset, g->deg, g->rb, g->L, (uint32_t)g->tmax[0], keep,
            (uint2 *)g->b_dirty.p, g->ctrl_d);
  GP_CHECK(g, scan_u32(g, keep, pos, nbig, s));
  GP_CHECK(g, readback(g, g->pin, pos + nbig, 4, s));
  GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  uint32_t m;
  memcpy(&m, g->pin, 4);
  *p2 = m;
  if (m) {
    GP_LAUNCH(g, k_compact_pending, grid_for(nbig), TB, 0, s, keep, pos, nbig, s2.k, s2.v, tgt, pk, pv, pt, g->ctrl_d);
    GP_LAUNCH(g, k_iota, grid_for(m), TB, 0, s, seq, (uint64_t)m, (uint32_t)seq0);
  }
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

// ---- dead-level skip (exact).  A window's density-test value -- n_W + |U_W| for inserts,
// n_W - |D_W| for strict deletes (Alg. 4 l.23-25) -- does not change when its sub-windows absorb
// their updates at lower levels: absorbed updates move from pending to live (or leave both
// counts).  So from the current leaf live counts and pending list, one pass finds the lowest level
// in [lvl0, lvl1) at which some window holding pending updates would accept; the levels below it
// change nothing (no window accepts, the pending list is carried up unchanged) and are skipped.
// A root-bound climb (a resizing batch) then goes from the first empty level straight to the root.
__global__ void k_set_u32(uint32_t *p, uint32_t v) { *p = v; }

struct LvlBound {
  uint64_t t[64];       // max_i (insert) or min_i (strict delete) per level
};
__global__ void k_lvl_first_accept(const uint32_t *__restrict__ pt, uint64_t p, const uint32_t *__restrict__ pre,
                                   uint32_t lvl0, uint32_t lvl1, LvlBound tb, int op, uint32_t *first) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < p; i += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t t = pt[i];
    const uint32_t tp = i ? pt[i - 1] : 0u;
    uint64_t e = i + 1;                        // end of i's window at the level below (exclusive)
    for (uint32_t j = lvl0; j < lvl1; ++j) {
      if (j >= *(volatile uint32_t *)first) break;          // a lower accepting level is known
      if (i && (tp >> j) == (t >> j)) break;                 // not the window's first update
      const uint32_t w = t >> j;
      uint64_t lo = e, hi = e, step = 1;                     // first index past the window
      while (hi < p && (pt[hi] >> j) == w) {
        lo = hi + 1;
        hi += step;
        step <<= 1;
      }
      if (hi > p) hi = p;
      while (lo < hi) {
        const uint64_t mid = (lo + hi) >> 1;
        if ((pt[mid] >> j) == w) lo = mid + 1;
        else hi = mid;
      }
      e = lo;
      const uint64_t a0 = (uint64_t)w << j, a1 = (uint64_t)(w + 1) << j;
      const uint64_t n = (uint64_t)(pre[a1] - pre[a0]);
      const uint64_t u = e - i;
      const bool ok = op == GPMA_INSERT ? n + u <= tb.t[j] : (n >= u && n - u >= tb.t[j]);
      if (ok) {
        atomicMin(first, j);
        break;
      }
    }
  }
}

// Root reach (exact, the same invariant): an update reaches the root iff the test fails for every
// window of its chain (levels lvl0 .. h-1); then the root is tested and re-lays out the whole
// array -- in place or resized -- from all live entries and all pending updates, so every
// rewrite of a lower window is overwritten and the levels below the root can be jumped over
// (the layout is the same).  One thread per window of level lvl0 (its first pending update)
// walks up its chain, the window bounds in the sorted pending list widened by exponential
// searches, and stops at the first window that accepts (also its chain's absorption level:
// the minimum over chains is the lowest accepting level, as k_lvl_first_accept).
__device__ __forceinline__ uint64_t pend_lo(const uint32_t *pt, uint64_t lo, uint32_t l, uint32_t w) {
  // pt[lo] is in window w (pt >> l is non-decreasing): the window's first index
  uint64_t good = lo, step = 1, bad;
  for (;;) {
    if (good == 0) return 0;
    const uint64_t probe = good > step ? good - step : 0;
    if ((pt[probe] >> l) == w) {
      good = probe;
      step <<= 1;
    } else {
      bad = probe;
      break;
    }
  }
  while (bad + 1 < good) {                               // pt[bad] outside, pt[good] inside
    const uint64_t mid = (bad + good) >> 1;
    if ((pt[mid] >> l) == w) good = mid;
    else bad = mid;
  }
  return good;
}
__device__ __forceinline__ uint64_t pend_hi(const uint32_t *pt, uint64_t p, uint64_t hi, uint32_t l, uint32_t w) {
  uint64_t lo = hi, step = 1;                            // first index past the window
  while (hi < p && (pt[hi] >> l) == w) {
    lo = hi + 1;
    hi += step;
    step <<= 1;
  }
  if (hi > p) hi = p;
  while (lo < hi) {
    const uint64_t mid = (lo + hi) >> 1;
    if ((pt[mid] >> l) == w) lo = mid + 1;
    else hi = mid;
  }
  return lo;
}
__global__ void k_lvl_root_reach(const uint32_t *__restrict__ pt, uint64_t p, const uint32_t *__restrict__ pre,
                                 uint32_t lvl0, uint32_t lvl1, LvlBound tb, int op, uint32_t *first,
                                 uint32_t *root, uint32_t *sup, uint64_t nl) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < p; i += (uint64_t)gridDim.x * blockDim.x) {
    const uint32_t t = pt[i];
    if (i && (pt[i - 1] >> lvl0) == (t >> lvl0)) continue;   // not its level-lvl0 window's first
    uint64_t lo = i, hi = i + 1;
    bool passed = false;
    for (uint32_t l = lvl0; l < lvl1 && !passed; ++l) {
      const uint32_t w = t >> l;
      lo = pend_lo(pt, lo, l, w);
      hi = pend_hi(pt, p, hi, l, w);
      const uint64_t n = (uint64_t)(pre[(uint64_t)(w + 1) << l] - pre[(uint64_t)w << l]);
      const uint64_t u = hi - lo;
      if (op == GPMA_INSERT ? n + u <= tb.t[l] : (n >= u && n - u >= tb.t[l])) {
        atomicMin(first, l);
        if (sup) {                                       // the chain's truly accepted window
          const uint64_t id = (nl >> l) + w;
          atomicOr(sup + (id >> 5), 1u << (id & 31));
        }
        passed = true;
      }
    }
    if (!passed) atomicOr(root, 1u);
  }
}

// the levels that hold a maximal truly accepted window (bit l of *mask): one thread per word of
// the heap-indexed bitmap
__global__ void k_lvl_maximal(const uint32_t *__restrict__ sup, uint64_t nwords, uint64_t nl,
                              unsigned long long *mask) {
  const uint32_t H = 63 - __clzll((long long)nl);        // log2(nl): level of id 1
  unsigned long long m = 0;
  for (uint64_t wd = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; wd < nwords;
       wd += (uint64_t)gridDim.x * blockDim.x) {
    uint32_t b = sup[wd];
    while (b) {
      const int k = __ffs(b) - 1;
      b &= b - 1;
      const uint64_t id = wd * 32 + (uint64_t)k;
      const uint32_t l = H - (63 - __clzll((long long)id));   // (nl >> l) <= id < 2 (nl >> l)
      const uint64_t w = id - (nl >> l);
      if (!lvl_superseded(sup, nl, l, w)) m |= 1ull << l;
    }
  }
  for (int o = 16; o; o >>= 1) m |= __shfl_xor_sync(0xffffffffu, m, o);
  if ((threadIdx.x & 31) == 0 && m) atomicOr(mask, m);
}

// GPMA_TRACE_LEVELS=1: every host-driven level of a batch on stderr (diagnostics)
static bool trace_levels() {
  static const bool on = [] {
    const char *e = getenv("GPMA_TRACE_LEVELS");
    return e && atoi(e) != 0;
  }();
  return on;
}

// GPMA_LVL_SKIP=0 disables the dead-level skip (read per call)
static bool lvl_skip_on() {
  const char *e = getenv("GPMA_LVL_SKIP");
  return !e || atoi(e) != 0;
}
constexpr uint64_t SKIP_MINP = 256;     // pending updates worth the prefix of the counts

// the lowest level in [lvl0, lvl1) at which a window of the pending list (buffers cur) accepts,
// lvl1 if none
// (root != nullptr: the per-chain walk of k_lvl_root_reach, which also tells whether some update
// reaches the root)
static gpma_status first_accept_level(gpma *g, int cur, uint64_t p, uint32_t lvl0, uint32_t lvl1, int op,
                                      uint32_t *out, cudaStream_t s, bool *root = nullptr) {
  const uint64_t nl = g->cap / g->L;
  GP_CHECK(g, ensure(g, g->b_misc3, (nl + 4) * 4, s));
  uint32_t *pre = (uint32_t *)g->b_misc3.p, *first = pre + nl + 1, *rf = pre + nl + 2;
  GP_CHECK(g, scan_u32(g, g->cnt, pre, nl, s));
  GP_LAUNCH(g, k_set_u32, 1, 1, 0, s, first, lvl1);
  if (root) GP_LAUNCH(g, k_set_u32, 1, 1, 0, s, rf, 0u);
  LvlBound tb{};
  const std::vector<uint64_t> &b = op == GPMA_INSERT ? g->tmax : g->tmin;
  for (uint32_t j = 0; j < 64 && j < b.size(); ++j) tb.t[j] = b[j];
  if (root)
    GP_LAUNCH(g, k_lvl_root_reach, grid_for(p), TB, 0, s, (const uint32_t *)g->b_pt[cur].p, p, pre, lvl0, lvl1, tb,
              op, first, rf, (uint32_t *)nullptr, nl);
  else
    GP_LAUNCH(g, k_lvl_first_accept, grid_for(p), TB, 0, s, (const uint32_t *)g->b_pt[cur].p, p, pre, lvl0, lvl1,
              tb, op, first);
  GP_CHECK(g, readback(g, g->pin, first, 8, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  uint32_t w2[2];
  memcpy(w2, g->pin, 8);
  *out = w2[0];
  if (root) *root = w2[1] != 0;
  return GPMA_OK;
}

// GPMA_ROOT_JUMP=0 disables the root-reach jump (read per call)
static bool root_jump_on() {
  const char *e = getenv("GPMA_ROOT_JUMP");
  return !e || atoi(e) != 0;
}

// GPMA_LVL_PLAN=0 disables the climb plan (read per call)
static bool lvl_plan_on() {
  const char *e = getenv("GPMA_LVL_PLAN");
  return !e || atoi(e) != 0;
}

// The plan of a host-driven climb from level lvl0 (exact, the dead-level skip's invariant): every
// chain's truly accepted window (its first passing window) marked in b_sup, whether some chain
// reaches the root, and the levels holding a maximal (not superseded) truly accepted window.
// Only those levels -- and the root, if reached -- need stepping; there the superseded windows
// are rejected (their updates are merged by the window above), so the final layout is the one
// the level-by-level loop produces, with each region rewritten once.
static gpma_status plan_levels(gpma *g, int cur, uint64_t p, uint32_t lvl0, int op, bool *root, uint64_t *mask,
                               cudaStream_t s) {
  const uint64_t nl = g->cap / g->L;
  const uint64_t nwords = (2 * nl + 31) / 32;
  GP_CHECK(g, ensure(g, g->b_misc3, (nl + 8) * 4, s));
  GP_CHECK(g, ensure(g, g->b_sup, nwords * 4 + 16, s));
  uint32_t *pre = (uint32_t *)g->b_misc3.p, *first = pre + nl + 1, *rf = pre + nl + 2;
  unsigned long long *mk = reinterpret_cast<unsigned long long *>(pre + nl + 4);   // 8-B aligned (nl even)
  uint32_t *sup = (uint32_t *)g->b_sup.p;
  GP_CHECK(g, scan_u32(g, g->cnt, pre, nl, s));
  GP_CHECK(g, fill_zero(g, sup, nwords * 4, s));
  GP_CHECK(g, fill_zero(g, first, 5 * 4, s));          // first, root, pad, mask
  LvlBound tb{};
  const std::vector<uint64_t> &b = op == GPMA_INSERT ? g->tmax : g->tmin;
  for (uint32_t j = 0; j < 64 && j < b.size(); ++j) tb.t[j] = b[j];
  GP_LAUNCH(g, k_lvl_root_reach, grid_for(p), TB, 0, s, (const uint32_t *)g->b_pt[cur].p, p, pre, lvl0, g->h, tb, op,
            first, rf, sup, nl);
  GP_LAUNCH(g, k_lvl_maximal, grid_for(nwords), TB, 0, s, (const uint32_t *)sup, nwords, nl, mk);
  GP_CHECK(g, readback(g, g->pin, first, 5 * 4, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  uint32_t w[5];
  memcpy(w, g->pin, 20);
  *root = w[1] != 0;
  *mask = (uint64_t)w[3] | ((uint64_t)w[4] << 32);
  return GPMA_OK;
}

// After the prefix's host round trip: the pending list of level 1 (if any), the level loop, the
// root resize, the head fix-up.  ik / iv: the batch the prefix read (staged or the caller's).
static gpma_status update_after_prefix(gpma *g, const uint64_t *ik, const uint32_t *iv, uint64_t n, int op, int path,
                                       const Sorted &srt, cudaStream_t s) {
  gpma_status st;
  uint32_t *keep2 = (uint32_t *)g->b_keep2.p, *kpos = (uint32_t *)g->b_kpos.p;
  const bool lock = op == GPMA_INSERT && g->algorithm == 1;   // GPMA (Alg. 1) instead of GPMA+
  const bool fused = !g->trace_on && !lock;
  if ((st = status_of(g))) return st;
  g->big_dirty.clear();
  g->sup_on = false;
  uint64_t p = (uint32_t)g->ctrl_h->sum;
  g->last.last_unique = g->ctrl_h->nunique;
  g->last.last_pending = p;
  if (p == 0 && !g->ctrl_h->big) return GPMA_OK;       // (oversized leaf groups still to do)
  if (lock) return gpma_lock_insert(g, p, s);
  int cur = 0;
  uint64_t dirty_base = 0;
  uint32_t lvl = 0;
  if (path == PATH_INS_SMALL) {
    // the one-kernel small batch left the rejected keys key-sorted in the level-1 buffers
    const uint64_t p_new = (uint32_t)g->ctrl_h->sum2;
    dirty_base = g->ctrl_h->ndirty;
    g->last.last_slots_rewritten += g->ctrl_h->windows_rewritten * g->L;
    g->last.last_windows_rewritten += g->ctrl_h->windows_rewritten;
    g->last.last_level0_windows = g->ctrl_h->windows_rewritten;
    if (p_new) g->last.last_top_level = 1;
    p = p_new;
    lvl = 1;
  } else if (path == PATH_INS_LEAF) {
    // pending after level 0: the new keys the leaves rejected, gathered in leaf order, then put
    // in key order (the level loop's pending lists are key-sorted, Alg. 4 l.12-15)
    uint64_t p_new = (uint32_t)g->ctrl_h->sum2;
    uint64_t *pk1 = (uint64_t *)g->b_pk[1].p;
    uint32_t *pv1 = (uint32_t *)g->b_pv[1].p, *pt1 = (uint32_t *)g->b_pt[1].p, *seq = (uint32_t *)g->b_keep2.p;
    if (p_new)
      GP_LAUNCH(g, k_pend_gather, grid_for(n), TB, 0, s, (const uint32_t *)g->b_keep.p, (const uint32_t *)g->b_pos.p,
                n, (const uint32_t *)srt.v, (const uint64_t *)srt.k, ik, iv, pk1, pv1, pt1, seq);
    if (g->ctrl_h->big) {
      // oversized leaf groups (an adversarial batch piling into one leaf): the key-sorted fused
      // path on their updates -- compacted in leaf order, which is arrival order inside a group
      uint64_t p2 = 0;
      if ((st = big_groups(g, ik, iv, n, srt, g->ctrl_h->big, pk1 + p_new, pv1 + p_new, pt1 + p_new, seq + p_new,
                           p_new, &p2, s)))
        return st;
      p_new += p2;
      g->last.last_unique = g->ctrl_h->nunique;
      g->last.last_pending = (uint32_t)g->ctrl_h->sum;
    }
    dirty_base = g->ctrl_h->ndirty;
    g->last.last_slots_rewritten += g->ctrl_h->windows_rewritten * g->L;
    g->last.last_windows_rewritten += g->ctrl_h->windows_rewritten;
    g->last.last_level0_windows = g->ctrl_h->windows_rewritten;
    if (p_new && !g->ctrl_h->big) {                    // leaf order: sort inside each leaf only
      GP_LAUNCH(g, k_pend_segsort, grid_for(p_new), TB, 0, s, pk1, pv1, pt1, p_new, (uint64_t *)g->b_pk[0].p,
                (uint32_t *)g->b_pv[0].p, (uint32_t *)g->b_pt[0].p);
      g->last.last_top_level = 1;
    } else if (p_new) {                                  // (+ oversized groups' keys appended: full sort)
      int sh[8], which = 0;
      const int ns = key_shifts(g->V, sh);
      GP_CHECK(g, radix_sort_pairs(g, pk1, seq, (uint64_t *)g->b_sk[1].p, (uint32_t *)g->b_sv[1].p, p_new, sh, ns, s,
                                   &which));
      const uint64_t *pks = which ? (const uint64_t *)g->b_sk[1].p : pk1;
      const uint32_t *perm = which ? (const uint32_t *)g->b_sv[1].p : seq;
      GP_LAUNCH(g, k_pend_permute, grid_for(p_new), TB, 0, s, perm, p_new, pv1, pt1, (uint32_t *)g->b_pv[0].p,
                (uint32_t *)g->b_pt[0].p);
      GP_CHECK(g, stage_in(g, g->b_pk[0].p, pks, p_new * 8, s));
      g->last.last_top_level = 1;
    }
    p = p_new;
    lvl = 1;
  } else if (path == PATH_INS_FUSED) {
    // pending after level 0: the new keys the leaves rejected, still sorted, with their targets
    const uint64_t p_new = (uint32_t)g->ctrl_h->sum2;
    dirty_base = g->ctrl_h->ndirty;
    g->last.last_slots_rewritten += g->ctrl_h->windows_rewritten * g->L;
    g->last.last_windows_rewritten += g->ctrl_h->windows_rewritten;
    g->last.last_level0_windows = g->ctrl_h->windows_rewritten;
    if (p_new) {
      GP_LAUNCH(g, k_compact_pending, grid_for(n), TB, 0, s, (const uint32_t *)g->b_keep.p,
                (const uint32_t *)g->b_pos.p, n, srt.k, srt.v, (const uint32_t *)g->b_tgt.p, (uint64_t *)g->b_pk[0].p,
                (uint32_t *)g->b_pv[0].p, (uint32_t *)g->b_pt[0].p, g->ctrl_d);
      g->last.last_top_level = 1;
    }
    p = p_new;
    lvl = 1;
  } else if (fused) {
    const uint64_t p_new = (uint32_t)g->ctrl_h->sum2;
    dirty_base = g->ctrl_h->ndirty;
    g->last.last_slots_rewritten += g->ctrl_h->windows_rewritten * g->L;
    g->last.last_windows_rewritten += g->ctrl_h->windows_rewritten;
    g->last.last_level0_windows = g->ctrl_h->windows_rewritten;
    if (p_new) {
      GP_LAUNCH(g, k_compact_pending, grid_for(p), TB, 0, s, keep2, kpos, p, (const uint64_t *)g->b_pk[0].p,
                (const uint32_t *)g->b_pv[0].p, (const uint32_t *)g->b_pt[0].p, (uint64_t *)g->b_pk[1].p,
                (uint32_t *)g->b_pv[1].p, (uint32_t *)g->b_pt[1].p, g->ctrl_d);
      cur = 1;
      g->last.last_top_level = 1;
    }
    p = p_new;
    lvl = 1;
  }
  if (lvl == 1) g->last.last_pending_level1 = p;
  if (trace_levels())
    fprintf(stderr, "[gpma] prefix + level 0: %llu pending for level %u at %.3f ms\n", (unsigned long long)p, lvl,
            std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - tl_call_start).count());
  if (p > 0 && lvl >= 1 && lvl <= g->h && !g->trace_on && coop_eligible(g, p, lvl)) {
    Nvtx nv("update: device level loop");
    const uint64_t p0 = p;
    const uint32_t l0 = lvl;
    if ((st = coop_levels(g, cur, p, lvl, &dirty_base, op, s))) return st;
    if (trace_levels())
      fprintf(stderr, "[gpma] device level loop %u..%u  pending %llu -> %llu  at %.3f ms\n", l0, lvl - 1,
              (unsigned long long)p0, (unsigned long long)p,
              std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - tl_call_start).count());
  }
  Nvtx nvtx_levels("update: host level loop");
  const bool skip = lvl_skip_on() && !g->trace_on && g->cap < (1ull << 32) && g->h < 64;
  uint32_t next_check = 0;
  bool planned = false;
  uint64_t lvl_mask = 0;
  g->sup_on = false;
  if (skip && lvl_plan_on() && p >= SKIP_MINP && lvl < g->h) {
    bool root = false;
    if ((st = plan_levels(g, cur, p, lvl, op, &root, &lvl_mask, s))) return st;
    if (root) lvl_mask = 0;                              // the root rewrite supersedes every level
    planned = true;
    g->sup_on = true;
    if (trace_levels())
      fprintf(stderr, "[gpma] plan from level %u: levels %llx, root %d\n", lvl, (unsigned long long)lvl_mask, (int)root);
  }
  for (; lvl <= g->h && p > 0; ++lvl) {
    if (planned && lvl < g->h && !((lvl_mask >> lvl) & 1ull)) {   // no maximal accepted window here
      g->last.last_levels_skipped++;
      continue;
    }
    Lvl a = make_lvl(g, cur, p, lvl, op);
    LevelOut lo{};
    if ((st = level_step(g, a, cur, &lo, &dirty_base, s, false, 0, nullptr, nullptr, nullptr))) return st;
    g->last.last_slots_rewritten += lo.nacc * ((uint64_t)g->L << lvl);
    g->last.last_windows_rewritten += lo.nacc;
    g->last.last_top_level = lvl;
    if (lo.p_new) cur ^= 1;
    const uint64_t p_in = p;
    p = lo.p_new;
    if (trace_levels())                                   // (level_step ended on a stream sync)
      fprintf(stderr, "[gpma] level %2u  pending %9llu -> %9llu  accepted %8llu  at %.3f ms\n", lvl,
              (unsigned long long)p_in, (unsigned long long)p, (unsigned long long)lo.nacc,
              std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - tl_call_start).count());
    if (!planned && skip && p >= SKIP_MINP && 2 * p > p_in && lvl + 1 < g->h && lvl >= next_check) {
      // a level that absorbed less than half of many pending updates: likely a root-bound climb
      // -- jump over the levels where no window accepts (nothing happens there), or, when some
      // update reaches the root (absorbed less than a fifth: the root-reach walk), straight to
      // the root.  A check that finds the next level accepting backs off for two levels.
      uint32_t j = 0;
      bool root = false;
      const bool rj = root_jump_on() && 5 * (p_in - p) < p_in;
      if ((st = first_accept_level(g, cur, p, lvl + 1, g->h, op, &j, s, rj ? &root : nullptr))) return st;
      if (root) j = g->h;
      g->last.last_levels_skipped += j - (lvl + 1);
      if (j == lvl + 1) next_check = lvl + 3;
      lvl = j - 1;
    }
  }
  g->sup_on = false;
  if (p > 0) {
    g->last.last_top_level = g->h + 1;
    return resize(g, cur, p, op, s, &dirty_base);
  }
  if (dirty_base) {
    if ((st = fix_heads(g, dirty_base, s))) return st;
  }
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

}  // namespace gp
