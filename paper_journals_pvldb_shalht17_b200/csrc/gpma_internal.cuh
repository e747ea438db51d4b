// gpma_internal.cuh -- internal definitions of the sm_100a GPMA+ library.
// Paper: Sha et al., PVLDB 11(1) 2017 (PAPER.md, cited P:<line>); readings R<n> in DESIGN.md.
#pragma once

#include <cuda_runtime.h>
#include <stdint.h>

#include <atomic>
#include <mutex>
#include <string>
#include <array>
#include <vector>

#include <nvtx3/nvToolsExt.h>

#include "../../include/gpma.h"

namespace gp {

// NVTX range of a phase (nsys / ncu timelines: every C-ABI call and the phases of an update
// batch show up by name; header-only NVTX3, inert unless a tool is attached)
struct Nvtx {
  explicit Nvtx(const char *name) { nvtxRangePushA(name); }
  ~Nvtx() { nvtxRangePop(); }
};

constexpr uint64_t KEY_NONE = ~0ull;          // R2 empty slot
constexpr uint32_t VAL_TOMB = 0xFFFFFFFFu;    // R12 lazy-delete mark
constexpr uint32_t COL_GUARD = 0xFFFFFFFFu;   // R1 guard column ("infinity")
constexpr int MAX_RESIDENT_BLOCKS = 148 * 8;  // grid-stride kernels: 8 x 256-thread CTAs per SM
// Sweeps over the slot array (PR push, CC sample/hook, export): 8 waves of resident CTAs, so
// the skewed (RMAT) work per chunk balances out -- measured 10-20% faster than one wave.
constexpr int SWEEP_BLOCKS = 148 * 64;

// L (slots per leaf) is a power of two (R3; gpma_create / gpma_create_raw reject others):
// slot -> leaf and slot-in-leaf are a shift and a mask, not a 64-bit division by a runtime L
__host__ __device__ __forceinline__ uint64_t leaf_div(uint64_t s, uint32_t L) {
#ifdef __CUDA_ARCH__
  return s >> (__ffs(L) - 1);
#else
  return s >> __builtin_ctz(L);
#endif
}
__host__ __device__ __forceinline__ uint32_t leaf_mod(uint64_t s, uint32_t L) { return (uint32_t)s & (L - 1); }

__host__ __device__ inline bool is_guard_key(uint64_t k) {
  return k != KEY_NONE && (uint32_t)k == COL_GUARD;
}

struct DevBuf {
  void *p = nullptr;
  size_t bytes = 0;
};

// Device-side control block (counters written by kernels, read back in one copy).
struct Ctrl {
  uint32_t err;            // validation bits: 1 = range, 2 = reserved
  uint32_t seq;            // host mirror only: the call's sequence number, written last (wait_ctrl)
  uint64_t nunique;        // distinct keys in the batch
  uint64_t slots_rewritten;
  uint64_t windows_rewritten;
  uint64_t ndirty;         // dirty windows recorded for the head fix-up
  uint64_t sum;            // scratch reductions
  uint64_t sum2;
  uint64_t big;            // updates in leaf groups too large for the thread-per-group merge
  uint64_t done;           // CTAs finished (multi-CTA one-kernel calls; reset by the last one)
};

// Per-level descriptors of one GPMA+ round (Alg. 4 l.7-15).
struct LevelBufs {
  uint32_t *hf = nullptr;     // [p+1] window-head flags -> exclusive scan (widx)
  uint32_t *widx = nullptr;
  uint32_t *wfirst = nullptr; // [p+1] offsets I
  uint32_t *acc = nullptr;    // [p+1] success flags -> aidx
  uint32_t *aidx = nullptr;
  uint32_t *alist = nullptr;  // accepted window ids
  uint64_t *nw = nullptr;     // [p+1] entries after merge -> woff
  uint64_t *woff = nullptr;
  uint32_t *keep = nullptr;   // [p+1]
  uint32_t *kpos = nullptr;
};

// Per-analytic scratch + control block: BFS, CC, PageRank, export and the query buffer only
// read the store, so each owns its temporaries and they may run concurrently on different
// streams from different host threads (include/gpma.h, "Concurrency").
enum { AN_BFS = 0, AN_CC, AN_PR, AN_EXPORT, AN_QUERY, AN_N };
struct Scratch {
  DevBuf b[4], misc, lpre, scan, stage[2];
  Ctrl *ctrl_d = nullptr;
  Ctrl *ctrl_h = nullptr;         // pinned mirror
};

#ifdef __CUDACC__
// Ascending sort of the (key, index) pairs sk/si[0, np2) in shared memory by one CTA (np2 a power
// of two, 2 <= np2 <= 2 * blockDim.x; entries past the real ones hold padding keys): a bitonic
// network with thread t holding elements 2t and 2t+1 in registers.  Strides 1..32 stay in
// registers (in-thread, then warp shuffles -- no barrier), only strides >= 64 go through the
// shared arrays (two barriers each): 15 of the 55 stages of a 1024-pair sort instead of all 55.
// Ties on the key are broken by the index, so with distinct indices the order is total (stable
// when the indices are the arrival positions).  Every thread of the CTA must call it.
__device__ __forceinline__ bool cta_pair_less(uint64_t ka, uint32_t ia, uint64_t kb, uint32_t ib) {
  return ka < kb || (ka == kb && ia < ib);
}
__device__ __forceinline__ void cta_pair_cas(uint64_t &k, uint32_t &x, uint64_t pk, uint32_t px, uint32_t i,
                                             uint32_t j, uint32_t size) {
  const bool up = (i & size) == 0;
  const bool keep_min = (i < j) == up;
  const bool own_less = cta_pair_less(k, x, pk, px);
  if (keep_min != own_less) {
    k = pk;
    x = px;
  }
}
__device__ inline void cta_bitonic_sort(uint64_t *sk, uint32_t *si, uint32_t np2) {
  const uint32_t t = threadIdx.x;
  const bool act = 2 * t < np2;
  const bool wact = 64 * (t >> 5) < np2;                 // warp-uniform: the warp holds elements
  uint64_t k0 = ~0ull, k1 = ~0ull;
  uint32_t x0 = ~0u, x1 = ~0u;
  if (act) {
    k0 = sk[2 * t];
    x0 = si[2 * t];
    k1 = sk[2 * t + 1];
    x1 = si[2 * t + 1];
  }
  for (uint32_t size = 2; size <= np2; size <<= 1)
    for (uint32_t stride = size >> 1; stride; stride >>= 1) {
      if (stride < 64 && !wact) continue;               // (no barrier below 64)
      if (stride == 1) {                                 // elements 2t, 2t+1 of this thread
        const bool up = ((2 * t) & size) == 0;
        if (cta_pair_less(k1, x1, k0, x0) == up) {
          const uint64_t tk = k0;
          k0 = k1;
          k1 = tk;
          const uint32_t tx = x0;
          x0 = x1;
          x1 = tx;
        }
      } else if (stride < 64) {                          // partner thread t ^ stride/2, same warp
        const int m = (int)(stride >> 1);
        const uint64_t p0 = __shfl_xor_sync(0xffffffffu, k0, m), p1 = __shfl_xor_sync(0xffffffffu, k1, m);
        const uint32_t q0 = __shfl_xor_sync(0xffffffffu, x0, m), q1 = __shfl_xor_sync(0xffffffffu, x1, m);
        cta_pair_cas(k0, x0, p0, q0, 2 * t, (2 * t) ^ stride, size);
        cta_pair_cas(k1, x1, p1, q1, 2 * t + 1, (2 * t + 1) ^ stride, size);
      } else {                                           // through shared memory
        __syncthreads();
        if (act) {
          sk[2 * t] = k0;
          si[2 * t] = x0;
          sk[2 * t + 1] = k1;
          si[2 * t + 1] = x1;
        }
        __syncthreads();
        if (act) {
          const uint32_t j0 = (2 * t) ^ stride, j1 = (2 * t + 1) ^ stride;
          const uint64_t p0 = sk[j0], p1 = sk[j1];
          const uint32_t q0 = si[j0], q1 = si[j1];
          cta_pair_cas(k0, x0, p0, q0, 2 * t, j0, size);
          cta_pair_cas(k1, x1, p1, q1, 2 * t + 1, j1, size);
        }
      }
    }
  __syncthreads();
  if (act) {
    sk[2 * t] = k0;
    si[2 * t] = x0;
    sk[2 * t + 1] = k1;
    si[2 * t + 1] = x1;
  }
  __syncthreads();
}

// The same network over distinct u64 keys only (sk[0, np2)): one compare and one 64-bit shuffle
// per element and stage -- for keys that carry their own tie-break (a packed arrival index).
__device__ inline void cta_bitonic_sort_u64(uint64_t *sk, uint32_t np2) {
  const uint32_t t = threadIdx.x;
  const bool act = 2 * t < np2;
  const bool wact = 64 * (t >> 5) < np2;
  uint64_t k0 = ~0ull, k1 = ~0ull;
  if (act) {
    k0 = sk[2 * t];
    k1 = sk[2 * t + 1];
  }
  for (uint32_t size = 2; size <= np2; size <<= 1)
    for (uint32_t stride = size >> 1; stride; stride >>= 1) {
      if (stride < 64 && !wact) continue;
      if (stride == 1) {
        const bool up = ((2 * t) & size) == 0;
        if ((k1 < k0) == up) {
          const uint64_t tk = k0;
          k0 = k1;
          k1 = tk;
        }
      } else if (stride < 64) {
        const int m = (int)(stride >> 1);
        const uint64_t p0 = __shfl_xor_sync(0xffffffffu, k0, m), p1 = __shfl_xor_sync(0xffffffffu, k1, m);
        const bool up = ((2 * t) & size) == 0;           // same for 2t and 2t+1 (size >= 4 here)
        const bool lo = ((2 * t) & stride) == 0;         // this thread holds the lower index of the pair
        const bool keep_min = lo == up;
        k0 = keep_min ? min(k0, p0) : max(k0, p0);
        k1 = keep_min ? min(k1, p1) : max(k1, p1);
      } else {
        __syncthreads();
        if (act) {
          sk[2 * t] = k0;
          sk[2 * t + 1] = k1;
        }
        __syncthreads();
        if (act) {
          const uint64_t p0 = sk[(2 * t) ^ stride], p1 = sk[(2 * t + 1) ^ stride];
          const bool up = ((2 * t) & size) == 0;
          const bool keep_min = (((2 * t) & stride) == 0) == up;
          k0 = keep_min ? min(k0, p0) : max(k0, p0);
          k1 = keep_min ? min(k1, p1) : max(k1, p1);
        }
      }
    }
  __syncthreads();
  if (act) {
    sk[2 * t] = k0;
    sk[2 * t + 1] = k1;
  }
  __syncthreads();
}

// Merge sort of distinct-or-padded u64 keys sk[0, np2) (np2 a power of two, 64 <= np2 <= 2 *
// blockDim.x, blockDim.x a multiple of 32): every warp sorts its 64 keys in registers with the
// shuffle network (no barrier), then log2(np2 / 64) rounds merge run pairs in shared memory --
// an element's new place is its offset in its run plus its rank in the partner run (lower bound
// from the left run, upper bound from the right: a stable merge, a permutation even for equal
// padding keys).  ~1/6 of the bitonic network's time at 1024 keys: the 15 bitonic stages with
// strides >= 64 (two barriers each) become 4 merge rounds.
__device__ inline void cta_merge_sort_u64(uint64_t *sk, uint32_t np2) {
  const uint32_t t = threadIdx.x;
  const bool act = 2 * t < np2;
  if (64 * (t >> 5) < np2) {                             // warps holding keys: sort 64 in registers
    const uint32_t li = 2 * (t & 31);                    // index inside the warp's 64 (all ascending)
    uint64_t k0 = act ? sk[2 * t] : ~0ull, k1 = act ? sk[2 * t + 1] : ~0ull;
#pragma unroll
    for (int ls = 1; ls <= 6; ++ls) {
      const uint32_t size = 1u << ls;
      const bool up = (li & size) == 0;                  // (size 64: every warp ascending)
#pragma unroll
      for (int lt = ls - 1; lt >= 0; --lt) {
        const uint32_t stride = 1u << lt;
        if (stride == 1) {
          if ((k1 < k0) == up) {
            const uint64_t tk = k0;
            k0 = k1;
            k1 = tk;
          }
        } else {
          const int m = (int)(stride >> 1);
          const uint64_t p0 = __shfl_xor_sync(0xffffffffu, k0, m), p1 = __shfl_xor_sync(0xffffffffu, k1, m);
          const bool keep_min = ((li & stride) == 0) == up;
          k0 = keep_min ? min(k0, p0) : max(k0, p0);
          k1 = keep_min ? min(k1, p1) : max(k1, p1);
        }
      }
    }
    if (act) {
      sk[2 * t] = k0;
      sk[2 * t + 1] = k1;
    }
  }
  __syncthreads();
  for (uint32_t run = 64; run < np2; run <<= 1) {
    // both elements' ranks by branch-free binary lifting, interleaved (independent LDS chains)
    uint64_t x[2];
    uint32_t pb[2], lo[2] = {0u, 0u};
    bool left[2];
    if (act) {
#pragma unroll
      for (int e = 0; e < 2; ++e) {
        const uint32_t i = 2 * t + e, r = i / run;
        x[e] = sk[i];
        pb[e] = (r ^ 1u) * run;
        left[e] = (r & 1u) == 0;
      }
      for (uint32_t st = run >> 1; st; st >>= 1) {
#pragma unroll
        for (int e = 0; e < 2; ++e) {
          const uint64_t y = sk[pb[e] + lo[e] + st - 1];
          if (left[e] ? (y < x[e]) : (y <= x[e])) lo[e] += st;
        }
      }
#pragma unroll
      for (int e = 0; e < 2; ++e) {
        const uint64_t y = sk[pb[e] + lo[e]];
        if (left[e] ? (y < x[e]) : (y <= x[e])) lo[e] += 1;
      }
    }
    __syncthreads();
    if (act) {
#pragma unroll
      for (int e = 0; e < 2; ++e) {
        const uint32_t i = 2 * t + e, r = i / run;
        sk[(r & ~1u) * run + (i - r * run) + lo[e]] = x[e];
      }
    }
    __syncthreads();
  }
}
#endif

// Replayable prefix of one update batch (everything up to its single host read-back) as a
// CUDA graph: small batches are bound by host launch overhead (~12 launches per insert), a
// graph replays them with one launch.  Valid while the signature -- batch shape plus every
// pointer / scalar the prefix bakes into its kernels -- is unchanged.
struct UpdGraph {
  std::vector<uint64_t> sig;      // signature of the captured graph
  std::vector<uint64_t> seen;     // signature after the last un-captured run of this op
  cudaGraphExec_t exec = nullptr;
  uint64_t nlaunch = 0;           // kernels in the graph (launch accounting)
  void *srt[4] = {nullptr, nullptr, nullptr, nullptr};   // sorted batch buffers of the captured shape
};

}  // namespace gp

struct gpma {
  // geometry (R3, R4, R5, R15)
  uint32_t V = 0, L = 0, h = 0, mode = 0;
  uint32_t rb = 0, nr = 0;        // owned rows [rb, rb + nr) (shard, R24); nr = V unsharded
  uint32_t algorithm = 0;         // 0 = GPMA+ (Alg. 4), 1 = GPMA lock-based (Alg. 1)
  bool rows_indexed = false;      // every owned row has its guard: row_offset locates leaves
  gp::UpdGraph ugraph[2];         // per op (insert, delete)
  bool graphs_off = false;        // a capture failed once: plain launches from then on
  uint64_t cap = 0;
  uint32_t rho0 = 800, rhoh = 4000, tau0 = 9200, tauh = 8000, init_bp = 6000;
  std::vector<uint64_t> tmin, tmax;

  struct SpareStore {              // the previous capacity's arrays, kept across a resize
    uint64_t cap = 0;
    uint64_t *key = nullptr;
    uint32_t *val = nullptr;
    uint32_t *cnt = nullptr;
    uint64_t *head = nullptr;
  } spare;

  // store (HBM-resident)
  uint64_t *key = nullptr;        // [cap]
  uint32_t *val = nullptr;        // [cap]
  bool root_heads_done = false;   // the last root re-layout wrote the locate heads
  gp::DevBuf b_sup;                // truly accepted windows of the planned climb (heap-indexed bits)
  bool sup_on = false;             // the host levels of this batch follow a plan (b_sup valid)
  std::vector<std::array<uint64_t, 3>> big_dirty;   // (first dirty entry, windows, leaves each) of big rewritten windows
  uint32_t *cnt = nullptr;        // [3*cap/L]: live entries (incl. guards) per leaf, then the
                                  // per-leaf tombstone bit mask (bit p = slot p is a tombstone),
                                  // then the guards per leaf
  uint32_t *deg = nullptr;        // [V] live out-degree per vertex, maintained by every batch
  uint64_t *head = nullptr;       // [cap/L] locate index (R9)
  uint64_t *row_offset = nullptr; // [V+1] (R8)

  // scratch arena
  gp::DevBuf b_sk[2], b_sv[2], b_keep, b_pos, b_tgt;       // batch
  gp::DevBuf b_pk[2], b_pv[2], b_pt[2];                      // pending (ping-pong)
  gp::DevBuf b_hf, b_widx, b_wfirst, b_acc, b_aidx, b_alist, b_nw, b_woff, b_keep2, b_kpos;
  gp::DevBuf b_lpre, b_wk, b_wv, b_dirty, b_scan, b_hist, b_stage[4], b_misc, b_misc2, b_misc3;
  gp::Ctrl *ctrl_d = nullptr;
  gp::Ctrl *ctrl_h = nullptr;     // pinned mirror
  uint32_t ctrl_seq = 0;          // sequence number of the last mirrored one-kernel call
  uint64_t root_need = 0;         // entries of a root re-layout (live + pending): its scratch size
  void *pin = nullptr;            // 256 B of pinned host scratch (read-backs of small device state)
  gp::Scratch an[gp::AN_N];       // analytics (read-only on the store)

  // device memory (gpma_config.alloc / free / alloc_ctx; NULL = the library's pool)
  void *(*alloc_fn)(size_t, gpma_stream_t, void *) = nullptr;
  void (*free_fn)(void *, gpma_stream_t, void *) = nullptr;
  void *alloc_ctx = nullptr;
  int device = 0;
  bool pool_attached = false;

  // multi-GPU (gpma_dist_create, dist_nccl.cu): the rank's NCCL communicator and its scratch
  void *comm = nullptr;           // ncclComm_t; null = a single store (or a shard driven from outside)
  int rank = 0, nranks = 1;
  gp::DevBuf d_k[2], d_v[2], d_misc;

  // state
  bool poisoned = false;
  std::string err;
  std::mutex mu;                  // guards err and the profiler across analytic threads
  std::atomic<uint64_t> launches{0};
  uint64_t resizes = 0;
  gpma_stats_t last{};
  uint64_t tot[5] = {0, 0, 0, 0, 0};   // batches, insert keys, delete keys, slots, windows rewritten
  bool trace_on = false;
  std::vector<uint64_t> trace;    // (level, start, offset, flag) x4
  cudaStream_t st = nullptr;

  // kernel-level CUDA-event profiler (bench evidence; off by default)
  std::string prof_filter;        // "" = off, "*" = every kernel, else exact kernel name
  std::vector<cudaEvent_t> ev_pool;
  size_t ev_used = 0;
  struct ProfRec { const char *name; size_t e0, e1; };
  std::vector<ProfRec> prof_recs;
};

// ---------------------------------------------------------------- helpers (host)
namespace gp {

long prof_begin(gpma *g, const char *name, cudaStream_t s);   // record index, -1 = not profiled
void prof_end(gpma *g, long rec, cudaStream_t s);
void set_err(gpma *g, const std::string &msg);

// scans issued by an analytic use that analytic's look-back status buffer
extern thread_local DevBuf *tl_scan;
struct ScanScope {
  DevBuf *prev;
  explicit ScanScope(DevBuf &b) : prev(tl_scan) { tl_scan = &b; }
  ~ScanScope() { tl_scan = prev; }
};

#define GP_LAUNCH(g, kernel, grid, block, smem, stream, ...)                 \
  do {                                                                       \
    long prof_ = (g)->prof_filter.empty() ? -1 : gp::prof_begin((g), #kernel, (stream)); \
    kernel<<<(grid), (block), (smem), (stream)>>>(__VA_ARGS__);              \
    (g)->launches++;                                                         \
    if (prof_ >= 0) gp::prof_end((g), prof_, (stream));                      \
  } while (0)

// grid cap of the grid-stride kernels (default MAX_RESIDENT_BLOCKS; GPMA_GRID_CAP overrides)
int grid_cap();
// copy `bytes` (multiple of 4, 4-B aligned) from device memory to PINNED host memory with a
// kernel (no copy engine); stream-ordered like cudaMemcpyAsync
cudaError_t readback(gpma *g, void *host_pinned, const void *dev, size_t bytes, cudaStream_t s);
// copy a caller's input (host or device pointer) into library scratch, stream-ordered
cudaError_t stage_in(gpma *g, void *dst, const void *src, size_t bytes, cudaStream_t s);
// zero `bytes` (multiple of 4, 4-B aligned) of device memory with a kernel, stream-ordered
cudaError_t fill_zero(gpma *g, void *dst, size_t bytes, cudaStream_t s);
// SMs of the current device (persistent sweeps launch one CTA per SM)
int num_sms();

inline unsigned grid_for(uint64_t n, int block = 256, int max_blocks = 0) {
  if (max_blocks <= 0) max_blocks = grid_cap();
  uint64_t b = (n + block - 1) / block;
  if (b < 1) b = 1;
  if (b > (uint64_t)max_blocks) b = max_blocks;
  return (unsigned)b;
}

// device memory of the library: the caller's hooks (gpma_config.alloc/free) or the
// library-owned stream-ordered pool of the device
cudaError_t dev_alloc(gpma *g, void **p, size_t bytes, cudaStream_t s);
void dev_free(gpma *g, void *p, cudaStream_t s);
void pool_attach(gpma *g);     // at create: pick the device's pool (counted per device)
void pool_detach(gpma *g);     // at destroy: the last handle of a device trims its pool
// allocate (stream-ordered) at least `bytes`, keeping the old block when large enough
cudaError_t ensure(gpma *g, DevBuf &b, size_t bytes, cudaStream_t s);
void release(gpma *g, DevBuf &b, cudaStream_t s);

// exclusive scan: out[0..n) = prefix sums of in[0..n), out[n] = total.  in == out allowed.
[[nodiscard]] cudaError_t scan_u32(gpma *g, const uint32_t *in, uint32_t *out, uint64_t n, cudaStream_t s);
[[nodiscard]] cudaError_t scan_u64(gpma *g, const uint64_t *in, uint64_t *out, uint64_t n, cudaStream_t s);
// exclusive scan of (cnt[l] - gl[l]) over l < nl into out[0..nl] (the export's leaf offsets)
[[nodiscard]] cudaError_t scan_leaf_edges(gpma *g, const uint32_t *cnt, const uint32_t *gl, uint64_t *out, uint64_t nl,
                                          cudaStream_t s);
// stable onesweep LSD radix sort of (key, val) pairs (vals may be null: keys only) on the
// given 8-bit digit shifts; *which = the index (0/1) of the buffer pair holding the result.
[[nodiscard]] cudaError_t radix_sort_pairs(gpma *g, uint64_t *k0, uint32_t *v0, uint64_t *k1, uint32_t *v1,
                                           uint64_t n, const int *shifts, int nshift, cudaStream_t s, int *which);
gpma_status radix_partition_owner(gpma *g, const uint64_t *k0, const uint32_t *v0, uint64_t *k1, uint32_t *v1,
                                  uint64_t n, uint32_t div, uint32_t nranks, uint64_t *starts_dev,
                                  cudaStream_t s);
// query buffer (query.cu)
gpma_status query_edges(gpma *g, const uint64_t *keys, uint64_t n, uint32_t *vals, uint8_t *found, cudaStream_t s);
gpma_status query_neighbors(gpma *g, const uint32_t *verts, uint64_t n, uint64_t *row_ptr, uint32_t *col,
                            uint32_t *val, uint64_t cap_nnz, uint64_t *nnz_out, cudaStream_t s);
gpma_status query_reachable(gpma *g, const uint32_t *src, const uint32_t *dst, uint64_t n, uint8_t *out,
                            cudaStream_t s);
// distributed primitives (dist.cu / analytics.cu)
gpma_status route(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, uint32_t nranks,
                  uint64_t *out_keys, uint32_t *out_vals, uint64_t *counts_host, cudaStream_t s);
gpma_status bfs_init(gpma *g, uint32_t root, int32_t *levels, cudaStream_t s);
gpma_status bfs_level(gpma *g, int32_t *levels, int32_t depth, uint32_t *frontier, cudaStream_t s);
gpma_status cc_round(gpma *g, uint32_t *labels, int init, uint64_t *changed, cudaStream_t s);
gpma_status pr_push(gpma *g, double *x, int init, uint64_t *y, cudaStream_t s);
gpma_status pr_update(gpma *g, double *x, uint64_t *y, double d, double *err, cudaStream_t s);
gpma_status pr_update_rows(gpma *g, double *x, const uint64_t *y_rows, double d, double *err, cudaStream_t s);
gpma_status pr_update_rows_dev(gpma *g, double *x, const uint64_t *y_rows, double d, double *err_dev,
                              cudaStream_t s);
gpma_status bfs_bits(gpma *g, const int32_t *levels, int32_t depth, uint32_t *bm, cudaStream_t s);
gpma_status bfs_merge(gpma *g, int32_t *levels, const uint32_t *bms, uint32_t nbm, int32_t depth, cudaStream_t s);
// digit shifts covering the significant bits of keys with src, dst < V
int key_shifts(uint32_t V, int *shifts);

// multi-GPU handle (dist_nccl.cu): NCCL communicator + the collective update / analytics
void dist_rows(uint32_t V, int P, int r, uint32_t *rb, uint32_t *re);
gpma_status dist_unique_id(void *out);
gpma_status dist_attach(gpma *g, const void *id, int rank, int nranks);
void dist_detach(gpma *g);
gpma_status dist_create_store(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, uint64_t cap,
                              uint32_t leaf, cudaStream_t s);
gpma_status dist_update(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, int op, cudaStream_t s);
gpma_status dist_bfs(gpma *g, uint32_t root, int32_t *levels, cudaStream_t s);
gpma_status dist_cc(gpma *g, uint32_t *labels, cudaStream_t s);
gpma_status dist_pagerank(gpma *g, double *x, int warm, double d, double tol, int max_iter, int *iters,
                          cudaStream_t s);

// thresholds (R4/R5) -- the library's own implementation (independent of oracle/)
void level_bounds(uint32_t L, uint32_t h, uint32_t rho0, uint32_t rhoh, uint32_t tau0,
                  uint32_t tauh, std::vector<uint64_t> &mn, std::vector<uint64_t> &mx);
uint32_t leaf_rule(uint64_t cap0);
inline uint32_t ilog2(uint64_t x) { uint32_t r = 0; while (x > 1) { x >>= 1; ++r; } return r; }

gpma_status cuda_fail(gpma *g, cudaError_t e, const char *where);

// update engine (update.cu)
gpma_status update_batch(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, int op,
                         cudaStream_t s);
gpma_status validate_slice(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, bool check_vals,
                           cudaStream_t s);
gpma_status create_from_batch(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n,
                              uint64_t cap_override, uint32_t leaf_override, cudaStream_t s);
gpma_status build_from_sorted(gpma *g, const uint64_t *sk, const uint32_t *sv, uint64_t m,
                              cudaStream_t s);
gpma_status load_raw(gpma *g, const uint64_t *keys, const uint32_t *vals, cudaStream_t s);
gpma_status recompute_heads(gpma *g, cudaStream_t s);
void spare_release(gpma *g, cudaStream_t s);
gpma_status count_slots(gpma *g, uint64_t *live_edges, uint64_t *tombs, cudaStream_t s);
gpma_status recompute_degrees(gpma *g, cudaStream_t s);   // analytics.cu
inline uint32_t *tmask_of(gpma *g) { return g->cnt + g->cap / g->L; }
inline uint32_t *gcnt_of(gpma *g) { return g->cnt + 2 * (g->cap / g->L); }

// analytics (analytics.cu)
gpma_status bfs(gpma *g, uint32_t root, int32_t *levels, cudaStream_t s);
gpma_status cc(gpma *g, uint32_t *labels, cudaStream_t s);
gpma_status pagerank_f64(gpma *g, double *x, int warm, double d, double tol, int max_iter, int *iters,
                         cudaStream_t s);
gpma_status pagerank_f32(gpma *g, float *x, int warm, float d, float tol, int max_iter, int *iters,
                         cudaStream_t s);
gpma_status export_csr(gpma *g, uint64_t *row_ptr, uint32_t *col, uint32_t *val, uint64_t cap_nnz,
                       uint64_t *nnz_out, cudaStream_t s);

}  // namespace gp

#define GP_CHECK(g, call)                                   \
  do {                                                      \
    cudaError_t e_ = (call);                                \
    if (e_ != cudaSuccess) return gp::cuda_fail((g), e_, #call); \
  } while (0)
