// primitives.cu -- scans, stable LSD radix sort, thresholds, memory helpers (sm_100a).
//
// Alg. 4 builds GPMA+ from standard GPU primitives (RunLengthEncoding,
// ExclusiveScan; radix sort of the integer keys).  These are this
// library's own implementations -- no CUB / Thrust.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstring>

#include "gpma_internal.cuh"

namespace gp {

// ------------------------------------------------------------------ memory
cudaError_t ensure(DevBuf &b, size_t bytes, cudaStream_t s) {
  if (bytes == 0) bytes = 16;
  if (b.bytes >= bytes) return cudaSuccess;
  const size_t want = std::max(bytes, b.bytes + b.bytes / 2);  // grow x1.5 at least
  if (b.p) cudaFreeAsync(b.p, s);
  b.p = nullptr;
  b.bytes = 0;
  cudaError_t e = cudaMallocAsync(&b.p, want, s);
  if (e != cudaSuccess) {
    b.p = nullptr;
    return e;
  }
  b.bytes = want;
  return cudaSuccess;
}

void release(DevBuf &b, cudaStream_t s) {
  if (b.p) cudaFreeAsync(b.p, s);
  b.p = nullptr;
  b.bytes = 0;
}

// ------------------------------------------------------------------ kernel profiler
static size_t take_event(gpma *g) {
  if (g->ev_used == g->ev_pool.size()) {
    cudaEvent_t e;
    cudaEventCreate(&e);
    g->ev_pool.push_back(e);
  }
  return g->ev_used++;
}

long prof_begin(gpma *g, const char *name, cudaStream_t s) {
  while (*name == '(') ++name;            // GP_LAUNCH((k<T, U>), ...) stringises the parentheses
  if (g->prof_filter != "*") {
    // exact match on the kernel name without template arguments
    const char *lt = strchr(name, '<');
    size_t n = lt ? (size_t)(lt - name) : strlen(name);
    // (a comma-separated filter matches any of its names)
    bool hit = false;
    for (size_t a = 0; a <= g->prof_filter.size() && !hit;) {
      size_t b = g->prof_filter.find(',', a);
      if (b == std::string::npos) b = g->prof_filter.size();
      hit = (b - a == n) && strncmp(g->prof_filter.c_str() + a, name, n) == 0;
      a = b + 1;
    }
    if (!hit) return -1;
  }
  std::lock_guard<std::mutex> lk(g->mu);
  size_t e0 = take_event(g), e1 = take_event(g);
  cudaEventRecord(g->ev_pool[e0], s);
  g->prof_recs.push_back({name, e0, e1});
  return (long)g->prof_recs.size() - 1;
}

void prof_end(gpma *g, long rec, cudaStream_t s) {
  std::lock_guard<std::mutex> lk(g->mu);
  cudaEventRecord(g->ev_pool[g->prof_recs[rec].e1], s);
}

thread_local DevBuf *tl_scan = nullptr;

int grid_cap() {
  static const int v = [] {
    const char *e = getenv("GPMA_GRID_CAP");
    int c = e ? atoi(e) : 0;
    return c > 0 ? c : MAX_RESIDENT_BLOCKS;
  }();
  return v;
}

// Small device -> pinned-host read-backs by a one-warp kernel (zero-copy stores over the bus)
// instead of cudaMemcpyAsync: a DMA read-back queues on the D2H copy engine behind whatever a
// user's copy stream is moving (e.g. the Fig. 2 pipeline's result transfers), which would
// stall every host round trip of the library for the length of that transfer.
__global__ void k_readback(uint32_t *dst, const uint32_t *__restrict__ src, uint32_t nwords) {
  for (uint32_t i = threadIdx.x; i < nwords; i += blockDim.x) dst[i] = src[i];
}

cudaError_t readback(gpma *g, void *host_pinned, const void *dev, size_t bytes, cudaStream_t s) {
  g->launches++;
  k_readback<<<1, 32, 0, s>>>((uint32_t *)host_pinned, (const uint32_t *)dev, (uint32_t)(bytes / 4));
  return cudaGetLastError();
}

// Staging copy of a caller's batch into library scratch: a kernel when the source is device
// memory (same reason as readback: a D2D cudaMemcpyAsync may wait on a busy copy engine), a
// DMA copy when it is host memory.  bytes % 4 == 0, 4-B aligned.
__global__ void k_copy_words(uint32_t *__restrict__ dst, const uint32_t *__restrict__ src, uint64_t nwords,
                             int vec4) {
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  uint64_t i0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
  uint64_t head = 0;
  if (vec4) {
    const uint64_t n4 = nwords / 4;
    for (uint64_t i = i0; i < n4; i += stride)
      reinterpret_cast<uint4 *>(dst)[i] = __ldcs(reinterpret_cast<const uint4 *>(src) + i);
    head = n4 * 4;
  }
  for (uint64_t i = head + i0; i < nwords; i += stride) dst[i] = src[i];
}

cudaError_t stage_in(gpma *g, void *dst, const void *src, size_t bytes, cudaStream_t s) {
  if (!bytes) return cudaSuccess;
  cudaPointerAttributes a{};
  cudaError_t e = cudaPointerGetAttributes(&a, src);
  if (e != cudaSuccess) {
    cudaGetLastError();   // unregistered host pointer on older runtimes: treat as host
    a.type = cudaMemoryTypeUnregistered;
  }
  if (a.type == cudaMemoryTypeDevice || a.type == cudaMemoryTypeManaged) {
    const int vec4 = ((((uintptr_t)dst) | ((uintptr_t)src)) & 15) == 0;
    const uint64_t words = bytes / 4;
    g->launches++;
    k_copy_words<<<grid_for(vec4 ? words / 4 + 1 : words), 256, 0, s>>>((uint32_t *)dst, (const uint32_t *)src,
                                                                         words, vec4);
    return cudaGetLastError();
  }
  return cudaMemcpyAsync(dst, src, bytes, cudaMemcpyDefault, s);
}

// Zero fill by a kernel: cudaMemsetAsync may run on a copy engine and then waits behind a
// user's large D2H (measured: BFS 1.7 -> 15.7 ms under a concurrent 256 MB D2H).
__global__ void k_zero_words(uint32_t *__restrict__ dst, uint64_t nwords, int vec4) {
  const uint64_t stride = (uint64_t)gridDim.x * blockDim.x;
  const uint64_t i0 = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x;
  uint64_t head = 0;
  if (vec4) {
    const uint64_t n4 = nwords / 4;
    for (uint64_t i = i0; i < n4; i += stride) reinterpret_cast<uint4 *>(dst)[i] = make_uint4(0, 0, 0, 0);
    head = n4 * 4;
  }
  for (uint64_t i = head + i0; i < nwords; i += stride) dst[i] = 0u;
}

cudaError_t fill_zero(gpma *g, void *dst, size_t bytes, cudaStream_t s) {
  if (!bytes) return cudaSuccess;
  const uint64_t words = bytes / 4;
  const int vec4 = (((uintptr_t)dst) & 15) == 0;
  g->launches++;
  k_zero_words<<<grid_for(vec4 ? words / 4 + 1 : words), 256, 0, s>>>((uint32_t *)dst, words, vec4);
  return cudaGetLastError();
}

int num_sms() {
  static const int v = [] {
    int d = 0, n = 0;
    cudaGetDevice(&d);
    cudaDeviceGetAttribute(&n, cudaDevAttrMultiProcessorCount, d);
    return n > 0 ? n : 148;
  }();
  return v;
}

void set_err(gpma *g, const std::string &msg) {
  std::lock_guard<std::mutex> lk(g->mu);
  g->err = msg;
}

gpma_status cuda_fail(gpma *g, cudaError_t e, const char *where) {
  if (e == cudaErrorMemoryAllocation) {
    cudaGetLastError();
    set_err(g, std::string("out of device memory in ") + where);
    return GPMA_ERR_OOM;
  }
  g->poisoned = true;
  set_err(g, std::string(cudaGetErrorString(e)) + " in " + where);
  return GPMA_ERR_CUDA;
}

// ------------------------------------------------------------------ thresholds
// R4: rho_i / tau_i linear in the level between the Fig. 3 leaf and root values
// (P:417-422); R5: integer entry bounds capped at twice the child's bound.
void level_bounds(uint32_t L, uint32_t h, uint32_t rho0, uint32_t rhoh, uint32_t tau0,
                  uint32_t tauh, std::vector<uint64_t> &mn, std::vector<uint64_t> &mx) {
  mn.assign(h + 1, 0);
  mx.assign(h + 1, 0);
  const uint64_t H = h ? h : 1;
  for (uint32_t i = 0; i <= h; ++i) {
    const uint64_t slots = (uint64_t)L << i;
    const uint64_t wr = h ? (uint64_t)rho0 * (h - i) + (uint64_t)rhoh * i : rho0;
    const uint64_t wt = h ? (uint64_t)tau0 * (h - i) + (uint64_t)tauh * i : tau0;
    const uint64_t q = 10000ull * H;
    uint64_t lo = (wr * slots) / q + ((wr * slots) % q != 0);  // ceil
    uint64_t hi = (wt * slots) / q;                              // floor
    if (i) {
      lo = std::min(lo, 2 * mn[i - 1]);
      hi = std::min(hi, 2 * mx[i - 1]);
    }
    mn[i] = lo;
    mx[i] = hi;
  }
}

// R3: leaf segment of O(log N) slots, a power of two: max(4, 2^floor(log2(log2 cap0))).
uint32_t leaf_rule(uint64_t cap0) {
  uint32_t lg = ilog2(cap0);
  uint32_t L = 1u << ilog2(lg);
  return L < 4 ? 4 : L;
}

int key_shifts(uint32_t V, int *shifts) {
  uint32_t bits = V <= 1 ? 1 : ilog2((uint64_t)V - 1) + 1;
  int n = 0;
  for (uint32_t s = 0; s < bits; s += 8) shifts[n++] = (int)s;
  for (uint32_t s = 0; s < bits; s += 8) shifts[n++] = (int)(32 + s);
  return n;
}

// ------------------------------------------------------------------ scans
constexpr int SC_THREADS = 256;
constexpr int SC_ITEMS = 16;
constexpr int SC_TILE = SC_THREADS * SC_ITEMS;   // 4096

template <typename T>
__device__ __forceinline__ T warp_sum(T x) {
#pragma unroll
  for (int o = 16; o; o >>= 1) x += __shfl_xor_sync(0xffffffffu, x, o);
  return x;
}

template <typename T>
__device__ __forceinline__ T warp_incl_scan(T x, int lane) {
#pragma unroll
  for (int o = 1; o < 32; o <<= 1) {
    T y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  return x;
}

// Single-pass scan with decoupled look-back: each CTA takes the next tile id from a
// counter, publishes its aggregate, then walks back over its predecessors' published
// (aggregate | inclusive) values until it meets an inclusive prefix.  Status word:
// flag in bits 62-63 (0 = not ready, 1 = aggregate, 2 = inclusive), value below.
template <typename T>
__global__ void __launch_bounds__(SC_THREADS) k_scan_lookback(const T *in, T *out, uint64_t n,
                                                               unsigned long long *status) {
  __shared__ uint32_t s_tile;
  __shared__ T ws[SC_THREADS / 32];
  __shared__ T s_prefix;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  if (threadIdx.x == 0) s_tile = status ? (uint32_t)atomicAdd(status, 1ull) : 0u;  // status[0] = tile counter
  __syncthreads();
  const uint32_t tile = s_tile;
  volatile unsigned long long *st = status ? status + 1 : nullptr;   // null: single tile
  const uint64_t base = (uint64_t)tile * SC_TILE + (uint64_t)w * (32 * SC_ITEMS);
  T x[SC_ITEMS];
  T part = 0;
#pragma unroll
  for (int j = 0; j < SC_ITEMS; ++j) {
    uint64_t i = base + j * 32 + lane;
    x[j] = i < n ? in[i] : T(0);
    part += x[j];
  }
  T wtot = warp_sum(part);
  if (lane == 0) ws[w] = wtot;
  __syncthreads();
  if (w == 0) {
    T agg = 0;
    for (int k = 0; k < SC_THREADS / 32; ++k) agg += ws[k];
    const unsigned long long VMASK = (1ull << 62) - 1;
    T prefix = 0;
    if (lane == 0 && st) {
      __threadfence();
      st[tile] = ((tile == 0 ? 2ull : 1ull) << 62) | ((unsigned long long)agg & VMASK);
    }
    // warp-parallel look-back over windows of 32 predecessors
    int64_t t = (int64_t)tile - 1;
    while (t >= 0) {
      int64_t mine = t - lane;
      unsigned long long v = 2ull << 62;        // lanes past tile 0 act as an inclusive zero
      if (mine >= 0) {
        do { v = st[mine]; } while ((v >> 62) == 0);
      }
      uint32_t inc = __ballot_sync(0xffffffffu, (v >> 62) == 2);
      int stop = inc ? __ffs(inc) - 1 : 31;     // nearest predecessor with an inclusive prefix
      T contrib = (lane <= stop) ? (T)(v & VMASK) : T(0);
      prefix += warp_sum(contrib);
      if (inc) break;
      t -= 32;
    }
    if (lane == 0) {
      if (tile && st) {
        __threadfence();
        st[tile] = (2ull << 62) | ((unsigned long long)(prefix + agg) & VMASK);
      }
      s_prefix = prefix;
      if ((uint64_t)(tile + 1) * SC_TILE >= n) out[n] = prefix + agg;   // last tile: total
    }
  }
  __syncthreads();
  T carry = s_prefix;
  for (int k = 0; k < w; ++k) carry += ws[k];
#pragma unroll
  for (int j = 0; j < SC_ITEMS; ++j) {
    uint64_t i = base + j * 32 + lane;
    T inc = warp_incl_scan(x[j], lane);
    if (i < n) out[i] = carry + inc - x[j];
    carry += __shfl_sync(0xffffffffu, inc, 31);
  }
}

template <typename T>
static void scan_impl(gpma *g, const T *in, T *out, uint64_t n, cudaStream_t s) {
  const uint64_t nt = (n + SC_TILE - 1) / SC_TILE > 0 ? (n + SC_TILE - 1) / SC_TILE : 1;
  if (nt == 1) {                       // one tile: no look-back, no status reset
    GP_LAUNCH(g, k_scan_lookback<T>, 1, SC_THREADS, 0, s, in, out, n, (unsigned long long *)nullptr);
    return;
  }
  DevBuf &sb = tl_scan ? *tl_scan : g->b_scan;
  ensure(sb, (nt + 1) * sizeof(unsigned long long), s);
  unsigned long long *status = (unsigned long long *)sb.p;
  fill_zero(g, status, (nt + 1) * sizeof(unsigned long long), s);
  GP_LAUNCH(g, k_scan_lookback<T>, (unsigned)nt, SC_THREADS, 0, s, in, out, n, status);
}

void scan_u32(gpma *g, const uint32_t *in, uint32_t *out, uint64_t n, cudaStream_t s) {
  scan_impl<uint32_t>(g, in, out, n, s);
}

void scan_u64(gpma *g, const uint64_t *in, uint64_t *out, uint64_t n, cudaStream_t s) {
  scan_impl<uint64_t>(g, in, out, n, s);
}

// ------------------------------------------------------------------ radix sort
// Stable LSD radix sort, 8-bit digits, only over the significant key bits (the
// u64 key is src<<32|dst with src,dst < V).  Per pass: tile histograms -> one
// exclusive scan over the digit-major (digit, tile) table -> stable scatter, where
// the rank inside a tile comes from __match_any_sync peer groups per warp round.
constexpr int RS_THREADS = 256;
constexpr int RS_ITEMS = 8;
constexpr int RS_WARPS = RS_THREADS / 32;
constexpr int RS_TILE = RS_THREADS * RS_ITEMS;

// digit of a key: 8 key bits at `shift`, or (div != 0) the owner rank src / div (routing)
__device__ __forceinline__ uint32_t rdigit(uint64_t k, int shift, uint32_t div) {
  return div ? min(255u, (uint32_t)(k >> 32) / div) : (uint32_t)(k >> shift) & 255u;
}

__global__ void __launch_bounds__(RS_THREADS) k_radix_hist(const uint64_t *__restrict__ keys,
                                                           uint64_t n, int shift,
                                                           uint32_t *__restrict__ hist,
                                                           uint32_t ntiles, uint32_t div) {
  __shared__ uint32_t h[256];
  h[threadIdx.x] = 0;
  __syncthreads();
  const uint64_t base = (uint64_t)blockIdx.x * RS_TILE;
#pragma unroll 4
  for (int j = 0; j < RS_ITEMS; ++j) {
    uint64_t i = base + (uint64_t)j * RS_THREADS + threadIdx.x;
    if (i < n) atomicAdd(&h[rdigit(keys[i], shift, div)], 1u);
  }
  __syncthreads();
  hist[(uint64_t)threadIdx.x * ntiles + blockIdx.x] = h[threadIdx.x];
}

__global__ void __launch_bounds__(RS_THREADS) k_radix_scatter(
    const uint64_t *__restrict__ kin, const uint32_t *__restrict__ vin, uint64_t *__restrict__ kout,
    uint32_t *__restrict__ vout, uint64_t n, int shift, const uint32_t *__restrict__ hscan,
    uint32_t ntiles, uint32_t div) {
  __shared__ uint32_t wc[RS_WARPS][256];
  for (int d = threadIdx.x; d < RS_WARPS * 256; d += RS_THREADS) (&wc[0][0])[d] = 0;
  __syncthreads();
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  const uint32_t lt = (1u << lane) - 1u;
  const uint64_t base = (uint64_t)blockIdx.x * RS_TILE + (uint64_t)w * (32 * RS_ITEMS);
  uint64_t k[RS_ITEMS];
  uint32_t v[RS_ITEMS], r[RS_ITEMS];
#pragma unroll
  for (int j = 0; j < RS_ITEMS; ++j) {
    uint64_t i = base + j * 32 + lane;
    bool ok = i < n;
    k[j] = ok ? kin[i] : 0;
    v[j] = ok ? vin[i] : 0;
  }
#pragma unroll
  for (int j = 0; j < RS_ITEMS; ++j) {
    uint64_t i = base + j * 32 + lane;
    bool ok = i < n;
    uint32_t d = ok ? rdigit(k[j], shift, div) : 256u + lane;
    uint32_t peers = __match_any_sync(0xffffffffu, d);
    uint32_t cur = ok ? wc[w][d] : 0u;
    __syncwarp();
    uint32_t rank = __popc(peers & lt);
    if (ok && rank == 0) wc[w][d] = cur + __popc(peers);
    __syncwarp();
    r[j] = cur + rank;
  }
  __syncthreads();
  {
    int d = threadIdx.x;  // 256 threads == 256 digits
    uint32_t run = 0;
#pragma unroll
    for (int ww = 0; ww < RS_WARPS; ++ww) {
      uint32_t t = wc[ww][d];
      wc[ww][d] = run;
      run += t;
    }
  }
  __syncthreads();
#pragma unroll
  for (int j = 0; j < RS_ITEMS; ++j) {
    uint64_t i = base + j * 32 + lane;
    if (i < n) {
      uint32_t d = rdigit(k[j], shift, div);
      uint64_t pos = (uint64_t)hscan[(uint64_t)d * ntiles + blockIdx.x] + wc[w][d] + r[j];
      kout[pos] = k[j];
      vout[pos] = v[j];
    }
  }
}

// Small batches: one CTA sorts (key, arrival index) pairs with a bitonic network in shared
// memory -- stable by construction (the index breaks ties) -- and gathers the values.  One
// launch instead of 4 per radix pass.
constexpr int SS_MAX = 2048;
__global__ void __launch_bounds__(1024) k_small_sort(uint64_t *k0, uint32_t *v0, uint64_t *k1, uint32_t *v1,
                                                     uint32_t n) {
  __shared__ uint64_t sk[SS_MAX];
  __shared__ uint32_t si[SS_MAX];
  uint32_t np2 = 1;
  while (np2 < n) np2 <<= 1;
  for (uint32_t i = threadIdx.x; i < np2; i += blockDim.x) {
    sk[i] = i < n ? k0[i] : ~0ull;
    si[i] = i;
  }
  __syncthreads();
  for (uint32_t size = 2; size <= np2; size <<= 1)
    for (uint32_t stride = size >> 1; stride; stride >>= 1) {
      for (uint32_t i = threadIdx.x; i < np2; i += blockDim.x) {
        const uint32_t j = i ^ stride;
        if (j > i) {
          const bool up = (i & size) == 0;
          const bool gt = sk[i] > sk[j] || (sk[i] == sk[j] && si[i] > si[j]);
          if (gt == up) {
            uint64_t tk = sk[i]; sk[i] = sk[j]; sk[j] = tk;
            uint32_t ti = si[i]; si[i] = si[j]; si[j] = ti;
          }
        }
      }
      __syncthreads();
    }
  for (uint32_t i = threadIdx.x; i < n; i += blockDim.x) {
    k1[i] = sk[i];
    v1[i] = v0[si[i]];
  }
}

int radix_sort_pairs(gpma *g, uint64_t *k0, uint32_t *v0, uint64_t *k1, uint32_t *v1, uint64_t n,
                     const int *shifts, int nshift, cudaStream_t s) {
  if (n <= 1) return 0;
  if (n <= (uint64_t)SS_MAX) {
    GP_LAUNCH(g, k_small_sort, 1, 1024, 0, s, k0, v0, k1, v1, (uint32_t)n);
    return 1;
  }
  const uint32_t ntiles = (uint32_t)((n + RS_TILE - 1) / RS_TILE);
  const uint64_t hn = (uint64_t)ntiles * 256;
  ensure(g->b_hist, (hn + 1) * sizeof(uint32_t), s);
  uint32_t *hist = (uint32_t *)g->b_hist.p;
  uint64_t *ks[2] = {k0, k1};
  uint32_t *vs[2] = {v0, v1};
  int cur = 0;
  for (int p = 0; p < nshift; ++p) {
    GP_LAUNCH(g, k_radix_hist, ntiles, RS_THREADS, 0, s, ks[cur], n, shifts[p], hist, ntiles, 0u);
    scan_u32(g, hist, hist, hn, s);
    GP_LAUNCH(g, k_radix_scatter, ntiles, RS_THREADS, 0, s, ks[cur], vs[cur], ks[cur ^ 1],
              vs[cur ^ 1], n, shifts[p], hist, ntiles, 0u);
    cur ^= 1;
  }
  return cur;
}

__global__ void k_owner_starts(const uint32_t *__restrict__ hscan, uint32_t ntiles, uint32_t nranks,
                               uint64_t n, uint64_t *__restrict__ starts) {
  for (uint32_t d = threadIdx.x; d <= nranks; d += blockDim.x)
    starts[d] = d < nranks ? hscan[(uint64_t)d * ntiles] : n;
}

// One stable counting pass by owner = src / div (the routing step of the sharded store).
gpma_status radix_partition_owner(gpma *g, const uint64_t *k0, const uint32_t *v0, uint64_t *k1, uint32_t *v1,
                                  uint64_t n, uint32_t div, uint32_t nranks, uint64_t *starts_dev,
                                  cudaStream_t s) {
  const uint32_t ntiles = (uint32_t)std::max<uint64_t>(1, (n + RS_TILE - 1) / RS_TILE);
  const uint64_t hn = (uint64_t)ntiles * 256;
  GP_CHECK(g, ensure(g->b_hist, (hn + 1) * sizeof(uint32_t), s));
  uint32_t *hist = (uint32_t *)g->b_hist.p;
  GP_LAUNCH(g, k_radix_hist, ntiles, RS_THREADS, 0, s, k0, n, 0, hist, ntiles, div);
  scan_u32(g, hist, hist, hn, s);
  GP_LAUNCH(g, k_radix_scatter, ntiles, RS_THREADS, 0, s, k0, v0, k1, v1, n, 0, hist, ntiles, div);
  GP_LAUNCH(g, k_owner_starts, 1, 256, 0, s, hist, ntiles, nranks, n, starts_dev);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

}  // namespace gp
