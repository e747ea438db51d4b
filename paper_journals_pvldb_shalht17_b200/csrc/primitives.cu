// primitives.cu -- scans, stable LSD radix sort, thresholds, memory helpers (sm_100a).
//
// Alg. 4 builds GPMA+ from standard GPU primitives (RunLengthEncoding,
// ExclusiveScan; radix sort of the integer keys).  These are this
// library's own implementations -- no CUB / Thrust.
#include <cuda_runtime.h>

#include <algorithm>
#include <chrono>
#include <cstdio>
#include <cstring>
#include <mutex>
#include <unordered_map>
#include <vector>

#include "gpma_internal.cuh"

namespace gp {

// ------------------------------------------------------------------ memory
// Every device allocation of the library goes through dev_alloc / dev_free: the caller's
// hooks (gpma_config.alloc / free / alloc_ctx, e.g. PyTorch's caching allocator) when set,
// else a stream-ordered allocation from a library-owned memory pool of the device.  The
// pool keeps freed blocks mapped while any handle lives on the device (each regrowth of a
// scratch buffer would otherwise map memory again) and is trimmed when the last handle of
// the device is destroyed; the device's default pool (shared with every other
// cudaMallocAsync user of the process) is left alone.
namespace {
std::mutex g_pool_mu;
struct DevPool {
  cudaMemPool_t pool = nullptr;
  int handles = 0;
};
DevPool g_pools[64];

// Blocks >= 1 MiB (store arrays, root-merge and level scratch) freed by the library are kept in a
// per-device cache keyed by exact size and handed back to the next request of that size, with
// an event ordering the reuse after the freeing stream's work.  The pool alone re-mapped
// fragmented free memory for such requests with its reserved size unchanged: 140-510 ms for
// one 0.5-2 GiB request in a resizing step (tools/resize_trace.py, GPMA_TRACE_ALLOC=1).
// GPMA_BLOCK_CACHE=0 disables it.  The cache is emptied into the pool when an allocation
// fails (then the request is retried) and trimmed with the pool on the last destroy.
constexpr size_t BIG_BLOCK = 1u << 20;
struct CachedBlock {
  void *p;
  size_t bytes;
  cudaEvent_t ev;
};
std::vector<CachedBlock> g_cache[64];                 // oldest first
size_t g_cache_bytes[64];
// bytes the cache may hold per device (GPMA_BLOCK_CACHE_MB, default an eighth of the device):
// beyond it the oldest blocks go back to the pool
size_t cache_limit(int dev) {
  static size_t lim[64];
  size_t &l = lim[dev & 63];
  if (!l) {
    size_t fr = 0, tot = 0;
    if (const char *e = getenv("GPMA_BLOCK_CACHE_MB")) l = (size_t)atoll(e) << 20;
    else if (cudaMemGetInfo(&fr, &tot) == cudaSuccess) l = tot / 8;
    else l = (size_t)8 << 30;
    cudaGetLastError();
    if (!l) l = 1;
  }
  return l;
}
std::unordered_map<void *, size_t> g_big_sizes[64];    // live big blocks of the library pool
bool block_cache_on() {
  static const bool on = [] {
    const char *e = getenv("GPMA_BLOCK_CACHE");
    return !e || atoi(e) != 0;
  }();
  return on;
}
// free every cached block of the device to its pool (caller holds g_pool_mu)
void cache_flush_locked(int dev, cudaStream_t s) {
  for (CachedBlock &b : g_cache[dev & 63]) {
    cudaStreamWaitEvent(s, b.ev, 0);
    cudaEventDestroy(b.ev);
    cudaFreeAsync(b.p, s);
  }
  g_cache[dev & 63].clear();
  g_cache_bytes[dev & 63] = 0;
}
}  // namespace

static cudaMemPool_t lib_pool(int dev) {
  std::lock_guard<std::mutex> lk(g_pool_mu);
  DevPool &P = g_pools[dev & 63];
  if (!P.pool) {
    cudaMemPoolProps props{};
    props.allocType = cudaMemAllocationTypePinned;
    props.handleTypes = cudaMemHandleTypeNone;
    props.location.type = cudaMemLocationTypeDevice;
    props.location.id = dev;
    if (cudaMemPoolCreate(&P.pool, &props) != cudaSuccess) {
      cudaGetLastError();
      P.pool = nullptr;
      return nullptr;
    }
    uint64_t thr = ~0ull;
    cudaMemPoolSetAttribute(P.pool, cudaMemPoolAttrReleaseThreshold, &thr);
  }
  return P.pool;
}

void pool_attach(gpma *g) {
  if (g->alloc_fn) return;
  cudaGetDevice(&g->device);
  lib_pool(g->device);
  std::lock_guard<std::mutex> lk(g_pool_mu);
  g_pools[g->device & 63].handles++;
  g->pool_attached = true;
}

// When the device's last handle goes, the pool is trimmed down to GPMA_POOL_KEEP_MB (default: a
// quarter of the device's memory): a later store of the process (e.g. the next pass of a
// benchmark, a re-created graph) reuses mapped blocks instead of mapping GBs again -- mapping is
// what made round-1 resizing steps vary from 16 ms to 1.1 s -- while the rest goes back to the
// driver for a co-resident allocator (PyTorch's).
void pool_detach(gpma *g) {
  if (!g->pool_attached) return;
  std::lock_guard<std::mutex> lk(g_pool_mu);
  DevPool &P = g_pools[g->device & 63];
  if (--P.handles == 0 && P.pool) {
    size_t keep = 0, fr = 0, tot = 0;
    if (const char *e = getenv("GPMA_POOL_KEEP_MB")) keep = (size_t)atoll(e) << 20;
    else if (cudaMemGetInfo(&fr, &tot) == cudaSuccess) keep = tot / 4;
    cudaGetLastError();
    // cached big blocks count against the budget: the largest go back first
    std::vector<CachedBlock> &C = g_cache[g->device & 63];
    std::sort(C.begin(), C.end(), [](const CachedBlock &a, const CachedBlock &b) { return a.bytes < b.bytes; });
    size_t cached = 0;
    for (const CachedBlock &b : C) cached += b.bytes;
    while (!C.empty() && cached > keep) {
      CachedBlock b = C.back();
      C.pop_back();
      cached -= b.bytes;
      g_cache_bytes[g->device & 63] -= b.bytes;
      cudaStreamWaitEvent(g->st, b.ev, 0);
      cudaEventDestroy(b.ev);
      cudaFreeAsync(b.p, g->st);
    }
    cudaStreamSynchronize(g->st);
    cudaMemPoolTrimTo(P.pool, keep - cached);          // every other block is free by now
  }
  g->pool_attached = false;
}

// GPMA_TRACE_ALLOC=1: every allocation >= 64 MiB with its host time on stderr (diagnostics)
static int trace_alloc() {                              // 1: blocks >= 64 MiB, 2: >= 1 MiB
  static const int on = [] {
    const char *e = getenv("GPMA_TRACE_ALLOC");
    return e ? atoi(e) : 0;
  }();
  return on;
}

cudaError_t dev_alloc(gpma *g, void **p, size_t bytes, cudaStream_t s) {
  *p = nullptr;
  const auto t0 = std::chrono::steady_clock::now();
  cudaError_t e;
  if (g->alloc_fn) {
    *p = g->alloc_fn(bytes, (gpma_stream_t)s, g->alloc_ctx);
    e = *p ? cudaSuccess : cudaErrorMemoryAllocation;
  } else {
    cudaMemPool_t pool = lib_pool(g->device);
    const bool big = pool && bytes >= BIG_BLOCK && block_cache_on();
    e = cudaErrorMemoryAllocation;
    if (big) {
      std::lock_guard<std::mutex> lk(g_pool_mu);
      std::vector<CachedBlock> &C = g_cache[g->device & 63];
      for (size_t i = 0; i < C.size(); ++i)
        if (C[i].bytes == bytes) {
          *p = C[i].p;
          cudaStreamWaitEvent(s, C[i].ev, 0);          // after the freeing stream's last use
          cudaEventDestroy(C[i].ev);
          g_cache_bytes[g->device & 63] -= C[i].bytes;
          C.erase(C.begin() + (long)i);
          g_big_sizes[g->device & 63][*p] = bytes;
          e = cudaSuccess;
          break;
        }
    }
    if (e != cudaSuccess) {
      e = pool ? cudaMallocFromPoolAsync(p, bytes, pool, s) : cudaMallocAsync(p, bytes, s);
      if (e != cudaSuccess && big) {                  // give the cached blocks back, retry once
        cudaGetLastError();
        {
          std::lock_guard<std::mutex> lk(g_pool_mu);
          cache_flush_locked(g->device, s);
        }
        e = cudaMallocFromPoolAsync(p, bytes, pool, s);
      }
      if (e != cudaSuccess) {
        cudaGetLastError();
        *p = nullptr;
      } else if (big) {
        std::lock_guard<std::mutex> lk(g_pool_mu);
        g_big_sizes[g->device & 63][*p] = bytes;
      }
    }
  }
  if (trace_alloc() && bytes >= (trace_alloc() > 1 ? (1u << 20) : (64u << 20))) {
    uint64_t res = 0, used = 0;
    if (!g->alloc_fn) {
      cudaMemPool_t pool = lib_pool(g->device);
      cudaMemPoolGetAttribute(pool, cudaMemPoolAttrReservedMemCurrent, &res);
      cudaMemPoolGetAttribute(pool, cudaMemPoolAttrUsedMemCurrent, &used);
    }
    fprintf(stderr, "[gpma] dev_alloc %.1f MiB: %.3f ms (%s; pool reserved %.0f used %.0f MiB)\n", bytes / 1048576.0,
            std::chrono::duration<double, std::milli>(std::chrono::steady_clock::now() - t0).count(),
            e == cudaSuccess ? "ok" : "failed", res / 1048576.0, used / 1048576.0);
  }
  return e;
}

void dev_free(gpma *g, void *p, cudaStream_t s) {
  if (!p) return;
  if (g->alloc_fn) {
    if (g->free_fn) g->free_fn(p, (gpma_stream_t)s, g->alloc_ctx);
    return;
  }
  {
    std::lock_guard<std::mutex> lk(g_pool_mu);
    auto &M = g_big_sizes[g->device & 63];
    auto it = M.find(p);
    if (it != M.end()) {
      CachedBlock b{p, it->second, nullptr};
      M.erase(it);
      if (cudaEventCreateWithFlags(&b.ev, cudaEventDisableTiming) == cudaSuccess &&
          cudaEventRecord(b.ev, s) == cudaSuccess) {
        std::vector<CachedBlock> &C = g_cache[g->device & 63];
        size_t &cb = g_cache_bytes[g->device & 63];
        C.push_back(b);
        cb += b.bytes;
        const size_t lim = cache_limit(g->device);
        while (cb > lim && C.size() > 1) {             // the oldest go back to the pool
          CachedBlock o = C.front();
          C.erase(C.begin());
          cb -= o.bytes;
          cudaStreamWaitEvent(s, o.ev, 0);
          cudaEventDestroy(o.ev);
          cudaFreeAsync(o.p, s);
        }
        return;
      }
      cudaGetLastError();
      if (b.ev) cudaEventDestroy(b.ev);
    }
  }
  cudaFreeAsync(p, s);
}

// At least `bytes` in b (grown x1.5 to amortise regrowth; on failure retried at exactly
// `bytes`).  On failure b is empty and the error is returned: every caller checks it.
cudaError_t ensure(gpma *g, DevBuf &b, size_t bytes, cudaStream_t s) {
  if (bytes == 0) bytes = 16;
  if (b.bytes >= bytes) return cudaSuccess;
  size_t want = std::max(bytes, b.bytes + b.bytes / 2);
  // Scratch >= 1 MiB in power-of-two sizes: the pool serves a request from one free chunk, and
  // chunks freed by a previous store / scratch of another size made it re-map fragmented free
  // memory (8-14 ms per 256-512 MiB request with the pool's reserved size unchanged,
  // tools/resize_trace.py with GPMA_TRACE_ALLOC=1; 1-5 ms, sometimes 40-80 ms, for the 14-32 MiB
  // level buffers of the configs[3] grow phase, tools/step_trace.py); equal size classes reuse
  // whole chunks.
  if (want >= (1u << 20)) {
    size_t p2 = 1u << 20;
    while (p2 < want) p2 <<= 1;
    want = p2;
  }
  dev_free(g, b.p, s);
  b.p = nullptr;
  b.bytes = 0;
  cudaError_t e = dev_alloc(g, &b.p, want, s);
  if (e != cudaSuccess && want > bytes) {
    e = dev_alloc(g, &b.p, bytes, s);
    if (e == cudaSuccess) b.bytes = bytes;
  } else if (e == cudaSuccess) {
    b.bytes = want;
  }
  if (e != cudaSuccess) b.p = nullptr;
  return e;
}

void release(gpma *g, DevBuf &b, cudaStream_t s) {
  dev_free(g, b.p, s);
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
// Scans of >= 2^22 items use 16K-item tiles: the look-back's inclusive prefix advances one
// 32-tile window per L2 round trip, so 4K-item tiles put ~128 round trips on the critical path
// of a 2^24-item scan (the export's leaf offsets: 107 us, 1.6 TB/s); small scans keep 4K tiles
// (more CTAs, measured faster for the BFS / level-loop sizes).
constexpr int SC_BIG_THREADS = 1024;
constexpr uint64_t SC_BIG_MIN = 1ull << 22;

template <typename T>
__device__ __forceinline__ T warp_sum(T x) {
  for (int o = 16; o; o >>= 1) x += __shfl_xor_sync(0xffffffffu, x, o);
  return x;
}

template <typename T>
__device__ __forceinline__ T warp_incl_scan(T x, int lane) {
  for (int o = 1; o < 32; o <<= 1) {
    T y = __shfl_up_sync(0xffffffffu, x, o);
    if (lane >= o) x += y;
  }
  return x;
}

template <typename T>
struct ScanIn {                     // the plain input array
  const T *in;
  __device__ __forceinline__ T operator()(uint64_t i) const { return in[i]; }
};

// Single-pass exclusive scan with decoupled look-back (Merrill & Garland): each CTA takes the
// next tile (atomic counter), publishes its aggregate, then sums predecessors' published
// values back to the first inclusive prefix.  out[n] = total.  Status words live in
// `status` (zeroed by the caller): [flag:2 | value:62], flag 1 = aggregate, 2 = inclusive.
// In(i) yields item i (i < n), so producers can be fused into the scan.
template <typename T, int NT, class In>
__global__ void __launch_bounds__(NT) k_scan_lookback(In in, T *out, uint64_t n, unsigned long long *status) {
  constexpr int TILE = NT * SC_ITEMS;
  __shared__ uint32_t s_tile;
  __shared__ T ws[NT / 32];
  __shared__ T s_prefix;
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5;
  if (threadIdx.x == 0) s_tile = status ? (uint32_t)atomicAdd(status, 1ull) : 0u;  // status[0] = tile counter
  __syncthreads();
  const uint32_t tile = s_tile;
  volatile unsigned long long *st = status ? status + 1 : nullptr;   // null: single tile
  const uint64_t base = (uint64_t)tile * TILE + (uint64_t)w * (32 * SC_ITEMS);
  T x[SC_ITEMS];
  T part = 0;
#pragma unroll
  for (int j = 0; j < SC_ITEMS; ++j) {
    uint64_t i = base + j * 32 + lane;
    x[j] = i < n ? in(i) : T(0);
    part += x[j];
  }
  T wtot = warp_sum(part);
  if (lane == 0) ws[w] = wtot;
  __syncthreads();
  if (w == 0) {
    T agg = 0;
    for (int k = 0; k < NT / 32; ++k) agg += ws[k];
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
      if ((uint64_t)(tile + 1) * TILE >= n) out[n] = prefix + agg;   // last tile: total
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

template <typename T, class In>
static cudaError_t scan_fn(gpma *g, const In &in, T *out, uint64_t n, cudaStream_t s) {
  const bool big = n >= SC_BIG_MIN;
  const uint64_t tile = big ? (uint64_t)SC_BIG_THREADS * SC_ITEMS : (uint64_t)SC_TILE;
  const uint64_t nt = (n + tile - 1) / tile > 0 ? (n + tile - 1) / tile : 1;
  if (nt == 1) {                       // one tile: no look-back, no status reset
    GP_LAUNCH(g, (k_scan_lookback<T, SC_THREADS, In>), 1, SC_THREADS, 0, s, in, out, n,
              (unsigned long long *)nullptr);
    return cudaGetLastError();
  }
  DevBuf &sb = tl_scan ? *tl_scan : g->b_scan;
  cudaError_t e = ensure(g, sb, (nt + 1) * sizeof(unsigned long long), s);
  if (e != cudaSuccess) return e;
  unsigned long long *status = (unsigned long long *)sb.p;
  if ((e = fill_zero(g, status, (nt + 1) * sizeof(unsigned long long), s)) != cudaSuccess) return e;
  if (big)
    GP_LAUNCH(g, (k_scan_lookback<T, SC_BIG_THREADS, In>), (unsigned)nt, SC_BIG_THREADS, 0, s, in, out, n, status);
  else
    GP_LAUNCH(g, (k_scan_lookback<T, SC_THREADS, In>), (unsigned)nt, SC_THREADS, 0, s, in, out, n, status);
  return cudaGetLastError();
}

template <typename T>
static cudaError_t scan_impl(gpma *g, const T *in, T *out, uint64_t n, cudaStream_t s) {
  return scan_fn<T>(g, ScanIn<T>{in}, out, n, s);
}

// live edges per leaf (live count minus guards), scanned: the export's per-leaf output offsets
struct LeafEdges {
  const uint32_t *cnt, *gl;
  __device__ __forceinline__ uint64_t operator()(uint64_t l) const { return (uint64_t)(cnt[l] - gl[l]); }
};
cudaError_t scan_leaf_edges(gpma *g, const uint32_t *cnt, const uint32_t *gl, uint64_t *out, uint64_t nl,
                            cudaStream_t s) {
  return scan_fn<uint64_t>(g, LeafEdges{cnt, gl}, out, nl, s);
}

cudaError_t scan_u32(gpma *g, const uint32_t *in, uint32_t *out, uint64_t n, cudaStream_t s) {
  return scan_impl<uint32_t>(g, in, out, n, s);
}

cudaError_t scan_u64(gpma *g, const uint64_t *in, uint64_t *out, uint64_t n, cudaStream_t s) {
  return scan_impl<uint64_t>(g, in, out, n, s);
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
  uint32_t np2 = 2;
  while (np2 < n) np2 <<= 1;
  for (uint32_t i = threadIdx.x; i < np2; i += blockDim.x) {
    sk[i] = i < n ? k0[i] : ~0ull;
    si[i] = i;
  }
  __syncthreads();
  cta_bitonic_sort(sk, si, np2);           // (key, arrival index): stable
  for (uint32_t i = threadIdx.x; i < n; i += blockDim.x) {
    k1[i] = sk[i];
    v1[i] = v0[si[i]];
  }
}

// ---- onesweep LSD radix sort (the sort of every update batch, Alg. 4 l.2)
// One read of the keys builds the digit histograms of every pass (k_os_hist); then each pass is
// ONE kernel (k_os_pass): a CTA takes the next 4096-key tile (tile ids from an atomic counter,
// so every predecessor is already resident), ranks its keys stably per warp (__match_any_sync
// peer groups, in input order), publishes its per-digit counts and walks back over the
// predecessors' published (aggregate | inclusive) counts digit by digit (decoupled look-back),
// reorders the tile by digit in shared memory and writes each digit's run contiguously.
// 2 + passes launches per sort instead of 4 per pass (hist, zero, scan, scatter), and the
// batch (12 B per key, <= 12 MiB at 2^20) stays L2-resident across the passes.
// Status words: [flag:2 | count:62]; flag 0 = not ready, 1 = tile aggregate, 2 = inclusive prefix.
// Two status regions alternate between passes: the histogram kernel zeroes both (ntiles x 256
// words each), and pass p's tile t zeroes its slot of the region pass p-1 used, which pass p+1
// uses next -- so every pass finds its region zero with no host-side state (graph-replay safe).
constexpr int OS_T = 256, OS_I = 16, OS_TILE = OS_T * OS_I, OS_W = OS_T / 32;
constexpr int OS_MAXPASS = 8;
struct OsPasses {
  int shift[OS_MAXPASS];
  int n;
};
constexpr uint64_t OS_CNT_MASK = (1ull << 62) - 1;
constexpr size_t OS_SMEM = (size_t)OS_TILE * 8 + (size_t)OS_TILE * 4 + (size_t)OS_W * 256 * 4 + 256 * 4 * 2 + 256 * 8;

__global__ void __launch_bounds__(OS_T) k_os_hist(const uint64_t *__restrict__ keys, uint64_t n, OsPasses ps,
                                                  uint32_t *__restrict__ ghist, uint4 *__restrict__ status,
                                                  uint64_t status_words16) {
  __shared__ uint32_t h[OS_MAXPASS][256];
  for (int i = threadIdx.x; i < OS_MAXPASS * 256; i += OS_T) (&h[0][0])[i] = 0;
  for (uint64_t i = blockIdx.x * (uint64_t)OS_T + threadIdx.x; i < status_words16; i += (uint64_t)gridDim.x * OS_T)
    status[i] = make_uint4(0, 0, 0, 0);               // both status regions
  __syncthreads();
  const uint64_t stride = (uint64_t)gridDim.x * OS_T * 2;
  for (uint64_t i = (blockIdx.x * (uint64_t)OS_T + threadIdx.x) * 2; i < n; i += stride) {
    uint64_t k0, k1 = 0;
    const bool two = i + 1 < n;
    if (two) {
      const ulonglong2 kk = __ldg(reinterpret_cast<const ulonglong2 *>(keys + i));
      k0 = kk.x;
      k1 = kk.y;
    } else {
      k0 = keys[i];
    }
    for (int p = 0; p < ps.n; ++p) {
      atomicAdd(&h[p][(uint32_t)(k0 >> ps.shift[p]) & 255u], 1u);
      if (two) atomicAdd(&h[p][(uint32_t)(k1 >> ps.shift[p]) & 255u], 1u);
    }
  }
  __syncthreads();
  for (int i = threadIdx.x; i < ps.n * 256; i += OS_T) {
    const uint32_t c = (&h[0][0])[i];
    if (c) atomicAdd(ghist + i, c);
  }
}

template <bool HASV>
__global__ void __launch_bounds__(OS_T, 2) k_os_pass(const uint64_t *__restrict__ kin, const uint32_t *__restrict__ vin,
                                                     uint64_t *__restrict__ kout, uint32_t *__restrict__ vout,
                                                     uint64_t n, int shift, const uint32_t *__restrict__ ghist,
                                                     unsigned long long *status, unsigned long long *status_prev,
                                                     uint32_t *tile_ctr) {
  extern __shared__ __align__(16) unsigned char os_smem[];
  uint64_t *sk = reinterpret_cast<uint64_t *>(os_smem);                           // [OS_TILE]
  uint32_t *sv = reinterpret_cast<uint32_t *>(sk + OS_TILE);                      // [OS_TILE]
  uint32_t *wc = sv + OS_TILE;                                                    // [OS_W][256]
  uint32_t *ldoff = wc + OS_W * 256;                                              // [256]
  uint32_t *sbase = ldoff + 256;                                                  // [256] (digit bases, then tile id)
  uint64_t *gofs = reinterpret_cast<uint64_t *>(sbase + 256);                     // [256]
  const int lane = threadIdx.x & 31, w = threadIdx.x >> 5, t = threadIdx.x;
  const uint32_t lt = (1u << lane) - 1u;
  for (int i = t; i < OS_W * 256; i += OS_T) wc[i] = 0;
  // exclusive scan of the pass's global digit histogram (digit t) -> bases of the digit runs
  const uint32_t gh = ghist[t];
  {
    uint32_t x = gh;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
      if (lane >= o) x += y;
    }
    if (lane == 31) ldoff[w] = x;                    // warp totals (ldoff reused as scratch)
    __syncthreads();
    uint32_t pre = 0;
    for (int k = 0; k < w; ++k) pre += ldoff[k];
    sbase[t] = pre + x - gh;
  }
  if (t == 0) ldoff[OS_W] = atomicAdd(tile_ctr, 1u);   // the tile of this CTA
  __syncthreads();
  const uint64_t tile = ldoff[OS_W];
  const uint64_t dbase = sbase[t];
  if (status_prev) status_prev[tile * 256 + t] = 0ull;   // the region pass p+1 uses (pass p-1 is done)
  __syncthreads();
  const uint64_t t0 = tile * OS_TILE;
  const uint64_t base = t0 + (uint64_t)w * (32 * OS_I);
  uint64_t k[OS_I];
  uint32_t v[OS_I], r[OS_I];
#pragma unroll
  for (int j = 0; j < OS_I; ++j) {
    const uint64_t i = base + j * 32 + lane;
    k[j] = i < n ? kin[i] : 0ull;
    if (HASV) v[j] = i < n ? vin[i] : 0u;
  }
  // stable per-warp ranks in input order (j-major, lane-minor)
#pragma unroll
  for (int j = 0; j < OS_I; ++j) {
    const uint64_t i = base + j * 32 + lane;
    const bool ok = i < n;
    const uint32_t d = ok ? (uint32_t)(k[j] >> shift) & 255u : 256u + lane;
    const uint32_t peers = __match_any_sync(0xffffffffu, d);
    const uint32_t cur = ok ? wc[w * 256 + d] : 0u;
    __syncwarp();
    const uint32_t rank = __popc(peers & lt);
    if (ok && rank == 0) wc[w * 256 + d] = cur + __popc(peers);
    __syncwarp();
    r[j] = cur + rank;
  }
  __syncthreads();
  // digit t: offsets of the warps inside the tile, tile count
  uint32_t run = 0;
#pragma unroll
  for (int ww = 0; ww < OS_W; ++ww) {
    const uint32_t c = wc[ww * 256 + t];
    wc[ww * 256 + t] = run;
    run += c;
  }
  // publish the tile's aggregate for digit t as early as possible (successors sum it)
  volatile unsigned long long *st = status;
  {
    const unsigned long long word = ((tile == 0 ? 2ull : 1ull) << 62) | (unsigned long long)run;
    __threadfence();
    st[tile * 256 + t] = word;
  }
  // local digit offsets inside the tile (exclusive scan of the tile counts over digits), then
  // the tile reordered by digit in shared memory -- all before the look-back, so the keys do
  // not occupy registers while it waits
  {
    uint32_t x = run;
#pragma unroll
    for (int o = 1; o < 32; o <<= 1) {
      const uint32_t y = __shfl_up_sync(0xffffffffu, x, o);
      if (lane >= o) x += y;
    }
    if (lane == 31) sbase[w] = x;
    __syncthreads();
    uint32_t pre = 0;
    for (int kk = 0; kk < w; ++kk) pre += sbase[kk];
    ldoff[t] = pre + x - run;
  }
  __syncthreads();
#pragma unroll
  for (int j = 0; j < OS_I; ++j) {
    const uint64_t i = base + j * 32 + lane;
    if (i < n) {
      const uint32_t d = (uint32_t)(k[j] >> shift) & 255u;
      const uint32_t lp = ldoff[d] + wc[w * 256 + d] + r[j];
      sk[lp] = k[j];
      if (HASV) sv[lp] = v[j];
    }
  }
  // windowed look-back: the words of 16 predecessors are loaded independently per round (a
  // serial walk pays one L2 round trip per predecessor while the tiles of a wave finish)
  uint64_t excl = 0;
  for (int64_t p = (int64_t)tile - 1; p >= 0; p -= 16) {
    unsigned long long x[16];
#pragma unroll
    for (int q = 0; q < 16; ++q) x[q] = p - q >= 0 ? st[(uint64_t)(p - q) * 256 + t] : (2ull << 62);
    bool done = false;
#pragma unroll
    for (int q = 0; q < 16; ++q) {
      if (done) break;
      while ((x[q] >> 62) == 0) x[q] = st[(uint64_t)(p - q) * 256 + t];
      excl += x[q] & OS_CNT_MASK;
      done = (x[q] >> 62) == 2;
    }
    if (done) break;
  }
  if (tile) {
    __threadfence();
    st[tile * 256 + t] = (2ull << 62) | (unsigned long long)(excl + run);
  }
  gofs[t] = dbase + excl;
  __syncthreads();
  // write each digit's run contiguously
  const uint32_t nt = (uint32_t)min((uint64_t)OS_TILE, n - t0);
#pragma unroll 4
  for (uint32_t i = t; i < nt; i += OS_T) {
    const uint64_t kk = sk[i];
    const uint32_t d = (uint32_t)(kk >> shift) & 255u;
    const uint64_t pos = gofs[d] + (i - ldoff[d]);
    kout[pos] = kk;
    if (HASV) vout[pos] = sv[i];
  }
}

// Sort (k0, v0)[0..n) by the given 8-bit digit shifts (stable); v0 == nullptr sorts keys only.
// *which = the buffer pair (0: k0/v0, 1: k1/v1) holding the result.
cudaError_t radix_sort_pairs(gpma *g, uint64_t *k0, uint32_t *v0, uint64_t *k1, uint32_t *v1, uint64_t n,
                             const int *shifts, int nshift, cudaStream_t s, int *which) {
  *which = 0;
  if (n <= 1 || nshift == 0) return cudaSuccess;
  if (n <= (uint64_t)SS_MAX && v0) {
    GP_LAUNCH(g, k_small_sort, 1, 1024, 0, s, k0, v0, k1, v1, (uint32_t)n);
    *which = 1;
    return cudaGetLastError();
  }
  static const bool attr = [] {
    cudaFuncSetAttribute(k_os_pass<true>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)OS_SMEM);
    cudaFuncSetAttribute(k_os_pass<false>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)OS_SMEM);
    return true;
  }();
  (void)attr;
  const uint64_t ntiles = (n + OS_TILE - 1) / OS_TILE;
  const size_t ctl = 64 + (size_t)OS_MAXPASS * 256 * 4;        // tile counters + histograms
  const uint64_t region = ntiles * 256;                         // status words per region
  cudaError_t e = ensure(g, g->b_hist, ctl + 2 * region * 8, s);
  if (e != cudaSuccess) return e;
  char *base = (char *)g->b_hist.p;
  uint32_t *ctr = (uint32_t *)base;
  uint32_t *ghist = (uint32_t *)(base + 64);
  unsigned long long *status = (unsigned long long *)(base + ctl);
  if ((e = fill_zero(g, base, ctl, s)) != cudaSuccess) return e;
  OsPasses ps{};
  ps.n = nshift;
  for (int p = 0; p < nshift; ++p) ps.shift[p] = shifts[p];
  GP_LAUNCH(g, k_os_hist, grid_for((n + 1) / 2, OS_T, num_sms() * 4), OS_T, 0, s, k0, n, ps, ghist,
            (uint4 *)status, region * 2 * 8 / 16);
  uint64_t *ks[2] = {k0, k1};
  uint32_t *vs[2] = {v0, v1};
  int cur = 0;
  for (int p = 0; p < nshift; ++p) {
    unsigned long long *sp = status + (uint64_t)(p & 1) * region;
    unsigned long long *sq = p ? status + (uint64_t)((p - 1) & 1) * region : nullptr;
    if (v0)
      GP_LAUNCH(g, k_os_pass<true>, (unsigned)ntiles, OS_T, OS_SMEM, s, ks[cur], vs[cur], ks[cur ^ 1], vs[cur ^ 1], n,
                shifts[p], ghist + p * 256, sp, sq, ctr + p);
    else
      GP_LAUNCH(g, k_os_pass<false>, (unsigned)ntiles, OS_T, OS_SMEM, s, ks[cur], (const uint32_t *)nullptr,
                ks[cur ^ 1], (uint32_t *)nullptr, n, shifts[p], ghist + p * 256, sp, sq, ctr + p);
    cur ^= 1;
  }
  *which = cur;
  return cudaGetLastError();
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
  GP_CHECK(g, ensure(g, g->b_misc3, (hn + 1) * sizeof(uint32_t), s));
  uint32_t *hist = (uint32_t *)g->b_misc3.p;
  GP_LAUNCH(g, k_radix_hist, ntiles, RS_THREADS, 0, s, k0, n, 0, hist, ntiles, div);
  GP_CHECK(g, scan_u32(g, hist, hist, hn, s));
  GP_LAUNCH(g, k_radix_scatter, ntiles, RS_THREADS, 0, s, k0, v0, k1, v1, n, 0, hist, ntiles, div);
  GP_LAUNCH(g, k_owner_starts, 1, 256, 0, s, hist, ntiles, nranks, n, starts_dev);
  GP_CHECK(g, cudaGetLastError());
  return GPMA_OK;
}

}  // namespace gp
