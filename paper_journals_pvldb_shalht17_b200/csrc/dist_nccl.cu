// dist_nccl.cu -- the multi-GPU GPMA+ behind the C ABI (SURVEY §8(b) gpma_dist_create, §8(e)).
//
// PAPER.md §6.4: "We evenly partition graphs according to the vertex index and
// synchronize all devices after each iteration."  One process per GPU; rank r holds an
// independent GPMA+ shard over the source rows [r*ceil(V/P), (r+1)*ceil(V/P)) (R24).  The
// library owns an NCCL communicator (NVLink / NVSwitch on a B200 box) and runs every exchange
// itself, between its own kernels, on the caller's stream:
//   update:   validate the rank's slice (global range) -> MAX all-reduce of the status, so a bad
//             key anywhere rejects the batch on EVERY rank before anything mutates -> stable
//             partition by owner (one counting pass) -> counts and payload all-to-all-v
//             (grouped ncclSend/ncclRecv; the rank-order concatenation keeps the global batch
//             order, so the last occurrence still wins, R10) -> the local GPMA+ batch.
//   BFS:      replicated levels; per level the owned frontier rows are expanded, the ranks'
//             discoveries are all-gathered as bitmaps (V/8 B per rank) and merged.
//   CC:       replicated labels; a hooking round over the owned edges, MIN all-reduce of the
//             labels, SUM all-reduce of the change count; stop at the fixpoint (min-id, R19).
//   PageRank: push of the owned rows into an exact 64-bit fixed-point y, REDUCE-SCATTER to the
//             owners, the dangling mass and the L1 error as one-word all-reduces (one host read
//             per iteration), the owned slice updated; one ALL-GATHER of the slices at the end.
// NCCL is loaded at run time (dlopen; the copy the process already has -- e.g. PyTorch's -- if
// any), so single-GPU users never need it.
#include <cuda_runtime.h>
#include <dlfcn.h>
#include <nccl.h>

#include <cstring>
#include <mutex>
#include <vector>

#include "gpma_internal.cuh"

namespace gp {

namespace {

struct Nccl {
  bool ok = false;
  std::string why;
  ncclResult_t (*GetUniqueId)(ncclUniqueId *) = nullptr;
  ncclResult_t (*CommInitRank)(ncclComm_t *, int, ncclUniqueId, int) = nullptr;
  ncclResult_t (*CommDestroy)(ncclComm_t) = nullptr;
  ncclResult_t (*AllReduce)(const void *, void *, size_t, ncclDataType_t, ncclRedOp_t, ncclComm_t,
                            cudaStream_t) = nullptr;
  ncclResult_t (*ReduceScatter)(const void *, void *, size_t, ncclDataType_t, ncclRedOp_t, ncclComm_t,
                                cudaStream_t) = nullptr;
  ncclResult_t (*AllGather)(const void *, void *, size_t, ncclDataType_t, ncclComm_t, cudaStream_t) = nullptr;
  ncclResult_t (*Send)(const void *, size_t, ncclDataType_t, int, ncclComm_t, cudaStream_t) = nullptr;
  ncclResult_t (*Recv)(void *, size_t, ncclDataType_t, int, ncclComm_t, cudaStream_t) = nullptr;
  ncclResult_t (*GroupStart)() = nullptr;
  ncclResult_t (*GroupEnd)() = nullptr;
  const char *(*GetErrorString)(ncclResult_t) = nullptr;
};

Nccl &nccl() {
  static Nccl N;
  static std::once_flag once;
  std::call_once(once, [] {
    void *h = nullptr;
    const char *env = getenv("GPMA_NCCL_LIB");
    if (env && *env) h = dlopen(env, RTLD_NOW | RTLD_GLOBAL);
    if (!h) h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_GLOBAL | RTLD_NOLOAD);   // already in the process
    if (!h) h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_GLOBAL);
    if (!h) h = dlopen("libnccl.so", RTLD_NOW | RTLD_GLOBAL);
    if (!h) {
      N.why = std::string("cannot load NCCL: ") + dlerror();
      return;
    }
#define GP_SYM(f)                                                   \
  *(void **)(&N.f) = dlsym(h, "nccl" #f);                           \
  if (!N.f) {                                                       \
    N.why = "NCCL symbol missing: nccl" #f;                         \
    return;                                                         \
  }
    GP_SYM(GetUniqueId) GP_SYM(CommInitRank) GP_SYM(CommDestroy) GP_SYM(AllReduce) GP_SYM(ReduceScatter)
    GP_SYM(AllGather) GP_SYM(Send) GP_SYM(Recv) GP_SYM(GroupStart) GP_SYM(GroupEnd) GP_SYM(GetErrorString)
#undef GP_SYM
    N.ok = true;
  });
  return N;
}

gpma_status nccl_fail(gpma *g, ncclResult_t r, const char *where) {
  g->poisoned = true;
  set_err(g, std::string("NCCL ") + (nccl().GetErrorString ? nccl().GetErrorString(r) : "?") + " in " + where);
  return GPMA_ERR_CUDA;
}

#define NC_CHECK(g, call)                                            \
  do {                                                               \
    ncclResult_t r_ = (call);                                        \
    if (r_ != ncclSuccess) return nccl_fail((g), r_, #call);         \
  } while (0)

inline ncclComm_t comm_of(gpma *g) { return (ncclComm_t)g->comm; }

}  // namespace

// R24: the rows of rank r
void dist_rows(uint32_t V, int P, int r, uint32_t *rb, uint32_t *re) {
  const uint64_t chunk = ((uint64_t)V + P - 1) / P;
  const uint64_t lo = std::min<uint64_t>(V, chunk * r);
  *rb = (uint32_t)lo;
  *re = (uint32_t)std::min<uint64_t>(V, lo + chunk);
}


// Route this rank's slice (keys/vals, any memory) to the owners: returns the owned batch in
// d_k[1]/d_v[1] (*m entries, rank order).  A slice with a bad key anywhere is rejected on every
// rank (one MAX all-reduce of the validation bits) before anything is exchanged or mutated.
static gpma_status dist_exchange(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, bool check_vals,
                                 uint64_t *m, cudaStream_t s) {
  const uint32_t P = (uint32_t)g->nranks;
  GP_CHECK(g, ensure(g, g->d_k[0], std::max<uint64_t>(n, 1) * 8, s));
  GP_CHECK(g, ensure(g, g->d_v[0], std::max<uint64_t>(n, 1) * 4, s));
  uint64_t *sk = (uint64_t *)g->d_k[0].p;
  uint32_t *sv = (uint32_t *)g->d_v[0].p;
  // validation bits of every rank's slice, reduced before anything is exchanged or mutated
  gpma_status st = validate_slice(g, keys, vals, n, check_vals && vals, s);
  if (st) return st;
  NC_CHECK(g, nccl().AllReduce(&g->ctrl_d->err, &g->ctrl_d->err, 1, ncclUint32, ncclMax, comm_of(g), s));
  GP_CHECK(g, readback(g, g->ctrl_h, g->ctrl_d, sizeof(Ctrl), s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  if (g->ctrl_h->err & 2u) return GPMA_ERR_RESERVED;
  if (g->ctrl_h->err & 1u) return GPMA_ERR_RANGE;
  // stable partition of the slice by owner (route() stages the caller's slice itself)
  std::vector<uint64_t> cnt_h(P, 0);
  if ((st = route(g, keys, vals, n, P, sk, sv, cnt_h.data(), s))) return st;
  // counts all-to-all (one u64 per peer), then the payload all-to-all-v
  GP_CHECK(g, ensure(g, g->d_misc, (size_t)(4 * P + 2) * 8, s));
  unsigned long long *scnt = (unsigned long long *)g->d_misc.p, *rcnt = scnt + P;
  std::vector<uint64_t> hc(2 * P);
  for (uint32_t r = 0; r < P; ++r) hc[r] = cnt_h[r];
  GP_CHECK(g, cudaMemcpyAsync(scnt, hc.data(), P * 8, cudaMemcpyHostToDevice, s));
  NC_CHECK(g, nccl().GroupStart());
  for (uint32_t r = 0; r < P; ++r) {
    NC_CHECK(g, nccl().Send(scnt + r, 1, ncclUint64, (int)r, comm_of(g), s));
    NC_CHECK(g, nccl().Recv(rcnt + r, 1, ncclUint64, (int)r, comm_of(g), s));
  }
  NC_CHECK(g, nccl().GroupEnd());
  GP_CHECK(g, cudaMemcpyAsync(hc.data() + P, rcnt, P * 8, cudaMemcpyDeviceToHost, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  uint64_t tot = 0;
  for (uint32_t r = 0; r < P; ++r) tot += hc[P + r];
  GP_CHECK(g, ensure(g, g->d_k[1], std::max<uint64_t>(tot, 1) * 8, s));
  GP_CHECK(g, ensure(g, g->d_v[1], std::max<uint64_t>(tot, 1) * 4, s));
  uint64_t *rk = (uint64_t *)g->d_k[1].p;
  uint32_t *rv = (uint32_t *)g->d_v[1].p;
  uint64_t so = 0, ro = 0;
  NC_CHECK(g, nccl().GroupStart());
  for (uint32_t r = 0; r < P; ++r) {
    const uint64_t sc = hc[r], rc = hc[P + r];
    if (sc) {
      NC_CHECK(g, nccl().Send(sk + so, sc, ncclUint64, (int)r, comm_of(g), s));
      if (vals) NC_CHECK(g, nccl().Send(sv + so, sc, ncclUint32, (int)r, comm_of(g), s));
    }
    if (rc) {
      NC_CHECK(g, nccl().Recv(rk + ro, rc, ncclUint64, (int)r, comm_of(g), s));
      if (vals) NC_CHECK(g, nccl().Recv(rv + ro, rc, ncclUint32, (int)r, comm_of(g), s));
    }
    so += sc;
    ro += rc;
  }
  NC_CHECK(g, nccl().GroupEnd());
  *m = tot;
  return GPMA_OK;
}

gpma_status dist_update(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, int op, cudaStream_t s) {
  uint64_t m = 0;
  gpma_status st = dist_exchange(g, keys, op == GPMA_INSERT ? vals : nullptr, n, op == GPMA_INSERT, &m, s);
  if (st) {
    g->last = gpma_stats_t{};
    return st;
  }
  return update_batch(g, (const uint64_t *)g->d_k[1].p, op == GPMA_INSERT ? (const uint32_t *)g->d_v[1].p : nullptr,
                      m, op, s);
}

gpma_status dist_bfs(gpma *g, uint32_t root, int32_t *levels, cudaStream_t s) {
  const uint64_t words = ((uint64_t)g->V + 31) / 32;
  const uint32_t P = (uint32_t)g->nranks;
  GP_CHECK(g, ensure(g, g->an[AN_BFS].stage[0], words * 4 * (P + 1), s));
  uint32_t *bm = (uint32_t *)g->an[AN_BFS].stage[0].p, *bms = bm + words;
  gpma_status st = bfs_init(g, root, levels, s);
  if (st) return st;
  for (int32_t depth = 1;; ++depth) {
    uint32_t F = 0;
    if ((st = bfs_level(g, levels, depth, &F, s))) return st;   // F: the replicated frontier
    if (F == 0) break;
    if (P > 1) {
      if ((st = bfs_bits(g, levels, depth, bm, s))) return st;
      NC_CHECK(g, nccl().AllGather(bm, bms, words, ncclUint32, comm_of(g), s));
      if ((st = bfs_merge(g, levels, bms, P, depth, s))) return st;
    }
  }
  return GPMA_OK;
}

gpma_status dist_cc(gpma *g, uint32_t *labels, cudaStream_t s) {
  Scratch &X = g->an[AN_CC];
  unsigned long long *chg = (unsigned long long *)&X.ctrl_d->sum;   // the round's change count (device)
  gpma_status st;
  for (int init = 1;; init = 0) {
    if ((st = cc_round(g, labels, init, nullptr, s))) return st;   // (no host read)
    if (g->nranks == 1) break;                      // one local round is the full answer
    NC_CHECK(g, nccl().AllReduce(labels, labels, g->V, ncclUint32, ncclMin, comm_of(g), s));
    NC_CHECK(g, nccl().AllReduce(chg, chg, 1, ncclUint64, ncclSum, comm_of(g), s));
    GP_CHECK(g, readback(g, &g->an[AN_CC].ctrl_h->sum, chg, 8, s));
    GP_CHECK(g, cudaStreamSynchronize(s));
    if (g->an[AN_CC].ctrl_h->sum == 0) break;
  }
  return GPMA_OK;
}

__global__ void k_dist_pr_slice(double *__restrict__ out, const double *__restrict__ x, uint32_t rb, uint32_t nr,
                                uint64_t chunk) {
  for (uint64_t i = blockIdx.x * (uint64_t)blockDim.x + threadIdx.x; i < chunk; i += (uint64_t)gridDim.x * blockDim.x)
    out[i] = i < nr ? x[rb + i] : 0.0;
}

gpma_status dist_pagerank(gpma *g, double *x, int warm, double d, double tol, int max_iter, int *iters,
                          cudaStream_t s) {
  const uint32_t P = (uint32_t)g->nranks, V = g->V;
  const uint64_t chunk = ((uint64_t)V + P - 1) / P;
  Scratch &X = g->an[AN_PR];
  GP_CHECK(g, ensure(g, X.stage[0], (chunk * P + 1) * 8 + (chunk + 1) * 8 + 16, s));
  GP_CHECK(g, ensure(g, X.stage[1], chunk * P * 8, s));
  uint64_t *y = (uint64_t *)X.stage[0].p;                 // [chunk*P + 1]: y[V] = dangling mass
  uint64_t *yr = y + chunk * P + 1;                        // [chunk + 1]: owned sums, dangling total
  double *err_d = (double *)(yr + chunk + 1);
  double *xs = (double *)X.stage[1].p;
  int it = 0;
  gpma_status st;
  GP_CHECK(g, fill_zero(g, y, (chunk * P + 1) * 8, s));
  while (it < max_iter) {
    if ((st = pr_push(g, x, (!warm) && it == 0, y, s))) return st;
    NC_CHECK(g, nccl().ReduceScatter(y, yr, chunk, ncclUint64, ncclSum, comm_of(g), s));
    NC_CHECK(g, nccl().AllReduce(y + V, yr + (g->nr), 1, ncclUint64, ncclSum, comm_of(g), s));
    if ((st = pr_update_rows(g, x, yr, d, nullptr, s))) return st;   // local error stays on the device
    NC_CHECK(g, nccl().AllReduce(&X.ctrl_d->sum2, err_d, 1, ncclFloat64, ncclSum, comm_of(g), s));
    GP_CHECK(g, fill_zero(g, y, (chunk * P + 1) * 8, s));
    GP_CHECK(g, readback(g, &X.ctrl_h->sum2, err_d, 8, s));
    GP_CHECK(g, cudaStreamSynchronize(s));
    double e;
    memcpy(&e, &X.ctrl_h->sum2, 8);
    ++it;
    if (e < tol) break;
  }
  // replicate x: the owned slices back to back (the last one padded to chunk)
  GP_LAUNCH(g, k_dist_pr_slice, grid_for(chunk), 256, 0, s, xs + (uint64_t)g->rank * chunk, x, g->rb, g->nr, chunk);
  NC_CHECK(g, nccl().AllGather(xs + (uint64_t)g->rank * chunk, xs, chunk, ncclFloat64, comm_of(g), s));
  GP_CHECK(g, cudaMemcpyAsync(x, xs, (uint64_t)V * 8, cudaMemcpyDeviceToDevice, s));
  GP_CHECK(g, cudaStreamSynchronize(s));
  if (iters) *iters = it;
  return GPMA_OK;
}

gpma_status dist_unique_id(void *out) {
  Nccl &N = nccl();
  if (!N.ok) return GPMA_ERR_CUDA;
  ncclUniqueId id;
  if (N.GetUniqueId(&id) != ncclSuccess) return GPMA_ERR_CUDA;
  memcpy(out, &id, sizeof id);
  return GPMA_OK;
}

// communicator of a new dist handle; then the initial slices go to their owners
gpma_status dist_attach(gpma *g, const void *id, int rank, int nranks) {
  Nccl &N = nccl();
  if (!N.ok) {
    set_err(g, N.why);
    return GPMA_ERR_CUDA;
  }
  ncclUniqueId uid;
  memcpy(&uid, id, sizeof uid);
  ncclComm_t c = nullptr;
  NC_CHECK(g, N.CommInitRank(&c, nranks, uid, rank));
  g->comm = c;
  g->rank = rank;
  g->nranks = nranks;
  return GPMA_OK;
}

gpma_status dist_create_store(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, uint64_t cap,
                              uint32_t leaf, cudaStream_t s) {
  uint64_t m = 0;
  gpma_status st = dist_exchange(g, keys, vals, n, true, &m, s);
  if (st) return st;
  return create_from_batch(g, (const uint64_t *)g->d_k[1].p, (const uint32_t *)g->d_v[1].p, m, cap, leaf, s);
}

void dist_detach(gpma *g) {
  if (g->comm && nccl().ok) nccl().CommDestroy(comm_of(g));
  g->comm = nullptr;
  for (DevBuf *b : {&g->d_k[0], &g->d_k[1], &g->d_v[0], &g->d_v[1], &g->d_misc}) release(g, *b, g->st);
}

}  // namespace gp
