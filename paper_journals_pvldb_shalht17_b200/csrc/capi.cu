// capi.cu -- the extern "C" boundary declared in include/gpma.h.
// Argument checking, host/device pointer staging and handle lifetime only; every step
// of the method runs in the kernels of update.cu / analytics.cu / primitives.cu.
#include <cuda_runtime.h>
#include <string.h>

#include <map>
#include <new>
#include <string>

#include "gpma_internal.cuh"

using gp::DevBuf;

namespace {

bool is_host_ptr(const void *p) {
  if (!p) return false;
  cudaPointerAttributes at;
  if (cudaPointerGetAttributes(&at, p) != cudaSuccess) {
    cudaGetLastError();
    return true;
  }
  return !(at.type == cudaMemoryTypeDevice || at.type == cudaMemoryTypeManaged);
}

// Output staging: kernels always write device memory; a host destination is filled
// by a D2H copy at the end of the call (which then synchronises the stream).
struct Out {
  gpma *g;
  void *user;
  size_t bytes;
  bool host;
  DevBuf buf;
  cudaStream_t s;
  Out(gpma *g_, void *u, size_t b, cudaStream_t s_) : g(g_), user(u), bytes(b), host(is_host_ptr(u)), s(s_) {}
  ~Out() { gp::release(g, buf, s); }
  cudaError_t dev(void **p, bool copy_in) {
    if (!user) { *p = nullptr; return cudaSuccess; }
    if (!host) { *p = user; return cudaSuccess; }
    cudaError_t e = gp::ensure(g, buf, bytes, s);
    if (e) return e;
    if (copy_in) {
      e = cudaMemcpyAsync(buf.p, user, bytes, cudaMemcpyHostToDevice, s);
      if (e) return e;
    }
    *p = buf.p;
    return cudaSuccess;
  }
  cudaError_t finish() {
    if (!user || !host) return cudaSuccess;
    cudaError_t e = cudaMemcpyAsync(user, buf.p, bytes, cudaMemcpyDeviceToHost, s);
    if (e) return e;
    return cudaStreamSynchronize(s);
  }
};

gpma_status begin(gpma *g) {
  if (!g) return GPMA_ERR_INVALID_ARG;
  if (g->poisoned) return GPMA_ERR_POISONED;
  {
    std::lock_guard<std::mutex> lk(g->mu);
    g->err.clear();
  }
  return GPMA_OK;
}

gpma_status end(gpma *g, gpma_status st) {
  if (st == GPMA_OK) {
    cudaError_t e = cudaGetLastError();
    if (e != cudaSuccess) return gp::cuda_fail(g, e, "kernel launch");
  }
  return st;
}

gpma_status apply_config(gpma *g, const gpma_config *cfg, uint32_t *leaf, uint64_t *cap) {
  gpma_config c;
  gpma_config_default(&c);
  if (cfg) {
    if (cfg->struct_size < sizeof(uint32_t) * 2) return GPMA_ERR_INVALID_ARG;
    size_t n = cfg->struct_size < sizeof(c) ? cfg->struct_size : sizeof(c);
    memcpy(&c, cfg, n);
  }
  if (c.leaf_slots && (c.leaf_slots < 4 || c.leaf_slots > 32 || (c.leaf_slots & (c.leaf_slots - 1))))
    return GPMA_ERR_INVALID_ARG;
  if (c.delete_mode > 1 || c.algorithm > 1) return GPMA_ERR_INVALID_ARG;
  g->algorithm = c.algorithm;
  if (c.rho_leaf_bp > 10000 || c.rho_root_bp > 10000 || c.tau_leaf_bp > 10000 || c.tau_root_bp > 10000 ||
      c.init_density_bp == 0 || c.init_density_bp > 10000)
    return GPMA_ERR_INVALID_ARG;
  g->rho0 = c.rho_leaf_bp;
  g->rhoh = c.rho_root_bp;
  g->tau0 = c.tau_leaf_bp;
  g->tauh = c.tau_root_bp;
  g->init_bp = c.init_density_bp;
  g->mode = c.delete_mode;
  if (c.row_end > c.row_begin) {
    if (c.row_end > g->V) return GPMA_ERR_INVALID_ARG;
    g->rb = c.row_begin;
    g->nr = c.row_end - c.row_begin;
  } else {
    g->rb = 0;
    g->nr = g->V;
  }
  if ((c.alloc == nullptr) != (c.free == nullptr)) return GPMA_ERR_INVALID_ARG;
  g->alloc_fn = c.alloc;
  g->free_fn = c.free;
  g->alloc_ctx = c.alloc_ctx;
  gp::pool_attach(g);
  *leaf = c.leaf_slots;
  *cap = c.initial_capacity;
  return GPMA_OK;
}

void free_handle(gpma *g);

gpma *new_handle(uint32_t V) {
  gpma *g = new (std::nothrow) gpma();
  if (!g) return nullptr;
  g->V = V;
  if (const char *e = getenv("GPMA_L2_FETCH")) {     // L2 fetch granularity (bytes) of the context
    cudaDeviceSetLimit(cudaLimitMaxL2FetchGranularity, (size_t)atoi(e));
    cudaGetLastError();
  }
  if (cudaMalloc((void **)&g->ctrl_d, sizeof(gp::Ctrl)) != cudaSuccess ||
      cudaMallocHost((void **)&g->ctrl_h, sizeof(gp::Ctrl)) != cudaSuccess ||
      cudaMallocHost(&g->pin, 256) != cudaSuccess) {
    cudaGetLastError();
    if (g->ctrl_d) cudaFree(g->ctrl_d);
    if (g->ctrl_h) cudaFreeHost(g->ctrl_h);
    delete g;
    return nullptr;
  }
  memset(g->ctrl_h, 0, sizeof(gp::Ctrl));
  if (cudaMemset(g->ctrl_d, 0, sizeof(gp::Ctrl)) != cudaSuccess) {   // (Ctrl::done starts at 0)
    cudaGetLastError();
    free_handle(g);
    return nullptr;
  }
  for (gp::Scratch &x : g->an) {
    if (cudaMalloc((void **)&x.ctrl_d, sizeof(gp::Ctrl)) != cudaSuccess ||
        cudaMallocHost((void **)&x.ctrl_h, sizeof(gp::Ctrl)) != cudaSuccess) {
      cudaGetLastError();
      free_handle(g);
      return nullptr;
    }
    memset(x.ctrl_h, 0, sizeof(gp::Ctrl));
  }
  return g;
}

void free_handle(gpma *g) {
  if (!g) return;
  // analytics may still run on other streams (include/gpma.h "Concurrency"): let all of the
  // device's work finish before the store and the scratch go back to the allocator
  cudaDeviceSynchronize();
  cudaGetLastError();
  cudaStream_t s = g->st;
  DevBuf *bufs[] = {&g->b_sk[0], &g->b_sk[1], &g->b_sv[0], &g->b_sv[1], &g->b_keep, &g->b_pos, &g->b_tgt,
                    &g->b_pk[0], &g->b_pk[1], &g->b_pv[0], &g->b_pv[1], &g->b_pt[0], &g->b_pt[1],
                    &g->b_hf, &g->b_widx, &g->b_wfirst, &g->b_acc, &g->b_aidx, &g->b_alist, &g->b_nw,
                    &g->b_woff, &g->b_keep2, &g->b_kpos, &g->b_lpre, &g->b_wk, &g->b_wv, &g->b_dirty,
                    &g->b_scan, &g->b_hist, &g->b_stage[0], &g->b_stage[1], &g->b_stage[2],
                    &g->b_stage[3], &g->b_misc, &g->b_misc2, &g->b_misc3, &g->b_sup};
  for (DevBuf *b : bufs) gp::release(g, *b, s);
  for (gp::Scratch &x : g->an) {
    DevBuf *xb[] = {&x.b[0], &x.b[1], &x.b[2], &x.b[3], &x.misc, &x.lpre, &x.scan, &x.stage[0], &x.stage[1]};
    for (DevBuf *b : xb) gp::release(g, *b, s);
  }
  gp::spare_release(g, s);
  gp::dev_free(g, g->key, s);
  gp::dev_free(g, g->val, s);
  gp::dev_free(g, g->cnt, s);
  gp::dev_free(g, g->head, s);
  gp::dev_free(g, g->row_offset, s);
  gp::dev_free(g, g->deg, s);
  cudaStreamSynchronize(s);
  gp::pool_detach(g);
  for (gp::UpdGraph &u : g->ugraph)
    if (u.exec) cudaGraphExecDestroy(u.exec);
  for (cudaEvent_t e : g->ev_pool) cudaEventDestroy(e);
  if (g->ctrl_d) cudaFree(g->ctrl_d);
  if (g->ctrl_h) cudaFreeHost(g->ctrl_h);
  if (g->pin) cudaFreeHost(g->pin);
  for (gp::Scratch &x : g->an) {
    if (x.ctrl_d) cudaFree(x.ctrl_d);
    if (x.ctrl_h) cudaFreeHost(x.ctrl_h);
  }
  cudaGetLastError();
  delete g;
}

}  // namespace

namespace gp {
gpma_status create_from_batch(gpma *g, const uint64_t *keys, const uint32_t *vals, uint64_t n,
                              uint64_t cap_override, uint32_t leaf_override, cudaStream_t s);
}

extern "C" {

void gpma_config_default(gpma_config *cfg) {
  if (!cfg) return;
  memset(cfg, 0, sizeof(*cfg));
  cfg->struct_size = sizeof(gpma_config);
  cfg->leaf_slots = 0;
  cfg->initial_capacity = 0;
  cfg->rho_leaf_bp = 800;
  cfg->rho_root_bp = 4000;
  cfg->tau_leaf_bp = 9200;
  cfg->tau_root_bp = 8000;
  cfg->init_density_bp = 6000;
  cfg->delete_mode = GPMA_DELETE_LAZY;
}

gpma_status gpma_create(uint32_t num_vertices, const uint64_t *init_keys, const uint32_t *init_vals,
                        uint64_t n_init, const gpma_config *cfg, gpma_stream_t stream, gpma_t **out) {
  if (!out || num_vertices == 0 || num_vertices == 0xFFFFFFFFu) return GPMA_ERR_INVALID_ARG;
  if (n_init && (!init_keys || !init_vals)) return GPMA_ERR_INVALID_ARG;
  *out = nullptr;
  gpma *g = new_handle(num_vertices);
  if (!g) return GPMA_ERR_OOM;
  cudaStream_t s = (cudaStream_t)stream;
  g->st = s;
  uint32_t leaf = 0;
  uint64_t cap = 0;
  gpma_status st = apply_config(g, cfg, &leaf, &cap);
  if (st == GPMA_OK && cap && (cap & (cap - 1))) st = GPMA_ERR_INVALID_ARG;
  if (st == GPMA_OK) st = gp::create_from_batch(g, init_keys, init_vals, n_init, cap, leaf, s);
  if (st == GPMA_OK) {
    cudaError_t e = cudaStreamSynchronize(s);
    if (e) st = gp::cuda_fail(g, e, "create");
  }
  if (st != GPMA_OK) {
    free_handle(g);
    return st;
  }
  *out = g;
  return GPMA_OK;
}

gpma_status gpma_dist_unique_id(void *id_out) {
  if (!id_out) return GPMA_ERR_INVALID_ARG;
  return gp::dist_unique_id(id_out);
}

gpma_status gpma_dist_create(const void *nccl_unique_id, int rank, int nranks, uint32_t num_vertices,
                             const uint64_t *init_keys, const uint32_t *init_vals, uint64_t n_init,
                             const gpma_config *cfg, gpma_stream_t stream, gpma_t **out) {
  if (!out || !nccl_unique_id || nranks < 1 || rank < 0 || rank >= nranks || num_vertices == 0 ||
      num_vertices == 0xFFFFFFFFu || (uint64_t)nranks > num_vertices)
    return GPMA_ERR_INVALID_ARG;
  if (n_init && (!init_keys || !init_vals)) return GPMA_ERR_INVALID_ARG;
  *out = nullptr;
  gpma *g = new_handle(num_vertices);
  if (!g) return GPMA_ERR_OOM;
  cudaStream_t s = (cudaStream_t)stream;
  g->st = s;
  gpma_config c;
  gpma_config_default(&c);
  if (cfg) {
    if (cfg->struct_size < sizeof(uint32_t) * 2) {
      free_handle(g);
      return GPMA_ERR_INVALID_ARG;
    }
    memcpy(&c, cfg, cfg->struct_size < sizeof(c) ? cfg->struct_size : sizeof(c));
  }
  gp::dist_rows(num_vertices, nranks, rank, &c.row_begin, &c.row_end);   // R24: this rank's rows
  uint32_t leaf = 0;
  uint64_t cap = 0;
  gpma_status st = apply_config(g, &c, &leaf, &cap);
  if (st == GPMA_OK && cap && (cap & (cap - 1))) st = GPMA_ERR_INVALID_ARG;
  if (st == GPMA_OK) st = gp::dist_attach(g, nccl_unique_id, rank, nranks);
  if (st == GPMA_OK) st = gp::dist_create_store(g, init_keys, init_vals, n_init, cap, leaf, s);
  if (st == GPMA_OK) {
    cudaError_t e = cudaStreamSynchronize(s);
    if (e) st = gp::cuda_fail(g, e, "dist_create");
  }
  if (st != GPMA_OK) {
    gp::dist_detach(g);
    free_handle(g);
    return st;
  }
  *out = g;
  return GPMA_OK;
}

gpma_status gpma_dist_info(const gpma_t *g, int *rank, int *nranks, uint32_t *row_begin, uint32_t *row_end) {
  if (!g) return GPMA_ERR_INVALID_ARG;
  if (rank) *rank = g->rank;
  if (nranks) *nranks = g->nranks;
  if (row_begin) *row_begin = g->rb;
  if (row_end) *row_end = g->rb + g->nr;
  return GPMA_OK;
}

gpma_status gpma_create_raw(uint32_t num_vertices, uint64_t capacity, uint32_t leaf_slots,
                            const uint64_t *keys, const uint32_t *vals, const gpma_config *cfg,
                            gpma_stream_t stream, gpma_t **out) {
  if (!out || !keys || !vals || num_vertices == 0) return GPMA_ERR_INVALID_ARG;
  if (leaf_slots < 4 || leaf_slots > 32 || (leaf_slots & (leaf_slots - 1))) return GPMA_ERR_INVALID_ARG;
  if (capacity < 2ull * leaf_slots || (capacity & (capacity - 1))) return GPMA_ERR_INVALID_ARG;
  *out = nullptr;
  gpma *g = new_handle(num_vertices);
  if (!g) return GPMA_ERR_OOM;
  cudaStream_t s = (cudaStream_t)stream;
  g->st = s;
  uint32_t leaf = 0;
  uint64_t cap = 0;
  gpma_status st = apply_config(g, cfg, &leaf, &cap);
  if (st == GPMA_OK) {
    g->L = leaf_slots;
    g->cap = capacity;
    g->h = gp::ilog2(capacity / leaf_slots);
    gp::level_bounds(g->L, g->h, g->rho0, g->rhoh, g->tau0, g->tauh, g->tmin, g->tmax);
    uint64_t nl = capacity / leaf_slots;
    if (gp::dev_alloc(g, (void **)&g->key, capacity * 8, s) || gp::dev_alloc(g, (void **)&g->val, capacity * 4, s) ||
        gp::dev_alloc(g, (void **)&g->cnt, nl * 12, s) || gp::dev_alloc(g, (void **)&g->head, nl * 8, s) ||
        gp::dev_alloc(g, (void **)&g->row_offset, ((uint64_t)g->nr + 1) * 8, s) ||
        gp::dev_alloc(g, (void **)&g->deg, (uint64_t)g->nr * 4 + 4, s)) {
      cudaGetLastError();
      st = GPMA_ERR_OOM;
    }
  }
  if (st == GPMA_OK) {
    gp::fill_zero(g, g->row_offset, ((uint64_t)g->nr + 1) * 8, s);
    st = gp::load_raw(g, keys, vals, s);
  }
  if (st == GPMA_OK && cudaStreamSynchronize(s) != cudaSuccess) st = GPMA_ERR_CUDA;
  if (st != GPMA_OK) {
    free_handle(g);
    return st;
  }
  *out = g;
  return GPMA_OK;
}

gpma_status gpma_destroy(gpma_t *g) {
  if (!g) return GPMA_ERR_INVALID_ARG;
  gp::dist_detach(g);
  free_handle(g);
  return GPMA_OK;
}

gpma_status gpma_update_batch(gpma_t *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, gpma_op op,
                              gpma_stream_t stream) {
  gp::Nvtx nvtx_("gpma_update_batch");
  gpma_status st = begin(g);
  if (st) return st;
  if (op != GPMA_INSERT && op != GPMA_DELETE) return GPMA_ERR_INVALID_ARG;
  if (n && !keys) return GPMA_ERR_INVALID_ARG;
  if (n && op == GPMA_INSERT && !vals) return GPMA_ERR_INVALID_ARG;
  if (n > 0xFFFFFFFFull) return GPMA_ERR_INVALID_ARG;
  g->st = (cudaStream_t)stream;
  st = end(g, g->comm ? gp::dist_update(g, keys, vals, n, (int)op, (cudaStream_t)stream)
                      : gp::update_batch(g, keys, vals, n, (int)op, (cudaStream_t)stream));
  if (st == GPMA_OK && n) {
    g->tot[0] += 1;
    g->tot[op == GPMA_INSERT ? 1 : 2] += n;
    g->tot[3] += g->last.last_slots_rewritten;
    g->tot[4] += g->last.last_windows_rewritten;
  }
  return st;
}

gpma_status gpma_bfs(gpma_t *g, uint32_t root, int32_t *levels, gpma_stream_t stream) {
  gp::Nvtx nvtx_("gpma_bfs");
  gpma_status st = begin(g);
  if (st) return st;
  if (!levels || root >= g->V) return GPMA_ERR_INVALID_ARG;
  cudaStream_t s = (cudaStream_t)stream;
  Out o(g, levels, (size_t)g->V * 4, s);
  void *d;
  if (cudaError_t e = o.dev(&d, false)) return gp::cuda_fail(g, e, "bfs staging");
  st = g->comm ? gp::dist_bfs(g, root, (int32_t *)d, s) : gp::bfs(g, root, (int32_t *)d, s);
  if (st == GPMA_OK)
    if (cudaError_t e = o.finish()) return gp::cuda_fail(g, e, "bfs copy-out");
  return end(g, st);
}

gpma_status gpma_cc(gpma_t *g, uint32_t *labels, gpma_stream_t stream) {
  gp::Nvtx nvtx_("gpma_cc");
  gpma_status st = begin(g);
  if (st) return st;
  if (!labels) return GPMA_ERR_INVALID_ARG;
  cudaStream_t s = (cudaStream_t)stream;
  Out o(g, labels, (size_t)g->V * 4, s);
  void *d;
  if (cudaError_t e = o.dev(&d, false)) return gp::cuda_fail(g, e, "cc staging");
  st = g->comm ? gp::dist_cc(g, (uint32_t *)d, s) : gp::cc(g, (uint32_t *)d, s);
  if (st == GPMA_OK)
    if (cudaError_t e = o.finish()) return gp::cuda_fail(g, e, "cc copy-out");
  return end(g, st);
}

gpma_status gpma_pagerank(gpma_t *g, double *rank, int warm_start, double damping, double tol_l1, int max_iter,
                          int *iters_out, gpma_stream_t stream) {
  gp::Nvtx nvtx_("gpma_pagerank");
  gpma_status st = begin(g);
  if (st) return st;
  if (!rank || max_iter < 0 || !(damping >= 0.0 && damping <= 1.0) || !(tol_l1 >= 0.0)) return GPMA_ERR_INVALID_ARG;
  if (g->nr != g->V && !g->comm) return GPMA_ERR_INVALID_ARG;   // a shard driven from outside: gpma_pr_push / _update
  cudaStream_t s = (cudaStream_t)stream;
  Out o(g, rank, (size_t)g->V * 8, s);
  void *d;
  if (cudaError_t e = o.dev(&d, warm_start != 0)) return gp::cuda_fail(g, e, "pagerank staging");
  st = g->comm ? gp::dist_pagerank(g, (double *)d, warm_start, damping, tol_l1, max_iter, iters_out, s)
               : gp::pagerank_f64(g, (double *)d, warm_start, damping, tol_l1, max_iter, iters_out, s);
  if (st == GPMA_OK)
    if (cudaError_t e = o.finish()) return gp::cuda_fail(g, e, "pagerank copy-out");
  return end(g, st);
}

gpma_status gpma_pagerank_f32(gpma_t *g, float *rank, int warm_start, float damping, float tol_l1, int max_iter,
                              int *iters_out, gpma_stream_t stream) {
  gp::Nvtx nvtx_("gpma_pagerank_f32");
  gpma_status st = begin(g);
  if (st) return st;
  if (g->comm) return GPMA_ERR_INVALID_ARG;
  if (!rank || max_iter < 0 || !(damping >= 0.0f && damping <= 1.0f) || !(tol_l1 >= 0.0f)) return GPMA_ERR_INVALID_ARG;
  if (g->nr != g->V) return GPMA_ERR_INVALID_ARG;
  cudaStream_t s = (cudaStream_t)stream;
  Out o(g, rank, (size_t)g->V * 4, s);
  void *d;
  if (cudaError_t e = o.dev(&d, warm_start != 0)) return gp::cuda_fail(g, e, "pagerank staging");
  st = gp::pagerank_f32(g, (float *)d, warm_start, damping, tol_l1, max_iter, iters_out, s);
  if (st == GPMA_OK)
    if (cudaError_t e = o.finish()) return gp::cuda_fail(g, e, "pagerank copy-out");
  return end(g, st);
}

gpma_status gpma_export_csr(gpma_t *g, uint64_t *row_ptr, uint32_t *col, uint32_t *val, uint64_t nnz_capacity,
                            uint64_t *nnz_out, gpma_stream_t stream) {
  gp::Nvtx nvtx_("gpma_export_csr");
  gpma_status st = begin(g);
  if (st) return st;
  if (col && (!row_ptr || !val)) return GPMA_ERR_INVALID_ARG;
  cudaStream_t s = (cudaStream_t)stream;
  uint64_t nnz = 0;
  if (!col) {
    st = gp::export_csr(g, nullptr, nullptr, nullptr, 0, &nnz, s);
    if (nnz_out) *nnz_out = nnz;
    return end(g, st);
  }
  Out orp(g, row_ptr, ((size_t)g->nr + 1) * 8, s), oc(g, col, (size_t)nnz_capacity * 4, s),
      ov(g, val, (size_t)nnz_capacity * 4, s);
  void *drp, *dc, *dv;
  if (cudaError_t e = orp.dev(&drp, false)) return gp::cuda_fail(g, e, "export staging");
  if (cudaError_t e = oc.dev(&dc, false)) return gp::cuda_fail(g, e, "export staging");
  if (cudaError_t e = ov.dev(&dv, false)) return gp::cuda_fail(g, e, "export staging");
  st = gp::export_csr(g, (uint64_t *)drp, (uint32_t *)dc, (uint32_t *)dv, nnz_capacity, &nnz, s);
  if (nnz_out) *nnz_out = nnz;
  if (st == GPMA_OK) {
    oc.bytes = (size_t)nnz * 4;
    ov.bytes = (size_t)nnz * 4;
    cudaError_t e;
    if ((e = orp.finish()) || (e = oc.finish()) || (e = ov.finish())) return gp::cuda_fail(g, e, "export copy-out");
  }
  return end(g, st);
}

gpma_status gpma_stats(gpma_t *g, gpma_stats_t *out) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!out) return GPMA_ERR_INVALID_ARG;
  *out = g->last;
  out->num_vertices = g->V;
  out->leaf_slots = g->L;
  out->capacity = g->cap;
  out->height = g->h;
  out->delete_mode = g->mode;
  out->resizes = g->resizes;
  out->total_batches = g->tot[0];
  out->total_insert_keys = g->tot[1];
  out->total_delete_keys = g->tot[2];
  out->total_slots_rewritten = g->tot[3];
  out->total_windows_rewritten = g->tot[4];
  st = gp::count_slots(g, &out->live_edges, &out->tombstones, g->st);
  return end(g, st);
}

gpma_status gpma_stats_host(const gpma_t *g, gpma_stats_t *out) {
  if (!g || !out) return GPMA_ERR_INVALID_ARG;
  *out = g->last;
  out->num_vertices = g->V;
  out->leaf_slots = g->L;
  out->capacity = g->cap;
  out->height = g->h;
  out->delete_mode = g->mode;
  out->resizes = g->resizes;
  out->total_batches = g->tot[0];
  out->total_insert_keys = g->tot[1];
  out->total_delete_keys = g->tot[2];
  out->total_slots_rewritten = g->tot[3];
  out->total_windows_rewritten = g->tot[4];
  out->live_edges = ~0ull;
  out->tombstones = ~0ull;
  return GPMA_OK;
}

gpma_status gpma_debug_dump(gpma_t *g, uint64_t *keys, uint32_t *vals, uint64_t *row_offset, uint32_t *leaf_live,
                            uint64_t *heads, gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  cudaStream_t s = (cudaStream_t)stream;
  uint64_t nl = g->cap / g->L;
  struct { void *dst; const void *src; size_t bytes; } cp[] = {
      {keys, g->key, g->cap * 8}, {vals, g->val, g->cap * 4}, {row_offset, g->row_offset, ((size_t)g->nr + 1) * 8},
      {leaf_live, g->cnt, nl * 4}, {heads, g->head, nl * 8}};
  for (auto &c : cp)
    if (c.dst)
      if (cudaError_t e = cudaMemcpyAsync(c.dst, c.src, c.bytes, cudaMemcpyDefault, s))
        return gp::cuda_fail(g, e, "debug_dump");
  if (cudaError_t e = cudaStreamSynchronize(s)) return gp::cuda_fail(g, e, "debug_dump");
  return GPMA_OK;
}

gpma_status gpma_debug_dump_aux(gpma_t *g, uint32_t *tomb_mask, uint32_t *leaf_guards, uint32_t *out_degree,
                                gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  cudaStream_t s = (cudaStream_t)stream;
  uint64_t nl = g->cap / g->L;
  struct { void *dst; const void *src; size_t bytes; } cp[] = {
      {tomb_mask, gp::tmask_of(g), nl * 4}, {leaf_guards, gp::gcnt_of(g), nl * 4}, {out_degree, g->deg, (size_t)g->nr * 4}};
  for (auto &c : cp)
    if (c.dst)
      if (cudaError_t e = cudaMemcpyAsync(c.dst, c.src, c.bytes, cudaMemcpyDefault, s))
        return gp::cuda_fail(g, e, "debug_dump_aux");
  if (cudaError_t e = cudaStreamSynchronize(s)) return gp::cuda_fail(g, e, "debug_dump_aux");
  return GPMA_OK;
}

gpma_status gpma_debug_set_trace(gpma_t *g, int enable) {
  if (!g) return GPMA_ERR_INVALID_ARG;
  g->trace_on = enable != 0;
  return GPMA_OK;
}

gpma_status gpma_debug_trace(gpma_t *g, uint64_t *out4, uint64_t max, uint64_t *count) {
  if (!g || !count) return GPMA_ERR_INVALID_ARG;
  uint64_t n = g->trace.size() / 4;
  *count = n;
  if (out4) memcpy(out4, g->trace.data(), (n < max ? n : max) * 4 * sizeof(uint64_t));
  return GPMA_OK;
}

gpma_status gpma_debug_profile(gpma_t *g, const char *kernel_filter) {
  if (!g) return GPMA_ERR_INVALID_ARG;
  g->prof_filter = kernel_filter ? kernel_filter : "";
  g->prof_recs.clear();
  g->ev_used = 0;
  return GPMA_OK;
}

gpma_status gpma_debug_profile_read(gpma_t *g, char *buf, size_t buflen) {
  if (!g || !buf || !buflen) return GPMA_ERR_INVALID_ARG;
  if (cudaError_t e = cudaDeviceSynchronize()) return gp::cuda_fail(g, e, "profile_read");
  std::map<std::string, std::pair<uint64_t, double>> agg;
  for (auto &r : g->prof_recs) {
    float ms = 0.f;
    cudaEventElapsedTime(&ms, g->ev_pool[r.e0], g->ev_pool[r.e1]);
    std::string nm(r.name);
    size_t lt = nm.find('<');
    if (lt != std::string::npos) nm = nm.substr(0, lt);
    auto &a = agg[nm];
    a.first += 1;
    a.second += ms;
  }
  std::string out;
  char line[256];
  for (auto &kv : agg) {
    snprintf(line, sizeof line, "%s\t%llu\t%.6f\n", kv.first.c_str(), (unsigned long long)kv.second.first,
             kv.second.second);
    out += line;
  }
  size_t n = out.size() < buflen - 1 ? out.size() : buflen - 1;
  memcpy(buf, out.data(), n);
  buf[n] = 0;
  g->prof_recs.clear();
  g->ev_used = 0;
  return GPMA_OK;
}

// ---- query buffer
gpma_status gpma_query_edges(gpma_t *g, const uint64_t *keys, uint64_t n, uint32_t *vals, uint8_t *found,
                             gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (n && !keys) return GPMA_ERR_INVALID_ARG;
  cudaStream_t s = (cudaStream_t)stream;
  Out ov(g, vals, (size_t)n * 4, s), of(g, found, (size_t)n, s);
  void *dv, *df;
  if (cudaError_t e = ov.dev(&dv, false)) return gp::cuda_fail(g, e, "query staging");
  if (cudaError_t e = of.dev(&df, false)) return gp::cuda_fail(g, e, "query staging");
  st = gp::query_edges(g, keys, n, (uint32_t *)dv, (uint8_t *)df, s);
  if (st == GPMA_OK) {
    cudaError_t e;
    if ((e = ov.finish()) || (e = of.finish())) return gp::cuda_fail(g, e, "query copy-out");
  }
  return end(g, st);
}

gpma_status gpma_query_neighbors(gpma_t *g, const uint32_t *verts, uint64_t n, uint64_t *row_ptr, uint32_t *col,
                                 uint32_t *val, uint64_t nnz_capacity, uint64_t *nnz_out, gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if ((n && !verts) || (col && !row_ptr)) return GPMA_ERR_INVALID_ARG;
  cudaStream_t s = (cudaStream_t)stream;
  uint64_t nnz = 0;
  if (!col) {
    st = gp::query_neighbors(g, verts, n, nullptr, nullptr, nullptr, 0, &nnz, s);
    if (nnz_out) *nnz_out = nnz;
    return end(g, st);
  }
  Out orp(g, row_ptr, ((size_t)n + 1) * 8, s), oc(g, col, (size_t)nnz_capacity * 4, s),
      ov(g, val, (size_t)nnz_capacity * 4, s);
  void *drp, *dc, *dv;
  if (cudaError_t e = orp.dev(&drp, false)) return gp::cuda_fail(g, e, "query staging");
  if (cudaError_t e = oc.dev(&dc, false)) return gp::cuda_fail(g, e, "query staging");
  if (cudaError_t e = ov.dev(&dv, false)) return gp::cuda_fail(g, e, "query staging");
  st = gp::query_neighbors(g, verts, n, (uint64_t *)drp, (uint32_t *)dc, (uint32_t *)dv, nnz_capacity, &nnz, s);
  if (nnz_out) *nnz_out = nnz;
  if (st == GPMA_OK) {
    oc.bytes = (size_t)nnz * 4;
    ov.bytes = (size_t)nnz * 4;
    cudaError_t e;
    if ((e = orp.finish()) || (e = oc.finish()) || (e = ov.finish())) return gp::cuda_fail(g, e, "query copy-out");
  }
  return end(g, st);
}

gpma_status gpma_query_reachable(gpma_t *g, const uint32_t *src, const uint32_t *dst, uint64_t n, uint8_t *reachable,
                                 gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (n && (!src || !dst || !reachable)) return GPMA_ERR_INVALID_ARG;
  if (g->nr != g->V) return GPMA_ERR_INVALID_ARG;
  cudaStream_t s = (cudaStream_t)stream;
  Out o(g, reachable, (size_t)n, s);
  void *d;
  if (cudaError_t e = o.dev(&d, false)) return gp::cuda_fail(g, e, "query staging");
  st = gp::query_reachable(g, src, dst, n, (uint8_t *)d, s);
  if (st == GPMA_OK)
    if (cudaError_t e = o.finish()) return gp::cuda_fail(g, e, "query copy-out");
  return end(g, st);
}

// ---- sharded-store primitives (device pointers)
gpma_status gpma_route(gpma_t *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, uint32_t nranks,
                       uint64_t *out_keys, uint32_t *out_vals, uint64_t *counts, gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if ((n && (!keys || !out_keys || !out_vals)) || !counts || nranks == 0 || nranks > 256)
    return GPMA_ERR_INVALID_ARG;
  return end(g, gp::route(g, keys, vals, n, nranks, out_keys, out_vals, counts, (cudaStream_t)stream));
}

gpma_status gpma_bfs_init(gpma_t *g, uint32_t root, int32_t *levels, gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!levels || root >= g->V) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::bfs_init(g, root, levels, (cudaStream_t)stream));
}

gpma_status gpma_bfs_level(gpma_t *g, int32_t *levels, int32_t depth, uint32_t *frontier_size,
                           gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!levels || !frontier_size || depth < 1) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::bfs_level(g, levels, depth, frontier_size, (cudaStream_t)stream));
}

gpma_status gpma_cc_round(gpma_t *g, uint32_t *labels, int init, uint64_t *changed, gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!labels || !changed) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::cc_round(g, labels, init, changed, (cudaStream_t)stream));
}

gpma_status gpma_pr_push(gpma_t *g, double *x, int init, uint64_t *y, gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!x || !y) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::pr_push(g, x, init, y, (cudaStream_t)stream));
}

gpma_status gpma_pr_update(gpma_t *g, double *x, uint64_t *y, double damping, double *err,
                           gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!x || !y || !err || !(damping >= 0.0 && damping <= 1.0)) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::pr_update(g, x, y, damping, err, (cudaStream_t)stream));
}

gpma_status gpma_pr_update_rows(gpma_t *g, double *x, const uint64_t *y_rows, double damping, double *err,
                                gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!x || !y_rows || !err || !(damping >= 0.0 && damping <= 1.0)) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::pr_update_rows(g, x, y_rows, damping, err, (cudaStream_t)stream));
}

gpma_status gpma_pr_update_rows_dev(gpma_t *g, double *x, const uint64_t *y_rows, double damping, double *err_dev,
                                    gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!x || !y_rows || !err_dev || !(damping >= 0.0 && damping <= 1.0)) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::pr_update_rows_dev(g, x, y_rows, damping, err_dev, (cudaStream_t)stream));
}

gpma_status gpma_validate_batch(gpma_t *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, gpma_op op,
                                gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (op != GPMA_INSERT && op != GPMA_DELETE) return GPMA_ERR_INVALID_ARG;
  if (n && !keys) return GPMA_ERR_INVALID_ARG;
  if (!n) return GPMA_OK;
  cudaStream_t s = (cudaStream_t)stream;
  gp::DevBuf kb, vb;
  const uint64_t *kd = keys;
  const uint32_t *vd = op == GPMA_INSERT ? vals : nullptr;
  // host slices are staged (the kernel reads device memory)
  if (is_host_ptr(keys)) {
    if (cudaError_t e = gp::ensure(g, kb, n * 8, s)) return gp::cuda_fail(g, e, "validate staging");
    if (cudaError_t e = gp::stage_in(g, kb.p, keys, n * 8, s)) return gp::cuda_fail(g, e, "validate staging");
    kd = (const uint64_t *)kb.p;
  }
  if (vd && is_host_ptr(vd)) {
    if (cudaError_t e = gp::ensure(g, vb, n * 4, s)) return gp::cuda_fail(g, e, "validate staging");
    if (cudaError_t e = gp::stage_in(g, vb.p, vd, n * 4, s)) return gp::cuda_fail(g, e, "validate staging");
    vd = (const uint32_t *)vb.p;
  }
  st = gp::validate_slice(g, kd, vd, n, vd != nullptr, s);
  if (st == GPMA_OK) {
    if (cudaError_t e = gp::readback(g, g->ctrl_h, g->ctrl_d, sizeof(gp::Ctrl), s)) st = gp::cuda_fail(g, e, "validate");
    else if (cudaError_t e2 = cudaStreamSynchronize(s)) st = gp::cuda_fail(g, e2, "validate");
  }
  gp::release(g, kb, s);
  gp::release(g, vb, s);
  if (st) return end(g, st);
  if (g->ctrl_h->err & 2u) return GPMA_ERR_RESERVED;
  if (g->ctrl_h->err & 1u) return GPMA_ERR_RANGE;
  return end(g, GPMA_OK);
}

gpma_status gpma_bfs_bits(gpma_t *g, const int32_t *levels, int32_t depth, uint32_t *bitmap, gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!levels || !bitmap) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::bfs_bits(g, levels, depth, bitmap, (cudaStream_t)stream));
}

gpma_status gpma_bfs_merge(gpma_t *g, int32_t *levels, const uint32_t *bitmaps, uint32_t nbitmaps, int32_t depth,
                           gpma_stream_t stream) {
  gpma_status st = begin(g);
  if (st) return st;
  if (!levels || (nbitmaps && !bitmaps) || depth < 1) return GPMA_ERR_INVALID_ARG;
  return end(g, gp::bfs_merge(g, levels, bitmaps, nbitmaps, depth, (cudaStream_t)stream));
}

uint64_t gpma_kernel_launches(const gpma_t *g) { return g ? g->launches.load() : 0; }

const char *gpma_status_string(gpma_status s) {
  switch (s) {
    case GPMA_OK: return "ok";
    case GPMA_ERR_INVALID_ARG: return "invalid argument";
    case GPMA_ERR_RANGE: return "vertex id out of range";
    case GPMA_ERR_RESERVED: return "reserved key or value";
    case GPMA_ERR_OOM: return "out of device memory";
    case GPMA_ERR_CUDA: return "CUDA error";
    case GPMA_ERR_POISONED: return "handle poisoned by an earlier CUDA error";
  }
  return "unknown";
}

const char *gpma_last_error(const gpma_t *g) { return g ? g->err.c_str() : "null handle"; }

}  // extern "C"
