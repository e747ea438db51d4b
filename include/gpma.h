/*
 * gpma.h -- C ABI of the B200-native GPMA+ dynamic-graph store.
 *
 * The method is GPMA+ of Sha, Li, He, Tan, "Accelerating Dynamic Graph Analytics on
 * GPUs", PVLDB 11(1), 2017 (cited as P:<line> of /root/reference/PAPER.md; R<n> are
 * the readings listed in DESIGN.md / SURVEY.md §8(c)).
 *
 * Store: a packed memory array (PMA, §4.1) of edge keys (src<<32 | dst) with
 * a u32 value, split into leaf segments of L slots; one guard entry (u, 0xFFFFFFFF)
 * per vertex u marks the end of row u so that row_offset[u+1] = slot(guard u) turns
 * the gapped array into a CSR (CSR on GPMA, §4.2, Fig. 5).
 *
 * Conventions for every entry point
 *   - Pointers to arrays may be DEVICE pointers (cudaMalloc / torch CUDA tensors) or
 *     HOST pointers (pinned or pageable); the library detects the kind with
 *     cudaPointerGetAttributes and stages host buffers through its own device memory
 *     on the given stream.  The library never retains a caller pointer past the call.
 *   - Calls are stream-ordered on `stream` (NULL = legacy default stream).  With device
 *     outputs the caller may read them after synchronising the stream; with host
 *     outputs the call synchronises the stream before returning.
 *   - The library owns all store memory (cudaMallocAsync on the call's stream).
 *   - Every function returns a gpma_status.  Argument, range and reserved-value
 *     errors are detected before anything is mutated (no partial batch).  A CUDA
 *     error poisons the handle; later calls return GPMA_ERR_POISONED.
 *   - Concurrency.  Calls that mutate the store (create, update_batch, destroy) are
 *     exclusive: nothing else may run on the handle meanwhile.  The read-only analytics
 *     BFS (gpma_bfs, gpma_bfs_init/level), CC (gpma_cc, gpma_cc_round), PageRank
 *     (gpma_pagerank*, gpma_pr_push/update), export (gpma_export_csr) and the query buffer
 *     (gpma_query_*) each own a private scratch + control block, so DIFFERENT analytics
 *     may run at the same time from different host threads, each on its own stream
 *     (the caller orders those streams after the last update and before the next one).
 *     Two calls of the SAME analytic on one handle must not overlap.
 *   - All compute runs in the sm_100a kernels of this library; there is no CPU path.
 */
#ifndef GPMA_H
#define GPMA_H

#include <stddef.h>
#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

struct CUstream_st;                       /* cudaStream_t == struct CUstream_st* */
typedef struct CUstream_st *gpma_stream_t;
typedef struct gpma gpma_t;               /* opaque: one store (or one shard)     */

typedef enum {
  GPMA_OK = 0,
  GPMA_ERR_INVALID_ARG = 1, /* NULL handle/pointer, bad op, bad config             */
  GPMA_ERR_RANGE = 2,       /* a src or dst >= num_vertices (R23)                   */
  GPMA_ERR_RESERVED = 3,    /* dst == 0xFFFFFFFF (guard column, R1) or
                               val == 0xFFFFFFFF (tombstone, R12)                   */
  GPMA_ERR_OOM = 4,         /* device allocation failed                             */
  GPMA_ERR_CUDA = 5,        /* a CUDA call failed; the handle is now poisoned       */
  GPMA_ERR_POISONED = 6     /* an earlier CUDA error poisoned this handle           */
} gpma_status;

typedef enum { GPMA_INSERT = 0, GPMA_DELETE = 1 } gpma_op;

/* R12: deletions are either lazy (the paper's sliding-window mode: mark
 * the slot deleted, no density maintenance, recycled by later rewrites) or the dual of
 * insertion (lower-bound test per level, root halving). */
typedef enum { GPMA_DELETE_LAZY = 0, GPMA_DELETE_REBALANCE = 1 } gpma_delete_mode;

typedef struct {
  uint32_t struct_size;       /* sizeof(gpma_config)                                  */
  uint32_t leaf_slots;        /* L; 0 = R3 rule max(4, 2^floor(log2 log2 cap0)).
                                 Must be a power of two in [4, 32].                   */
  uint64_t initial_capacity;  /* 0 = R15 rule (smallest 2^k >= 8 holding E0+V at
                                 init_density_bp); else a power of two >= 2L          */
  uint16_t rho_leaf_bp, rho_root_bp, tau_leaf_bp, tau_root_bp; /* R4, basis points:
                                 800, 4000, 9200, 8000 = Fig. 3           */
  uint16_t init_density_bp;   /* R15: 6000                                            */
  uint16_t algorithm;         /* insertion: 0 = GPMA+ segment-oriented (Alg. 4, default);
                                 1 = GPMA lock-based (Alg. 1) with deterministic
                                 lock arbitration (R28: the contender from the highest
                                 child segment wins, then the smallest key; Ex. 2)      */
  uint32_t delete_mode;       /* gpma_delete_mode                                     */
  uint32_t row_begin, row_end;/* shard (R24): the store holds the rows
                                 (sources) [row_begin, row_end) only -- guards, row
                                 offsets and out-degrees for those rows; destinations
                                 range over [0, num_vertices).  0,0 = all rows.       */
  /* Device memory of the store and of every scratch buffer (SURVEY §8(b) "Ownership"):
   * alloc(bytes, stream, ctx) returns device memory usable in stream order on `stream`
   * (NULL = out of memory -> GPMA_ERR_OOM); free(ptr, stream, ctx) releases it in stream
   * order.  Both NULL (default) = a stream-ordered pool owned by the library (one per
   * device, trimmed when the device's last handle is destroyed).  Set both or neither; the
   * hooks must stay valid until gpma_destroy returns.  Added in the second version of this
   * struct: callers compiled against the first (smaller struct_size) get the default.    */
  void *(*alloc)(size_t bytes, gpma_stream_t stream, void *ctx);
  void (*free)(void *ptr, gpma_stream_t stream, void *ctx);
  void *alloc_ctx;
} gpma_config;

typedef struct {
  uint32_t num_vertices;
  uint32_t leaf_slots;        /* L                                                    */
  uint64_t capacity;          /* slots (power of two)                                 */
  uint32_t height;            /* h: capacity = L * 2^h                                */
  uint32_t delete_mode;
  uint64_t live_edges;        /* live entries excluding guards                        */
  uint64_t tombstones;        /* lazily deleted entries still occupying slots         */
  uint64_t resizes;           /* root doublings + halvings since create               */
  /* last gpma_update_batch: */
  uint64_t last_unique;       /* distinct keys in the batch                           */
  uint64_t last_pending;      /* updates entering the level loop after the pre-pass   */
  uint64_t last_slots_rewritten;   /* sum of |W| over re-dispatched windows (+ resize) */
  uint64_t last_windows_rewritten;
  uint32_t last_top_level;    /* highest level reached (h+1 = resized)                */
  uint32_t last_resized;
  uint64_t last_rounds;       /* GPMA (algorithm 1): retry rounds of the last insert    */
  uint64_t last_level0_windows;    /* leaves rewritten at level 0 by the last batch        */
  /* cumulative since create (measurement: SURVEY §8(d) algorithmic bytes per slide) */
  uint64_t total_batches;     /* non-empty update batches accepted                     */
  uint64_t total_insert_keys; /* keys of insert batches (as passed, duplicates included) */
  uint64_t total_delete_keys; /* keys of delete batches                                */
  uint64_t total_slots_rewritten;   /* sum of last_slots_rewritten                       */
  uint64_t total_windows_rewritten;
  uint64_t last_pending_level1;    /* updates the leaves rejected (climbing to level 1)   */
  uint64_t last_levels_skipped;    /* levels a root-bound climb passed over (no window there
                                      could accept: dead-level skip)           */
  uint64_t last_big_head_windows;  /* rewritten windows of >= 2048 leaves whose locate heads
                                      were fixed up CTA-parallel              */
} gpma_stats_t;

/* Fill *cfg with the defaults above. */
void gpma_config_default(gpma_config *cfg);

/* Build a store over vertices [0, num_vertices) from n_init edges (keys u64[n_init],
 * vals u32[n_init]; may repeat, the last occurrence wins, R10).  Inserts the V guards
 * (R1), picks capacity (R15) and leaf size (R3), lays everything out evenly (R7).
 * cfg may be NULL (defaults).  On success *out owns the store. */
gpma_status gpma_create(uint32_t num_vertices, const uint64_t *init_keys,
                        const uint32_t *init_vals, uint64_t n_init, const gpma_config *cfg,
                        gpma_stream_t stream, gpma_t **out);

/* Test hook: load a raw slot layout keys u64[capacity], vals u32[capacity] (e.g. the
 * Fig. 3 PMA) with leaf size leaf_slots; guards are optional.  The layout must
 * be sorted over occupied slots and left-packed per leaf. */
gpma_status gpma_create_raw(uint32_t num_vertices, uint64_t capacity, uint32_t leaf_slots,
                            const uint64_t *keys, const uint32_t *vals, const gpma_config *cfg,
                            gpma_stream_t stream, gpma_t **out);

gpma_status gpma_destroy(gpma_t *g);

/* Apply one homogeneous batch (Alg. 4): keys u64[n] (src<<32|dst), vals
 * u32[n] (ignored and may be NULL for GPMA_DELETE).  Keys may be unsorted and repeat
 * (last occurrence wins).  INSERT of a live key overwrites its value; of a tombstoned
 * key revives it in place (R11, R12).  DELETE of an absent key is a no-op (R13).
 * n == 0 is a no-op.  Errors: RANGE / RESERVED before any mutation. */
gpma_status gpma_update_batch(gpma_t *g, const uint64_t *keys, const uint32_t *vals, uint64_t n,
                              gpma_op op, gpma_stream_t stream);

/* BFS from root over the live out-edges (Alg. 2-3):
 * levels i32[V] = hop distance, -1 if unreachable. */
gpma_status gpma_bfs(gpma_t *g, uint32_t root, int32_t *levels, gpma_stream_t stream);

/* Weakly connected components (R19): labels u32[V] = the minimum vertex
 * id of each vertex's component. */
gpma_status gpma_cc(gpma_t *g, uint32_t *labels, gpma_stream_t stream);

/* PageRank by power iteration (R20/R21):
 *   x'[v] = (1-d)/V + d * (sum_{u->v} x[u]/outdeg(u) + D/V),  D = sum of dangling x[u];
 * stops after the first iteration with ||x'-x||_1 < tol_l1 (tol 0 = exactly max_iter
 * iterations).  rank f64[V]: input when warm_start != 0, else
 * initialised to 1/V; output = the last x'.  *iters_out (may be NULL) = iterations. */
gpma_status gpma_pagerank(gpma_t *g, double *rank, int warm_start, double damping,
                          double tol_l1, int max_iter, int *iters_out, gpma_stream_t stream);
/* Same in fp32 (accumulation in fp32). */
gpma_status gpma_pagerank_f32(gpma_t *g, float *rank, int warm_start, float damping,
                              float tol_l1, int max_iter, int *iters_out, gpma_stream_t stream);

/* CSR view (Fig. 5): row_ptr u64[V+1], col u32[nnz], val u32[nnz]
 * of the live edges in key order.  col == NULL: only *nnz_out is computed (size
 * query).  nnz_capacity < nnz -> GPMA_ERR_INVALID_ARG with *nnz_out set. */
gpma_status gpma_export_csr(gpma_t *g, uint64_t *row_ptr, uint32_t *col, uint32_t *val,
                            uint64_t nnz_capacity, uint64_t *nnz_out, gpma_stream_t stream);

gpma_status gpma_stats(gpma_t *g, gpma_stats_t *out);
/* The same without any device work (no synchronisation): live_edges and tombstones are set to
 * UINT64_MAX (not counted); everything else as gpma_stats.  For per-batch logging. */
gpma_status gpma_stats_host(const gpma_t *g, gpma_stats_t *out);

/* Parity hooks.  Raw layout: keys u64[capacity] (0xFFFF..FF = empty), vals
 * u32[capacity] (0 on empty slots); row_offset u64[V+1] (R8); leaf_live u32[cap/L]
 * (live entries incl. guards per leaf); heads u64[cap/L] (locate index, R9).  Any
 * output pointer may be NULL. */
gpma_status gpma_debug_dump(gpma_t *g, uint64_t *keys, uint32_t *vals, uint64_t *row_offset,
                            uint32_t *leaf_live, uint64_t *heads, gpma_stream_t stream);

/* The maintained per-leaf / per-row summaries the analytics read instead of the slots:
 * tomb_mask u32[cap/L] (bit p = slot p of the leaf holds a tombstone, R12), leaf_guards
 * u32[cap/L] (guards per leaf, R1), out_degree u32[row_end-row_begin] (live out-edges per
 * owned row, PageRank's outdeg, R21).  Any output pointer may be NULL. */
gpma_status gpma_debug_dump_aux(gpma_t *g, uint32_t *tomb_mask, uint32_t *leaf_guards, uint32_t *out_degree,
                                gpma_stream_t stream);

/* Per-level trace of the following update batches (Fig. 6 "Update Segments /
 * Offsets / Successful Flag"), off by default (it adds host syncs). */
gpma_status gpma_debug_set_trace(gpma_t *g, int enable);
/* Records (level, seg_start_slot, offset, flag) x4 u64; flag 2 closes a level and
 * carries the final offset.  Returns the record count in *count; copies at most max. */
gpma_status gpma_debug_trace(gpma_t *g, uint64_t *out4, uint64_t max, uint64_t *count);

/* ---------------------------------------------------------------- query buffer
 * Batched ad-hoc queries on the live store (the dynamic query buffer, §3). */

/* Edge lookup: keys u64[n] -> vals u32[n] (0xFFFFFFFF if absent or deleted) and found u8[n]
 * (either output may be NULL). */
gpma_status gpma_query_edges(gpma_t *g, const uint64_t *keys, uint64_t n, uint32_t *vals, uint8_t *found,
                             gpma_stream_t stream);
/* Neighbourhoods: the live out-edges of verts u32[n] as a CSR -- row_ptr u64[n+1],
 * col u32[nnz], val u32[nnz] (val may be NULL), rows in query order, columns in key order.
 * col == NULL: only *nnz_out (size query).  Not available on sharded stores for rows they
 * do not own (those rows come back empty). */
gpma_status gpma_query_neighbors(gpma_t *g, const uint32_t *verts, uint64_t n, uint64_t *row_ptr, uint32_t *col,
                                 uint32_t *val, uint64_t nnz_capacity, uint64_t *nnz_out, gpma_stream_t stream);
/* Reachability of pairs: reachable u8[n] = 1 iff a directed path src[i] -> dst[i] exists over the
 * live edges ("check the dynamic reachability between pairs of vertices"); a
 * multi-source BFS answers 64 pairs per sweep.  Unsharded stores only. */
gpma_status gpma_query_reachable(gpma_t *g, const uint32_t *src, const uint32_t *dst, uint64_t n,
                                 uint8_t *reachable, gpma_stream_t stream);

/* ---------------------------------------------------------------- multi-GPU handle
 * SURVEY §8(b)/(e); §6.4: "We evenly partition graphs according to the vertex index
 * and synchronize all devices after each iteration".  One process per GPU, one
 * handle per rank; the library owns an NCCL communicator (loaded at run time: the process's
 * libnccl.so.2, or GPMA_NCCL_LIB) and runs every exchange itself on the call's stream.
 * Rank r's store holds the source rows [r*ceil(V/P), min(V, (r+1)*ceil(V/P))) (R24).
 *
 * On a handle made by gpma_dist_create, every call below is COLLECTIVE (all ranks, same order):
 *   gpma_update_batch(keys, vals, n): the rank's slice (any n >= 0, host or device) of a global
 *     batch; the slices are validated first and a bad key on ANY rank rejects the whole batch
 *     on EVERY rank with the same status, nothing mutated; then routed to the owners by an
 *     all-to-all-v in rank order (the last occurrence of a key in the global batch -- rank
 *     order, then slice order -- wins, R10) and applied to each rank's shard.
 *   gpma_bfs(root, levels[V]) / gpma_cc(labels[V]) / gpma_pagerank(rank[V], ...): the full,
 *     replicated result vector on every rank (PR: fixed-point pushes reduce-scattered to their
 *     owners each iteration, bit-identical to the single-store sums; one all-gather at the end).
 * Local (not collective): gpma_export_csr (the owned rows: row_ptr has row_end-row_begin+1
 * entries), gpma_stats, gpma_query_* on owned rows, gpma_destroy (collective teardown of the
 * communicator is the caller's responsibility: destroy on every rank).  gpma_pagerank_f32 is not
 * available on a dist handle (GPMA_ERR_INVALID_ARG). */

/* 128-byte NCCL unique id (ncclGetUniqueId): call on ONE rank, broadcast it (e.g. with
 * torch.distributed) and pass it to gpma_dist_create on every rank. */
gpma_status gpma_dist_unique_id(void *id_out);

/* Create rank `rank` of `nranks` over the global vertex set [0, num_vertices): the CUDA device
 * current on the calling thread is the rank's GPU.  init_keys/init_vals: this rank's slice of
 * the initial edge set (routed to the owners).  cfg: as gpma_create (row_begin/row_end are
 * ignored -- R24 sets them).  Collective.  Errors: INVALID_ARG (nranks > V, bad rank, bad cfg),
 * RANGE / RESERVED (a bad initial key on any rank), CUDA (NCCL missing or failing), OOM. */
gpma_status gpma_dist_create(const void *nccl_unique_id, int rank, int nranks, uint32_t num_vertices,
                             const uint64_t *init_keys, const uint32_t *init_vals, uint64_t n_init,
                             const gpma_config *cfg, gpma_stream_t stream, gpma_t **out);

/* Rank, rank count and owned rows of a handle (a plain handle: 0, 1, its rows). */
gpma_status gpma_dist_info(const gpma_t *g, int *rank, int *nranks, uint32_t *row_begin, uint32_t *row_end);

/* ---------------------------------------------------------------- sharded stores
 * Multi-GPU ("evenly partition graphs according to the vertex index and
 * synchronize all devices after each iteration"; R24): one store per rank holds
 * the rows [row_begin, row_end) of owner(u) = u / ceil(V / P) (gpma_config.row_begin/end).
 * The primitives below are the per-rank steps between the collectives of a distributed
 * update / BFS / CC / PageRank (the caller, e.g. paper_journals_pvldb_shalht17_b200.dist,
 * runs the collectives).  All their array arguments are DEVICE pointers. */

/* Stable partition of a batch slice by owner rank: out_keys/out_vals (n each) hold the
 * owner-0 keys, then owner-1, ...; counts[nranks] (HOST) the piece sizes.  vals may be NULL
 * (zeros are routed).  Works on any handle (only V is used). */
gpma_status gpma_route(gpma_t *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, uint32_t nranks,
                       uint64_t *out_keys, uint32_t *out_vals, uint64_t *counts, gpma_stream_t stream);

/* levels[V] := -1, levels[root] := 0. */
gpma_status gpma_bfs_init(gpma_t *g, uint32_t root, int32_t *levels, gpma_stream_t stream);
/* One BFS level (Alg. 3 over the owned rows): frontier = {v : levels[v] == depth-1};
 * unreached out-neighbours of the owned frontier rows get `depth`.  *frontier_size (HOST) =
 * |frontier| (0: done).  Combine shards with an element-wise MAX of levels between levels. */
gpma_status gpma_bfs_level(gpma_t *g, int32_t *levels, int32_t depth, uint32_t *frontier_size,
                           gpma_stream_t stream);
/* One CC round over the owned edges on top of labels[V] (a forest with labels[x] <= x;
 * init != 0 starts from the identity): hook + compress.  *changed (HOST) = labels moved.
 * Combine shards with an element-wise MIN; the fixpoint (no shard changes) is the min-id
 * labelling of the weak components (R19). */
gpma_status gpma_cc_round(gpma_t *g, uint32_t *labels, int init, uint64_t *changed, gpma_stream_t stream);
/* PageRank push over the owned rows: x[V] (replicated; init != 0 sets 1/V first) ->
 * y[0..V) += sum over owned edges u->v of x[u]/outdeg(u), y[V] += dangling mass of the owned
 * rows; y is 64-bit fixed point with 2^-62 units.  Combine shards with a SUM of y. */
gpma_status gpma_pr_push(gpma_t *g, double *x, int init, uint64_t *y, gpma_stream_t stream);
/* x'[v] = (1-d)/V + d*(y[v] + y[V]/V) for every v; *err (HOST) = ||x'-x||_1; y := 0. */
gpma_status gpma_pr_update(gpma_t *g, double *x, uint64_t *y, double damping, double *err,
                           gpma_stream_t stream);
/* The same update for the OWNED rows only, after a reduce-scatter of the pushes (SURVEY
 * §8(e)): y_rows[0..nr) (device) = the summed y of rows [row_begin, row_end), y_rows[nr] = the
 * total dangling mass (2^-62 units); x[row_begin + i] := (1-d)/V + d*(y_rows[i] + y_rows[nr]/V);
 * *err (HOST) = the owned rows' part of ||x'-x||_1 (sum it over the ranks).  y_rows is not
 * modified; x outside the owned rows is not touched (all-gather the owned slices for the full
 * vector).  P:1215-1227. */
gpma_status gpma_pr_update_rows(gpma_t *g, double *x, const uint64_t *y_rows, double damping, double *err,
                                gpma_stream_t stream);
/* gpma_pr_update_rows with the error left on the DEVICE: *err_dev (device double) += the owned
 * rows' part of ||x'-x||_1; no host synchronisation (the caller all-reduces err_dev and reads
 * it once per iteration). */
gpma_status gpma_pr_update_rows_dev(gpma_t *g, double *x, const uint64_t *y_rows, double damping, double *err_dev,
                                    gpma_stream_t stream);
/* Validate a batch slice against the GLOBAL vertex range without touching the store (the
 * first step of a distributed update: every rank validates its slice and the ranks agree on
 * the status before anything is routed or applied).  Returns GPMA_OK / GPMA_ERR_RANGE /
 * GPMA_ERR_RESERVED (insert: vals checked too; vals may be NULL for a delete). */
gpma_status gpma_validate_batch(gpma_t *g, const uint64_t *keys, const uint32_t *vals, uint64_t n, gpma_op op,
                                gpma_stream_t stream);
/* Multi-GPU BFS exchange ("synchronize all devices after each
 * iteration"): bitmap[ceil(V/32)] (device) := bit v set iff levels[v] == depth, i.e. this
 * rank's discoveries of the level just expanded.  Ranks all-gather their bitmaps (V/8 bytes
 * each instead of an all-reduce of 4V-byte levels). */
gpma_status gpma_bfs_bits(gpma_t *g, const int32_t *levels, int32_t depth, uint32_t *bitmap, gpma_stream_t stream);
/* levels[v] := depth where levels[v] == -1 and bit v is set in any of the nbitmaps bitmaps
 * laid out back to back (ceil(V/32) words each, device).  After it, levels are replicated. */
gpma_status gpma_bfs_merge(gpma_t *g, int32_t *levels, const uint32_t *bitmaps, uint32_t nbitmaps, int32_t depth,
                           gpma_stream_t stream);

/* Kernel profiler (bench evidence, CUDA events on the call's stream around each launch):
 * filter NULL/"" = off, "*" = every kernel, else one kernel name (e.g. "k_pr_push").
 * Setting the filter clears the records. */
gpma_status gpma_debug_profile(gpma_t *g, const char *kernel_filter);
/* Synchronises the stream of the recorded launches and writes one line per kernel name,
 * "name<TAB>launches<TAB>total_ms\n", into buf (NUL-terminated, truncated to buflen);
 * clears the records. */
gpma_status gpma_debug_profile_read(gpma_t *g, char *buf, size_t buflen);

/* Number of kernels this handle has launched since create (bench evidence). */
uint64_t gpma_kernel_launches(const gpma_t *g);

const char *gpma_status_string(gpma_status s);
const char *gpma_last_error(const gpma_t *g);

#ifdef __cplusplus
}
#endif
#endif /* GPMA_H */
