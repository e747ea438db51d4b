/*
 * gpma_oracle.c -- TEST INFRASTRUCTURE ONLY.
 *
 * A plain, slow, sequential CPU oracle for the GPMA+ dynamic-graph store of
 * Sha, Li, He, Tan, "Accelerating Dynamic Graph Analytics on GPUs", PVLDB 11(1)
 * 2017 (/root/reference/PAPER.md, cited as P:<line>).  Only tests/,
 * __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference legs may
 * load this library.  It shares no code, header, table or constant generator with
 * the CUDA library under paper_journals_pvldb_shalht17_b200/csrc/.
 *
 * What it implements, step by step in the paper's order (Alg. 4):
 *   Sort(U) -> BinarySearchLeafSegments -> level loop {UniqueSegments,
 *   TryInsert+ (CountSegment, CountUpdatesInSegment, density test, Merge,
 *   re-dispatch evenly), promote to parent} -> double the root;
 * deletions as the dual and lazy deletions
 * (P:1260-1266); the CSR-on-GPMA guard entries and row offsets (P:685-689,
 * Fig. 5); export to CSR; textbook BFS (Alg. 2), union-find
 * connected components and power-iteration PageRank
 * on the exported CSR.
 *
 * Readings of silent / garbled passages are SURVEY.md §8(c) R1-R29, repeated
 * in DESIGN.md "Readings".  Pins: tests/test_oracle_*.py -- the paper's worked
 * examples (Fig. 3, Ex. 1, Ex. 2, Ex. 4, Fig. 5), hand-derived root-resize and
 * strict-delete examples on the Fig. 3-size PMA (R6, R14, min_i;
 * tests/test_oracle_resize_pins.py), brute-force replay, closed forms and
 * library routines for the analytics; tools/oracle_mutations.sh checks that a
 * plausible mistake in each rule fails a pin.
 */
#include <stdint.h>
#include <stdlib.h>
#include <string.h>
#include <math.h>

#define ORC_KEY_NONE 0xFFFFFFFFFFFFFFFFull /* R2: empty slot                 */
#define ORC_TOMB 0xFFFFFFFFu               /* R12: lazily deleted entry      */
#define ORC_GUARD_COL 0xFFFFFFFFu          /* R1: guard column "infinity"    */

enum { ORC_OK = 0, ORC_INVALID = 1, ORC_RANGE = 2, ORC_RESERVED = 3, ORC_OOM = 4 };
enum { ORC_INSERT = 0, ORC_DELETE = 1 };
enum { ORC_LAZY = 0, ORC_REBALANCE = 1 };

typedef struct { uint64_t key; uint32_t val; uint32_t leaf; } upd_t;
typedef struct { uint32_t level; uint64_t seg_start_slot; uint64_t offset; uint32_t flag; } trace_t;

typedef struct orc {
  uint32_t V;
  uint32_t rb, nr;     /* owned rows [rb, rb+nr) of a source-range shard (R24); nr = V unsharded */
  uint64_t cap;        /* slots, a power of two                       */
  uint32_t L;          /* leaf segment size (R3)                      */
  uint32_t h;          /* height: cap = L * 2^h                       */
  int mode;            /* ORC_LAZY / ORC_REBALANCE (R12)              */
  uint32_t rho0, rhoh, tau0, tauh, init_bp; /* basis points (R4, R15)  */
  uint64_t *key;
  uint32_t *val;
  uint64_t *row_offset; /* nr+1 (R8), indexed by src - rb               */
  uint64_t *tmin, *tmax;/* h+1 integer entry bounds (R5)              */
  /* last-batch diagnostics */
  trace_t *trace; uint64_t ntrace, trace_cap;
  uint64_t slots_rewritten, windows_rewritten, top_level, pending_after_prepass;
  uint64_t resizes, resizes_last;
  int algorithm;       /* 0 = GPMA+ (Alg. 4), 1 = GPMA lock-based (Alg. 1)            */
  uint64_t rounds_last;/* GPMA: retry rounds of the last batch                        */
  uint64_t max_rounds; /* GPMA test hook: stop after this many rounds (0 = until done) */
} orc_t;

/* ---------------------------------------------------------------- thresholds */
/* R4: rho_i, tau_i linear in the level between the leaf and root values of the
 * Fig. 3 table.  R5: min_i = min(ceil(rho_i * size_i), 2*min_{i-1}),
 * max_i = min(floor(tau_i * size_i), 2*max_{i-1}), exact integer arithmetic.    */
void orc_thresholds(uint64_t L, uint32_t h, uint32_t rho0, uint32_t rhoh, uint32_t tau0,
                    uint32_t tauh, uint64_t *mn, uint64_t *mx) {
  uint32_t i;
  for (i = 0; i <= h; i++) {
    uint64_t size = L << i;
    uint64_t den = 10000ull * (h ? h : 1);
    uint64_t rnum = h ? ((uint64_t)rho0 * (h - i) + (uint64_t)rhoh * i) : rho0;
    uint64_t tnum = h ? ((uint64_t)tau0 * (h - i) + (uint64_t)tauh * i) : tau0;
    uint64_t raw_min = (rnum * size + den - 1) / den;
    uint64_t raw_max = (tnum * size) / den;
    if (i == 0) { mn[i] = raw_min; mx[i] = raw_max; }
    else {
      mn[i] = raw_min < 2 * mn[i - 1] ? raw_min : 2 * mn[i - 1];
      mx[i] = raw_max < 2 * mx[i - 1] ? raw_max : 2 * mx[i - 1];
    }
  }
}

static uint32_t ilog2_u64(uint64_t x) { uint32_t r = 0; while (x > 1) { x >>= 1; r++; } return r; }

/* R3: L = max(4, 2^floor(log2(log2 cap0))). */
uint32_t orc_leaf_rule(uint64_t cap0) {
  uint32_t lg = ilog2_u64(cap0);
  uint32_t L = 1u << ilog2_u64(lg);
  return L < 4 ? 4 : L;
}

static int is_occupied(uint64_t k) { return k != ORC_KEY_NONE; }
static int is_guard(uint64_t k) { return k != ORC_KEY_NONE && (uint32_t)(k & 0xFFFFFFFFu) == ORC_GUARD_COL; }
static int is_live(const orc_t *o, uint64_t s) { return is_occupied(o->key[s]) && o->val[s] != ORC_TOMB; }

static int set_geometry(orc_t *o, uint64_t cap) {
  o->cap = cap;
  o->h = ilog2_u64(cap / o->L);
  free(o->tmin); free(o->tmax);
  o->tmin = (uint64_t *)malloc(sizeof(uint64_t) * (o->h + 1));
  o->tmax = (uint64_t *)malloc(sizeof(uint64_t) * (o->h + 1));
  if (!o->tmin || !o->tmax) return ORC_OOM;
  orc_thresholds(o->L, o->h, o->rho0, o->rhoh, o->tau0, o->tauh, o->tmin, o->tmax);
  return ORC_OK;
}

/* R7 "re-dispatch entries in s evenly" (Alg. 4 l.27; Alg. 1 l.17):
 * leaf l of the nl leaves starting at leaf l0 receives entries
 * [floor(l*N/nl), floor((l+1)*N/nl)) of the sorted list, left-packed (the new
 * entry is "placed at the rear of leaf segment"); the rest is empty.
 * R8: a guard written to slot s sets row_offset[src+1] = s. */
static void redispatch(orc_t *o, uint64_t l0, uint64_t nl, const uint64_t *k, const uint32_t *v,
                       uint64_t N) {
  uint64_t l, p;
  for (l = 0; l < nl; l++) {
    uint64_t lo = l * N / nl, hi = (l + 1) * N / nl;
    for (p = 0; p < o->L; p++) {
      uint64_t s = (l0 + l) * o->L + p;
      if (p < hi - lo) {
        o->key[s] = k[lo + p];
        o->val[s] = v[lo + p];
        if (is_guard(k[lo + p]) && o->row_offset)
          o->row_offset[(k[lo + p] >> 32) - o->rb + 1] = s;
      } else {
        o->key[s] = ORC_KEY_NONE;
        o->val[s] = 0;
      }
    }
  }
}

static void trace_push(orc_t *o, uint32_t level, uint64_t start, uint64_t off, uint32_t flag) {
  if (o->ntrace == o->trace_cap) {
    o->trace_cap = o->trace_cap ? 2 * o->trace_cap : 64;
    o->trace = (trace_t *)realloc(o->trace, sizeof(trace_t) * o->trace_cap);
  }
  o->trace[o->ntrace].level = level;
  o->trace[o->ntrace].seg_start_slot = start;
  o->trace[o->ntrace].offset = off;
  o->trace[o->ntrace].flag = flag;
  o->ntrace++;
}

/* ---------------------------------------------------------------- create */
static orc_t *alloc_orc(uint32_t V, int mode) {
  orc_t *o = (orc_t *)calloc(1, sizeof(orc_t));
  if (!o) return NULL;
  o->V = V; o->mode = mode; o->rb = 0; o->nr = V;
  o->rho0 = 800; o->rhoh = 4000; o->tau0 = 9200; o->tauh = 8000; o->init_bp = 6000;
  return o;
}

void orc_set_thresholds_bp(orc_t *o, uint32_t rho0, uint32_t rhoh, uint32_t tau0, uint32_t tauh) {
  o->rho0 = rho0; o->rhoh = rhoh; o->tau0 = tau0; o->tauh = tauh;
  set_geometry(o, o->cap);
}

typedef struct { uint64_t key; uint64_t idx; uint32_t val; } kv_t;
static int cmp_kv(const void *a, const void *b) {
  const kv_t *x = (const kv_t *)a, *y = (const kv_t *)b;
  if (x->key != y->key) return x->key < y->key ? -1 : 1;
  return x->idx < y->idx ? -1 : (x->idx > y->idx);
}

/* Validation (SURVEY §8(b) "Errors"): RESERVED (guard column / tombstone value)
 * takes precedence over RANGE (src or dst >= V); nothing is mutated on error. */
static int validate(uint32_t V, uint32_t rb, uint32_t nr, const uint64_t *k, const uint32_t *v, uint64_t n,
                    int check_vals) {
  uint64_t i; int range = 0;
  for (i = 0; i < n; i++) {
    uint32_t src = (uint32_t)(k[i] >> 32), dst = (uint32_t)k[i];
    if (dst == ORC_GUARD_COL) return ORC_RESERVED;
    if (check_vals && v && v[i] == ORC_TOMB) return ORC_RESERVED;
    if (src < rb || src - rb >= nr || dst >= V) range = 1;
  }
  return range ? ORC_RANGE : ORC_OK;
}

/* Stable sort by key, keep the LAST occurrence of each key (R10).  Returns m. */
static uint64_t sort_unique_last(const uint64_t *k, const uint32_t *v, uint64_t n, kv_t **out) {
  uint64_t i, m = 0;
  kv_t *a = (kv_t *)malloc(sizeof(kv_t) * (n ? n : 1));
  for (i = 0; i < n; i++) { a[i].key = k[i]; a[i].idx = i; a[i].val = v ? v[i] : 0; }
  qsort(a, n, sizeof(kv_t), cmp_kv);
  for (i = 0; i < n; i++)
    if (i + 1 == n || a[i + 1].key != a[i].key) a[m++] = a[i];
  *out = a;
  return m;
}

/* R15: initial capacity = smallest power of two >= 8 with E0 + V <= floor(cap * 0.6);
 * L from cap0 (R3); bump cap0 to 2L if smaller; proportional split over all leaves. */
/* Source-range shard (R24): the store holds rows [row_begin, row_end) -- their guards,
 * row offsets and edges; row_end == 0 means all rows. */
orc_t *orc_create_shard(uint32_t V, uint32_t row_begin, uint32_t row_end, const uint64_t *keys,
                        const uint32_t *vals, uint64_t n, uint32_t leaf_slots, uint64_t cap_override,
                        int mode, int *status) {
  kv_t *u = NULL; uint64_t m, E, i, j, cap;
  uint64_t *ek; uint32_t *ev;
  orc_t *o;
  uint32_t rb = row_end > row_begin ? row_begin : 0, nr = row_end > row_begin ? row_end - row_begin : V;
  int st = validate(V, rb, nr, keys, vals, n, 1);
  if (st) { *status = st; return NULL; }
  o = alloc_orc(V, mode);
  o->rb = rb; o->nr = nr;
  m = sort_unique_last(keys, vals, n, &u);
  E = m + nr;
  /* merge the sorted edges with the guards (u<<32 | inf) of the owned rows, R1 */
  ek = (uint64_t *)malloc(sizeof(uint64_t) * (E ? E : 1));
  ev = (uint32_t *)malloc(sizeof(uint32_t) * (E ? E : 1));
  for (i = 0, j = 0; i < m || j < nr;) {
    uint64_t g = j < nr ? (((uint64_t)(j + rb) << 32) | ORC_GUARD_COL) : ORC_KEY_NONE;
    if (i < m && u[i].key < g) { ek[i + j] = u[i].key; ev[i + j] = u[i].val; i++; }
    else { ek[i + j] = g; ev[i + j] = 0; j++; }
  }
  free(u);
  if (cap_override) {
    cap = cap_override;
    o->L = leaf_slots ? leaf_slots : orc_leaf_rule(cap);
  } else {
    cap = 8;
    while (E > cap * o->init_bp / 10000) cap *= 2;
    o->L = leaf_slots ? leaf_slots : orc_leaf_rule(cap);
    if (cap < 2ull * o->L) cap = 2ull * o->L;
  }
  o->key = (uint64_t *)malloc(sizeof(uint64_t) * cap);
  o->val = (uint32_t *)malloc(sizeof(uint32_t) * cap);
  o->row_offset = (uint64_t *)calloc((uint64_t)nr + 1, sizeof(uint64_t));
  set_geometry(o, cap);
  redispatch(o, 0, cap / o->L, ek, ev, E);
  free(ek); free(ev);
  *status = ORC_OK;
  return o;
}

orc_t *orc_create(uint32_t V, const uint64_t *keys, const uint32_t *vals, uint64_t n,
                  uint32_t leaf_slots, uint64_t cap_override, int mode, int *status) {
  return orc_create_shard(V, 0, 0, keys, vals, n, leaf_slots, cap_override, mode, status);
}

/* Test hook: load a raw layout (e.g. the Fig. 3 PMA), no guards required. */
orc_t *orc_create_raw(uint32_t V, uint64_t cap, uint32_t L, const uint64_t *keys,
                      const uint32_t *vals, int mode, int *status) {
  uint64_t s;
  orc_t *o = alloc_orc(V, mode);
  o->L = L;
  o->key = (uint64_t *)malloc(sizeof(uint64_t) * cap);
  o->val = (uint32_t *)malloc(sizeof(uint32_t) * cap);
  o->row_offset = (uint64_t *)calloc((uint64_t)V + 1, sizeof(uint64_t));
  set_geometry(o, cap);
  for (s = 0; s < cap; s++) {
    o->key[s] = keys[s];
    o->val[s] = vals ? vals[s] : 0;
    if (is_guard(keys[s])) o->row_offset[(keys[s] >> 32) + 1] = s;
  }
  *status = ORC_OK;
  return o;
}

void orc_destroy(orc_t *o) {
  if (!o) return;
  free(o->key); free(o->val); free(o->row_offset); free(o->tmin); free(o->tmax); free(o->trace);
  free(o);
}

/* ---------------------------------------------------------------- locate */
/* R9 (Alg. 4 l.3 BinarySearchLeafSegments; "the corresponding leaf segment is
 * firstly identified by a binary search"): target(k) = the largest leaf
 * containing an occupied slot (live, tombstone or guard) with key <= k, or 0.  Leaves
 * are left-packed and sorted, so a leaf's smallest key is its first slot. */
static uint64_t *nonempty_leaves(const orc_t *o, uint64_t *count) {
  uint64_t nl = o->cap / o->L, l, c = 0;
  uint64_t *idx = (uint64_t *)malloc(sizeof(uint64_t) * (nl ? nl : 1));
  for (l = 0; l < nl; l++)
    if (is_occupied(o->key[l * o->L])) idx[c++] = l;
  *count = c;
  return idx;
}

static uint32_t target_leaf(const orc_t *o, const uint64_t *ne, uint64_t nne, uint64_t k) {
  uint64_t lo = 0, hi = nne; /* first index whose head > k */
  while (lo < hi) {
    uint64_t mid = (lo + hi) / 2;
    if (o->key[ne[mid] * o->L] <= k) lo = mid + 1; else hi = mid;
  }
  return lo == 0 ? 0 : (uint32_t)ne[lo - 1];
}

/* ---------------------------------------------------------------- level loop */
/* Collect the live entries of slots [s0, s1) in order (tombstones dropped, R12). */
static uint64_t collect_live(const orc_t *o, uint64_t s0, uint64_t s1, uint64_t *k, uint32_t *v) {
  uint64_t s, c = 0;
  for (s = s0; s < s1; s++)
    if (is_live(o, s)) { k[c] = o->key[s]; v[c] = o->val[s]; c++; }
  return c;
}

/* Root resize (Alg. 4 l.16-17 "double the space of the old root segment", P:983-984;
 * halving as the dual).  R14: double repeatedly until everything fits
 * max_h of the new capacity; halve while below min_h and cap > 2L.  Everything live
 * plus the pending updates is re-dispatched over the whole new array (R7). */
static int resize(orc_t *o, const upd_t *P, uint64_t np, int op) {
  uint64_t nlive = 0, s, i, j, N, cap = o->cap, c;
  uint64_t *lk, *nk; uint32_t *lv, *nv;
  uint64_t *mn, *mx;
  for (s = 0; s < o->cap; s++) nlive += is_live(o, s);
  N = op == ORC_INSERT ? nlive + np : nlive - np;
  mn = (uint64_t *)malloc(sizeof(uint64_t) * 70);
  mx = (uint64_t *)malloc(sizeof(uint64_t) * 70);
  if (op == ORC_INSERT) {
    for (;;) {
      orc_thresholds(o->L, ilog2_u64(cap / o->L), o->rho0, o->rhoh, o->tau0, o->tauh, mn, mx);
      if (N <= mx[ilog2_u64(cap / o->L)]) break;
      cap *= 2;
    }
  } else {
    for (;;) {
      uint32_t hh = ilog2_u64(cap / o->L);
      orc_thresholds(o->L, hh, o->rho0, o->rhoh, o->tau0, o->tauh, mn, mx);
      if (!(cap > 2ull * o->L && N < mn[hh])) break;
      /* guard: never halve below what the smaller root may hold */
      orc_thresholds(o->L, hh - 1, o->rho0, o->rhoh, o->tau0, o->tauh, mn, mx);
      if (N > mx[hh - 1]) break;
      cap /= 2;
    }
  }
  free(mn); free(mx);
  lk = (uint64_t *)malloc(sizeof(uint64_t) * (nlive ? nlive : 1));
  lv = (uint32_t *)malloc(sizeof(uint32_t) * (nlive ? nlive : 1));
  collect_live(o, 0, o->cap, lk, lv);
  nk = (uint64_t *)malloc(sizeof(uint64_t) * (N + nlive + np + 1));
  nv = (uint32_t *)malloc(sizeof(uint32_t) * (N + nlive + np + 1));
  /* merge (insert) or subtract (delete) the sorted pending list */
  for (i = 0, j = 0, c = 0; i < nlive || j < np;) {
    if (op == ORC_INSERT) {
      if (j >= np || (i < nlive && lk[i] < P[j].key)) { nk[c] = lk[i]; nv[c] = lv[i]; c++; i++; }
      else { nk[c] = P[j].key; nv[c] = P[j].val; c++; j++; }
    } else {
      if (j < np && i < nlive && lk[i] == P[j].key) { i++; j++; }
      else if (j >= np || (i < nlive && lk[i] < P[j].key)) { nk[c] = lk[i]; nv[c] = lv[i]; c++; i++; }
      else j++; /* cannot happen: pending deletes are live keys */
    }
  }
  free(lk); free(lv);
  if (cap != o->cap) {
    uint64_t *k2 = (uint64_t *)malloc(sizeof(uint64_t) * cap);
    uint32_t *v2 = (uint32_t *)malloc(sizeof(uint32_t) * cap);
    if (!k2 || !v2) { free(k2); free(v2); free(nk); free(nv); return ORC_OOM; }
    free(o->key); free(o->val);
    o->key = k2; o->val = v2;
    set_geometry(o, cap);
    o->resizes++; o->resizes_last++;
  }
  redispatch(o, 0, o->cap / o->L, nk, nv, c);
  o->slots_rewritten += o->cap;
  o->windows_rewritten += 1;
  free(nk); free(nv);
  return ORC_OK;
}

/* Root doubling of GPMA (Alg. 1 l.20 "double the space of the root segment"): all
 * live entries re-dispatched evenly over twice the capacity (R7); nothing is inserted. */
static int double_root(orc_t *o) {
  uint64_t nlive = 0, s;
  uint64_t *lk, *k2; uint32_t *lv, *v2;
  for (s = 0; s < o->cap; s++) nlive += is_live(o, s);
  lk = (uint64_t *)malloc(sizeof(uint64_t) * (nlive ? nlive : 1));
  lv = (uint32_t *)malloc(sizeof(uint32_t) * (nlive ? nlive : 1));
  collect_live(o, 0, o->cap, lk, lv);
  k2 = (uint64_t *)malloc(sizeof(uint64_t) * o->cap * 2);
  v2 = (uint32_t *)malloc(sizeof(uint32_t) * o->cap * 2);
  free(o->key); free(o->val);
  o->key = k2; o->val = v2;
  set_geometry(o, o->cap * 2);
  redispatch(o, 0, o->cap / o->L, lk, lv, nlive);
  o->resizes++; o->resizes_last++;
  o->slots_rewritten += o->cap;
  o->windows_rewritten += 1;
  free(lk); free(lv);
  return ORC_OK;
}

static int cmp_upd(const void *a, const void *b) {
  const upd_t *x = (const upd_t *)a, *y = (const upd_t *)b;
  return x->key < y->key ? -1 : (x->key > y->key);
}

/* GPMA concurrent insertion (Alg. 1; Ex. 2) with deterministic lock
 * arbitration: every insertion searches its leaf, then the rounds climb level by level
 * ("all threads are synchronized after updating all segments located at the same tree
 * height").  At each level the insertions that reach the same segment compete for
 * its lock and the others abort until the next round (l.11-12).  The paper leaves the winner
 * open ("Assuming Insertion-1 succeeds"; "Insertion-48 wins"); R28: the
 * contender that climbed from the highest child segment wins, and among contenders of one
 * child (always the case at the leaves) the smallest key -- the one rule that reproduces both
 * printed choices of Ex. 2 (1 beats 4 in leaf 0; 48 from leaf 7 beats 35 from leaf 6 for
 * segment [24,31]).  A winner whose segment can take one more entry (count + 1 <= max_i, R5)
 * merges and re-dispatches it (l.16-17); otherwise it climbs (l.13-14).  As for GPMA+ (R6),
 * the root is tested too; a winner the root cannot take doubles it (l.20) and retries next
 * round.  Rounds repeat until every insertion took effect (l.2), or -- test hook only --
 * until max_rounds rounds ran (the aborted insertions are then dropped). */
static int gpma_lock_insert(orc_t *o, upd_t *P, uint64_t np) {
  upd_t *A = (upd_t *)malloc(sizeof(upd_t) * (np ? np : 1));
  upd_t *W = (upd_t *)malloc(sizeof(upd_t) * (np ? np : 1));
  uint64_t *wk = NULL; uint32_t *wv = NULL; uint64_t wcap = 0;
  o->rounds_last = 0;
  while (np > 0 && (!o->max_rounds || o->rounds_last < o->max_rounds)) {
    uint64_t na = 0, nw, j, nne;
    uint32_t i;
    uint64_t *ne = nonempty_leaves(o, &nne);
    o->rounds_last++;
    for (j = 0; j < np; j++) P[j].leaf = target_leaf(o, ne, nne, P[j].key);   /* l.4 */
    free(ne);
    memcpy(W, P, sizeof(upd_t) * np);
    nw = np;
    for (i = 0; i <= o->h && nw > 0; i++) {           /* up to the root, tested too (R6) */
      uint64_t nk = 0, g0 = 0;
      while (g0 < nw) {
        uint64_t seg = W[g0].leaf >> i, g1 = g0 + 1, s0, s1, n = 0, s, win, c;
        while (g1 < nw && (W[g1].leaf >> i) == seg) g1++;  /* contenders W[g0..g1), by key */
        /* R28: the highest child wins (child = leaf >> (i-1); one child at the leaves), and
         * within it the smallest key: the first contender of the last child run */
        win = g1 - 1;
        if (i > 0) {
          c = W[g1 - 1].leaf >> (i - 1);
          while (win > g0 && (W[win - 1].leaf >> (i - 1)) == c) win--;
        } else {
          win = g0;
        }
        for (s = g0; s < g1; s++)
          if (s != win) A[na++] = W[s];                 /* lose the lock: abort (l.11-12) */
        W[g0] = W[win];                                 /* the winner goes on below      */
        s0 = (seg << i) * o->L; s1 = s0 + ((uint64_t)o->L << i);
        for (s = s0; s < s1; s++) n += is_live(o, s);
        if (n + 1 <= o->tmax[i]) {                    /* l.13 test fails -> insert (l.16-17) */
          uint64_t a = 0, c = 0;
          uint64_t *lk = (uint64_t *)malloc(sizeof(uint64_t) * (n ? n : 1));
          uint32_t *lv = (uint32_t *)malloc(sizeof(uint32_t) * (n ? n : 1));
          int placed = 0;
          collect_live(o, s0, s1, lk, lv);
          if (n + 1 > wcap) {
            wcap = n + 1;
            wk = (uint64_t *)realloc(wk, sizeof(uint64_t) * wcap);
            wv = (uint32_t *)realloc(wv, sizeof(uint32_t) * wcap);
          }
          for (a = 0; a < n; a++) {
            if (!placed && W[g0].key < lk[a]) { wk[c] = W[g0].key; wv[c] = W[g0].val; c++; placed = 1; }
            wk[c] = lk[a]; wv[c] = lv[a]; c++;
          }
          if (!placed) { wk[c] = W[g0].key; wv[c] = W[g0].val; c++; }
          free(lk); free(lv);
          redispatch(o, seg << i, 1ull << i, wk, wv, c);
          o->slots_rewritten += s1 - s0;
          o->windows_rewritten += 1;
        } else {
          W[nk++] = W[g0];                            /* climb to the parent (l.14) */
        }
        g0 = g1;
      }
      nw = nk;
      if (i > o->top_level) o->top_level = i;
    }
    if (nw > 0) {                                     /* reached the root: double (l.20) */
      double_root(o);
      for (j = 0; j < nw; j++) A[na++] = W[j];
    }
    qsort(A, na, sizeof(upd_t), cmp_upd);
    memcpy(P, A, sizeof(upd_t) * na);
    np = na;
  }
  free(A); free(W); free(wk); free(wv);
  return ORC_OK;
}

void orc_set_algorithm(orc_t *o, int algorithm) { o->algorithm = algorithm; }
void orc_set_max_rounds(orc_t *o, uint64_t r) { o->max_rounds = r; }
uint64_t orc_rounds_last(const orc_t *o) { return o->rounds_last; }

/* GpmaPlusInsertion (Alg. 4) and its dual for strict deletions over the
 * pending list P (sorted by key, with leaf targets). */
static int level_loop(orc_t *o, upd_t *P, uint64_t np, int op) {
  uint32_t i;
  uint64_t *wk = NULL; uint32_t *wv = NULL; uint64_t wcap = 0;
  upd_t *Q = (upd_t *)malloc(sizeof(upd_t) * (np ? np : 1));
  int st = ORC_OK;
  for (i = 0; i <= o->h && np > 0; i++) {               /* "while root segment is not reached" */
    uint64_t j = 0, nq = 0;
    o->top_level = i;
    while (j < np) {                                    /* UniqueSegments = RLE + scan (l.18-21) */
      uint64_t seg = P[j].leaf >> i, g = j, u, n, s0, s1, N, a, b, c;
      int accept;
      while (g < np && (P[g].leaf >> i) == seg) g++;
      u = g - j;                                        /* CountUpdatesInSegment (l.24) */
      s0 = (seg << i) * o->L; s1 = s0 + ((uint64_t)o->L << i);
      n = 0;                                            /* CountSegment (l.23) */
      { uint64_t s; for (s = s0; s < s1; s++) n += is_live(o, s); }
      /* density test (l.25) with the integer bounds of R5 */
      accept = op == ORC_INSERT ? (n + u <= o->tmax[i]) : (n >= u && n - u >= o->tmin[i]);
      trace_push(o, i, s0, j, (uint32_t)accept);
      if (accept) {                                     /* Merge + re-dispatch (l.26-27) */
        if (n + u > wcap) {
          wcap = n + u;
          wk = (uint64_t *)realloc(wk, sizeof(uint64_t) * wcap);
          wv = (uint32_t *)realloc(wv, sizeof(uint32_t) * wcap);
        }
        {
          uint64_t *lk = (uint64_t *)malloc(sizeof(uint64_t) * (n ? n : 1));
          uint32_t *lv = (uint32_t *)malloc(sizeof(uint32_t) * (n ? n : 1));
          collect_live(o, s0, s1, lk, lv);
          for (a = 0, b = j, c = 0; a < n || b < g;) {
            if (op == ORC_INSERT) {
              if (b >= g || (a < n && lk[a] < P[b].key)) { wk[c] = lk[a]; wv[c] = lv[a]; c++; a++; }
              else { wk[c] = P[b].key; wv[c] = P[b].val; c++; b++; }
            } else {
              if (b < g && a < n && lk[a] == P[b].key) { a++; b++; }
              else if (b >= g || (a < n && lk[a] < P[b].key)) { wk[c] = lk[a]; wv[c] = lv[a]; c++; a++; }
              else b++;
            }
          }
          free(lk); free(lv);
          N = c;
        }
        redispatch(o, seg << i, 1ull << i, wk, wv, N);
        o->slots_rewritten += s1 - s0;
        o->windows_rewritten += 1;
      } else {                                          /* keep for the parent (l.12-15) */
        memcpy(Q + nq, P + j, sizeof(upd_t) * u);
        nq += u;
      }
      j = g;
    }
    trace_push(o, i, ORC_KEY_NONE, np, 2);              /* closing offset of level i */
    memcpy(P, Q, sizeof(upd_t) * nq);
    np = nq;
  }
  if (np > 0) {                                         /* root failed: resize (l.16-17) */
    o->top_level = o->h + 1;
    st = resize(o, P, np, op);
  }
  free(Q); free(wk); free(wv);
  return st;
}

int orc_update(orc_t *o, const uint64_t *keys, const uint32_t *vals, uint64_t n, int op) {
  kv_t *u = NULL; uint64_t m, i, np = 0, nne;
  uint64_t *ne;
  upd_t *P;
  int st;
  if (op != ORC_INSERT && op != ORC_DELETE) return ORC_INVALID;
  if (op == ORC_INSERT && n && !vals) return ORC_INVALID;
  st = validate(o->V, o->rb, o->nr, keys, vals, n, op == ORC_INSERT);
  if (st) return st;
  o->ntrace = 0; o->slots_rewritten = 0; o->windows_rewritten = 0; o->top_level = 0;
  o->resizes_last = 0; o->pending_after_prepass = 0;
  if (n == 0) return ORC_OK;
  m = sort_unique_last(keys, op == ORC_INSERT ? vals : NULL, n, &u);   /* Sort(U), l.2 */
  ne = nonempty_leaves(o, &nne);
  P = (upd_t *)malloc(sizeof(upd_t) * (m ? m : 1));
  for (i = 0; i < m; i++) {
    uint32_t t = target_leaf(o, ne, nne, u[i].key);                    /* l.3 */
    uint64_t s, hit = ORC_KEY_NONE;
    for (s = (uint64_t)t * o->L; s < (uint64_t)(t + 1) * o->L; s++)
      if (o->key[s] == u[i].key) hit = s;
    /* pre-pass: "modifications are trivial", R11/R12 */
    if (op == ORC_INSERT) {
      if (hit != ORC_KEY_NONE) { o->val[hit] = u[i].val; continue; }   /* overwrite / revive */
    } else if (o->mode == ORC_LAZY) {
      if (hit != ORC_KEY_NONE && o->val[hit] != ORC_TOMB) o->val[hit] = ORC_TOMB;
      continue;
    } else {
      if (hit == ORC_KEY_NONE || o->val[hit] == ORC_TOMB) continue;   /* absent: no-op */
    }
    P[np].key = u[i].key; P[np].val = u[i].val; P[np].leaf = t; np++;
  }
  free(ne); free(u);
  o->pending_after_prepass = np;
  if (np && op == ORC_INSERT && o->algorithm == 1) st = gpma_lock_insert(o, P, np);
  else st = np ? level_loop(o, P, np, op) : ORC_OK;
  free(P);
  return st;
}

/* ---------------------------------------------------------------- introspection */
uint64_t orc_capacity(const orc_t *o) { return o->cap; }
void orc_dump(const orc_t *o, uint64_t *k, uint32_t *v) {
  memcpy(k, o->key, sizeof(uint64_t) * o->cap);
  memcpy(v, o->val, sizeof(uint32_t) * o->cap);
}
void orc_row_offset(const orc_t *o, uint64_t *out) {
  memcpy(out, o->row_offset, sizeof(uint64_t) * ((uint64_t)o->nr + 1));
}
void orc_level_bounds(const orc_t *o, uint64_t *mn, uint64_t *mx) {
  memcpy(mn, o->tmin, sizeof(uint64_t) * (o->h + 1));
  memcpy(mx, o->tmax, sizeof(uint64_t) * (o->h + 1));
}
/* stats: cap, L, h, V, live edges, tombstones, guards, slots_rewritten(last),
 * windows_rewritten(last), top_level(last), pending_after_prepass(last),
 * resizes(total), resizes(last) */
void orc_stats(const orc_t *o, uint64_t *out) {
  uint64_t s, live = 0, tomb = 0, guards = 0;
  for (s = 0; s < o->cap; s++) {
    if (!is_occupied(o->key[s])) continue;
    if (is_guard(o->key[s])) guards++;
    else if (o->val[s] == ORC_TOMB) tomb++;
    else live++;
  }
  out[0] = o->cap; out[1] = o->L; out[2] = o->h; out[3] = o->V; out[4] = live; out[5] = tomb;
  out[6] = guards; out[7] = o->slots_rewritten; out[8] = o->windows_rewritten;
  out[9] = o->top_level; out[10] = o->pending_after_prepass; out[11] = o->resizes;
  out[12] = o->resizes_last;
  out[13] = o->rb;
  out[14] = o->nr;
}
/* Per-level trace of the last batch (Fig. 6 "Update Segments / Offsets / Successful
 * Flag"): records (level, seg_start_slot, offset, flag); flag 2 closes a level and
 * carries the final offset. */
uint64_t orc_trace(const orc_t *o, uint64_t *out4, uint64_t max_records) {
  uint64_t i;
  for (i = 0; i < o->ntrace && i < max_records; i++) {
    out4[4 * i + 0] = o->trace[i].level;
    out4[4 * i + 1] = o->trace[i].seg_start_slot;
    out4[4 * i + 2] = o->trace[i].offset;
    out4[4 * i + 3] = o->trace[i].flag;
  }
  return o->ntrace;
}

/* ---------------------------------------------------------------- export + analytics */
/* CSR view of the store (Fig. 5): live edges in slot order (= key order). */
/* rows [rb, rb+nr) of the shard (all rows unsharded): row_ptr has nr+1 entries */
uint64_t orc_export_csr(const orc_t *o, uint64_t *row_ptr, uint32_t *col, uint32_t *val) {
  uint64_t s, nnz = 0, u;
  if (row_ptr) for (u = 0; u <= o->nr; u++) row_ptr[u] = 0;
  for (s = 0; s < o->cap; s++) {
    if (!is_live(o, s) || is_guard(o->key[s])) continue;
    if (col) { col[nnz] = (uint32_t)o->key[s]; val[nnz] = o->val[s]; }
    if (row_ptr) row_ptr[(o->key[s] >> 32) - o->rb + 1]++;
    nnz++;
  }
  if (row_ptr) for (u = 0; u < o->nr; u++) row_ptr[u + 1] += row_ptr[u];
  return nnz;
}

/* BFS (Alg. 2): queue BFS, level = hop distance from root, -1 unreached. */
void orc_bfs_csr(uint32_t V, const uint64_t *row_ptr, const uint32_t *col, uint32_t root,
                 int32_t *level) {
  uint32_t *q = (uint32_t *)malloc(sizeof(uint32_t) * (V ? V : 1));
  uint64_t head = 0, tail = 0, e;
  uint32_t v;
  for (v = 0; v < V; v++) level[v] = -1;
  if (root < V) { level[root] = 0; q[tail++] = root; }
  while (head < tail) {
    uint32_t u = q[head++];
    for (e = row_ptr[u]; e < row_ptr[u + 1]; e++) {
      uint32_t w = col[e];
      if (level[w] < 0) { level[w] = level[u] + 1; q[tail++] = w; }
    }
  }
  free(q);
}

/* Connected components (R19 weak components, canonical min-id labels):
 * union-find with path halving, union by smaller id as root. */
static uint32_t uf_find(uint32_t *p, uint32_t x) {
  while (p[x] != x) { p[x] = p[p[x]]; x = p[x]; }
  return x;
}
void orc_cc_csr(uint32_t V, const uint64_t *row_ptr, const uint32_t *col, uint32_t *label) {
  uint32_t u; uint64_t e;
  for (u = 0; u < V; u++) label[u] = u;
  for (u = 0; u < V; u++)
    for (e = row_ptr[u]; e < row_ptr[u + 1]; e++) {
      uint32_t a = uf_find(label, u), b = uf_find(label, col[e]);
      if (a < b) label[b] = a; else if (b < a) label[a] = b;
    }
  for (u = 0; u < V; u++) label[u] = uf_find(label, u);
}

/* PageRank by power iteration (R20/R21): x' = (1-d)/V + d*(sum_{u->v}
 * x[u]/outdeg(u) + D/V), D = dangling mass; stop after the first iteration with
 * ||x'-x||_1 < tol (tol = 1e-3 in the paper; 0 = run max_iter); warm start uses the
 * caller's x.  Returns the number of iterations. */
int orc_pagerank_csr(uint32_t V, const uint64_t *row_ptr, const uint32_t *col, double *x,
                     int warm, double d, double tol, int max_iter) {
  double *y = (double *)malloc(sizeof(double) * (V ? V : 1));
  int it = 0;
  uint32_t u; uint64_t e;
  if (!warm) for (u = 0; u < V; u++) x[u] = 1.0 / V;
  while (it < max_iter) {
    double dangling = 0.0, err = 0.0;
    for (u = 0; u < V; u++) y[u] = 0.0;
    for (u = 0; u < V; u++) {
      uint64_t deg = row_ptr[u + 1] - row_ptr[u];
      if (deg == 0) { dangling += x[u]; continue; }
      for (e = row_ptr[u]; e < row_ptr[u + 1]; e++) y[col[e]] += x[u] / (double)deg;
    }
    for (u = 0; u < V; u++) {
      double nx = (1.0 - d) / V + d * (y[u] + dangling / V);
      err += fabs(nx - x[u]);
      x[u] = nx;
    }
    it++;
    if (err < tol) break;
  }
  free(y);
  return it;
}
