"""CUDA path vs the CPU oracle, element by element (bit-exact layout; PR within 1e-6 / 1e-4).

Every call goes through the C ABI (libgpma.so) via the thin ctypes binding.
"""
import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import config_stream, fig3_layout, fig5_edges, bfs_root
from tests.brute import Replay
from tests.gpu_helpers import (DEV, assert_pr_close, assert_same_csr, assert_same_layout, gpu_bfs, gpu_cc,
                               gpu_pr, keys_t, vals_t)

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_journals_pvldb_shalht17_b200 import DELETE_LAZY, DELETE_REBALANCE, Gpma, GpmaError


def _trace_levels(tr):
    levels = []
    for lvl, start, off, flag in tr.tolist():
        while len(levels) <= lvl:
            levels.append({"segments": [], "offsets": [], "flags": []})
        if flag == 2:
            levels[lvl]["offsets"].append(off)
        else:
            levels[lvl]["segments"].append(start)
            levels[lvl]["offsets"].append(off)
            levels[lvl]["flags"].append("Y" if flag else "N")
    return levels


def test_example4_on_gpu(golden):
    """Ex. 4 / Fig. 6 on the GPU: every round and the final layout."""
    g4 = golden("ex4_gpma_plus.json")
    raw = fig3_layout()
    g = Gpma.gpma_create_raw(64, 32, 4, raw.to(DEV), torch.zeros(32, dtype=torch.int32, device=DEV))
    o = O.Oracle.raw(64, 32, 4, raw)
    g.gpma_debug_set_trace(True)
    g.insert(keys_t(g4["insert"]), vals_t([7] * 5))
    o.insert(g4["insert"], [7] * 5)
    tr = _trace_levels(g.gpma_debug_trace())
    assert len(tr) == len(g4["rounds"])
    for got, want in zip(tr, g4["rounds"]):
        assert got["segments"] == want["segments"]
        assert got["offsets"] == want["offsets"]
        assert got["flags"] == want["flags"]
    assert_same_layout(g, o, guards=False, what="ex4")


def test_example1_on_gpu():
    raw = fig3_layout()
    g = Gpma.gpma_create_raw(64, 32, 4, raw.to(DEV), torch.zeros(32, dtype=torch.int32, device=DEV))
    o = O.Oracle.raw(64, 32, 4, raw)
    g.gpma_debug_set_trace(True)
    g.insert(keys_t([48]), vals_t([1]))
    o.insert([48], [1])
    tr = _trace_levels(g.gpma_debug_trace())
    assert [lv["flags"] for lv in tr] == [["N"], ["N"], ["Y"]]
    assert tr[2]["segments"] == [16]
    assert_same_layout(g, o, guards=False, what="ex1")


def test_fig5_on_gpu(golden):
    f5 = golden("fig5_csr.json")
    keys = [s << 32 | d for s, d, _ in fig5_edges()]
    vals = [w for _, _, w in fig5_edges()]
    g = Gpma.gpma_create(3, keys_t(keys), vals_t(vals))
    o = O.Oracle(3, keys, vals)
    st = assert_same_layout(g, o, what="fig5")
    assert st["capacity"] == 16 and st["leaf_slots"] == 4
    rp, col = assert_same_csr(g, o, what="fig5")
    assert rp.tolist() == f5["csr_row_ptr"] and col.tolist() == f5["csr_col"]


def _slide_parity(seed, mode, analytics=True, trace=True, stream=None):
    """One configs[0] stream, every slide.  trace=True runs the generic level-0 step (per-level
    trace compared too); trace=False the fused kernels (k_del_mark, k_ins_leaf); a side stream
    additionally replays the batch prefix as a CUDA graph from the second slide of a shape on."""
    sw = config_stream(0, seed=seed)
    V = 1024
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV), delete_mode=mode)
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    assert_same_layout(g, o, what=f"seed {seed} create")
    g.gpma_debug_set_trace(trace)
    x_g = x_o = None
    for s in range(sw.n_slides):
        dk, ik, iv = sw.slide(s)
        if stream is not None:
            with torch.cuda.stream(stream):
                g.gpma_update_batch(dk.to(DEV), None, 1, stream=stream)
                o.delete(dk)
                assert_same_layout(g, o, what=f"seed {seed} slide {s} delete (stream)")
                g.gpma_update_batch(ik.to(DEV), iv.to(DEV), 0, stream=stream)
                o.insert(ik, iv)
                stream.synchronize()
                assert_same_layout(g, o, what=f"seed {seed} slide {s} insert (stream)")
                assert_same_csr(g, o, what=f"seed {seed} slide {s}")
            continue
        g.delete(dk.to(DEV))
        o.delete(dk)
        if trace and mode == DELETE_REBALANCE:
            assert _trace_levels(g.gpma_debug_trace()) == o.trace(), f"seed {seed} slide {s} delete trace"
        assert_same_layout(g, o, what=f"seed {seed} slide {s} delete")
        g.insert(ik.to(DEV), iv.to(DEV))
        o.insert(ik, iv)
        if trace:
            assert _trace_levels(g.gpma_debug_trace()) == o.trace(), f"seed {seed} slide {s} insert trace"
        assert_same_layout(g, o, what=f"seed {seed} slide {s} insert")
        assert_same_csr(g, o, what=f"seed {seed} slide {s}")
        if analytics:
            root = bfs_root(sw, seed, s)
            assert np.array_equal(gpu_bfs(g, root), o.bfs(root)), f"seed {seed} slide {s} BFS"
            assert np.array_equal(gpu_cc(g), o.cc()), f"seed {seed} slide {s} CC"
            # PageRank: fixed K iterations, warm-started from the previous slide (R20)
            xg, itg = gpu_pr(g, x_g, tol=0.0, max_iter=8)
            xo, ito = o.pagerank(x=x_o, tol=0.0, max_iter=8)
            assert itg == ito == 8
            assert_pr_close(xg, xo, what=f"seed {seed} slide {s} PR")
            x_g, x_o = xg, xo


@pytest.mark.parametrize("path", ["small", "large"])
@pytest.mark.parametrize("seed", range(20))
def test_config0_sliding_window_lazy(seed, path, monkeypatch):
    """BASELINE configs[0]: RMAT s10 sliding window, every slide, 20 seeds, through
    both batch paths the bench times: the one-kernel small batch (1024-key batches take it by
    default) and the large-batch kernels (interleaved lazy delete, leaf-keyed insert)."""
    monkeypatch.setenv("GPMA_SMALL", "1024" if path == "small" else "0")
    _slide_parity(seed, DELETE_LAZY, trace=False)


@pytest.mark.parametrize("seed", range(6))
def test_config0_sliding_window_lazy_traced(seed):
    """The same streams through the generic level-0 step, with the per-level trace compared."""
    _slide_parity(seed, DELETE_LAZY, trace=True)


@pytest.mark.parametrize("seed", range(8))
def test_config0_sliding_window_graph_replay(seed, monkeypatch):
    """The 20-seed sweep's streams on a side stream: every batch after the first of a shape is a
    replayed CUDA graph of the batch prefix (validate, sort, locate, fused leaf merge, summary).
    (The one-kernel small path is not graph-replayed: GPMA_SMALL=0.)"""
    monkeypatch.setenv("GPMA_SMALL", "0")
    _slide_parity(seed, DELETE_LAZY, analytics=False, trace=False, stream=torch.cuda.Stream())


@pytest.mark.parametrize("knob", ["GPMA_DEL_SORT=1", "GPMA_INS_FUSED=0", "GPMA_INS_LEAFSORT=0",
                                  "GPMA_INS_LEAFSORT=0,GPMA_INS_THREAD=0", "GPMA_LVL_COOP=0", "GPMA_LVL_WARP=0", "GPMA_INTERP=0", "GPMA_ILP=1",
                                  "GPMA_ILP=4", "GPMA_SMALL=2048", "GPMA_SMALL=0,GPMA_DEL_SORT=1",
                                  "GPMA_GSTART_FUSED=0", "GPMA_LVL_SKIP=0", "GPMA_ROOT_JUMP=0", "GPMA_LVL_PLAN=0"])
@pytest.mark.parametrize("seed", range(3))
def test_config0_alternative_paths(seed, knob, monkeypatch):
    """The strategy switches give the same layouts as the defaults (configs[0] batches are 1024 keys,
    forced onto the large-batch kernels -- leaf-keyed insert, interleaved lazy delete -- with
    GPMA_SMALL=0; GPMA_SMALL=2048 sends them through the one-kernel small-batch path -- and the other
    knobs through the alternatives: sorted lazy delete, separate pre-pass + k_level0, key-sorted
    fused insert by a thread or a sub-warp per leaf, the host-driven level loop, 1- or 4-way probe
    interleaving)."""
    for kv in knob.split(","):
        k, v = kv.split("=")
        monkeypatch.setenv(k, v)
    if "GPMA_SMALL" not in knob:
        monkeypatch.setenv("GPMA_SMALL", "0")         # the knobs act on the large-batch kernels
    _slide_parity(300 + seed, DELETE_LAZY, analytics=False, trace=False)


@pytest.mark.parametrize("seed", range(5))
def test_config0_sliding_window_rebalance(seed):
    _slide_parity(100 + seed, DELETE_REBALANCE)


def _keys(src, dst):
    return [(int(s) << 32) | int(d) for s, d in zip(src, dst)]


@pytest.mark.parametrize("mode", [0, 1])
@pytest.mark.parametrize("seed", range(12))
def test_random_small_with_resizes(seed, mode):
    """Tiny graphs, random mixed batches with duplicates: doubling, halving, tombstones."""
    rng = np.random.default_rng(seed)
    V = int(rng.integers(8, 64))
    n0 = int(rng.integers(0, 3 * V))
    k0 = _keys(rng.integers(0, V, n0), rng.integers(0, V, n0))
    v0 = rng.integers(0, 1 << 31, n0).tolist()
    g = Gpma.gpma_create(V, keys_t(k0), vals_t(v0), delete_mode=mode) if n0 else \
        Gpma.gpma_create(V, None, None, delete_mode=mode)
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    ref = Replay(V, k0, v0)
    assert_same_layout(g, o, what="create")
    for step in range(30):
        b = int(rng.integers(1, 4 * V))
        ks = _keys(rng.integers(0, V, b), rng.integers(0, V, b))
        if rng.random() < 0.55:
            vs = rng.integers(0, 1 << 31, len(ks)).tolist()
            g.insert(keys_t(ks), vals_t(vs))
            o.insert(ks, vs)
            ref.insert(ks, vs)
        else:
            if ref.m:
                pres = list(ref.m)
                ks = [pres[i] for i in rng.integers(0, len(pres), min(b, len(pres)))] + ks[: b // 4]
            g.delete(keys_t(ks))
            o.delete(ks)
            ref.delete(ks)
        assert_same_layout(g, o, what=f"seed {seed} step {step}")
    assert_same_csr(g, o)
    assert g.gpma_stats()["live_edges"] == len(ref.m)


def test_errors_leave_store_untouched():
    V = 16
    k0 = _keys([0, 1, 2], [1, 2, 3])
    g = Gpma.gpma_create(V, keys_t(k0), vals_t([1, 2, 3]))
    o = O.Oracle(V, k0, [1, 2, 3])
    for keys, vals, op, want in [
        ([(20 << 32) | 1], [1], 0, 2),                 # src out of range
        ([(1 << 32) | 17], None, 1, 2),                # dst out of range (delete)
        ([(1 << 32) | 0xFFFFFFFF], [1], 0, 3),         # guard column
        ([(1 << 32) | 5], [0xFFFFFFFF], 0, 3),         # tombstone value
    ]:
        st = g.gpma_update_batch(keys_t(keys), None if vals is None else vals_t(vals), op, check=False)
        assert st == want
        assert_same_layout(g, o, what="after rejected batch")
    assert g.gpma_update_batch(keys_t([]), vals_t([]), 0, check=False) == 0


def test_host_pointer_api():
    """The C ABI accepts host buffers (staged by the library) and returns the same results."""
    sw = config_stream(0, seed=3)
    V = 1024
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.contiguous(), v0.contiguous())        # CPU tensors = host pointers
    o = O.Oracle(V, k0, v0)
    dk, ik, iv = sw.slide(0)
    g.delete(dk.contiguous().pin_memory())
    g.insert(ik.contiguous(), iv.contiguous())
    o.delete(dk)
    o.insert(ik, iv)
    assert_same_layout(g, o)
    lv = np.zeros(V, np.int32)
    g.gpma_bfs(7, lv)
    assert np.array_equal(lv, o.bfs(7))
    lab = np.zeros(V, np.uint32)
    g.gpma_cc(lab)
    assert np.array_equal(lab, o.cc())
    x = np.zeros(V, np.float64)
    g.gpma_pagerank(x, tol_l1=0.0, max_iter=5)
    assert_pr_close(x, o.pagerank(tol=0.0, max_iter=5)[0], what="host pointers")
    nnz = g.gpma_export_csr()
    rp, col, val = np.zeros(V + 1, np.uint64), np.zeros(nnz, np.uint32), np.zeros(nnz, np.uint32)
    g.gpma_export_csr(rp, col, val)
    orp, ocol, oval = o.export_csr()
    assert np.array_equal(rp, orp) and np.array_equal(col, ocol) and np.array_equal(val, oval)


def test_pagerank_f32_and_tolerance_mode():
    sw = config_stream(0, seed=7)
    V = 1024
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV))
    o = O.Oracle(V, k0, v0)
    x32, it32 = gpu_pr(g, tol=0.0, max_iter=15, dtype=torch.float32)
    xo, _ = o.pagerank(tol=0.0, max_iter=15)
    assert it32 == 15
    assert_pr_close(x32, xo, fp64=False, what="fp32 V=1024")
    # tolerance mode: same stopping iteration as the oracle
    xg, itg = gpu_pr(g, tol=1e-3, max_iter=100)
    xo, ito = o.pagerank(tol=1e-3, max_iter=100)
    assert itg == ito
    assert_pr_close(xg, xo, what="tolerance mode")


@pytest.mark.parametrize("mode", [0, 1])
def test_medium_rmat_multi_tile(mode):
    """RMAT s16 (64K vertices, 1M edges), 32K-edge batches: multi-tile sort/scan, higher levels."""
    from gpma_gen.streams import StreamConfig
    cfg = StreamConfig("rmat-s16", "rmat", 1 << 16, 1 << 20, 1 << 19, 1 << 15, 0x5EED, scale=16)
    sw = config_stream(cfg, device=DEV)
    sw.keys, sw.vals = sw.keys.cpu(), sw.vals.cpu()
    V = 1 << 16
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV), delete_mode=mode)
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    assert_same_layout(g, o, what="create")
    for s in range(4):
        dk, ik, iv = sw.slide(s)
        g.delete(dk.to(DEV))
        o.delete(dk)
        g.insert(ik.to(DEV), iv.to(DEV))
        o.insert(ik, iv)
        assert_same_layout(g, o, what=f"slide {s}")
    assert_same_csr(g, o)
    root = bfs_root(sw, 1, 3)
    assert np.array_equal(gpu_bfs(g, root), o.bfs(root))
    assert np.array_equal(gpu_cc(g), o.cc())
    xg, _ = gpu_pr(g, tol=0.0, max_iter=6)
    xo = o.pagerank(tol=0.0, max_iter=6)[0]
    assert_pr_close(xg, xo, what="rmat-s16 fp64")
    x32, _ = gpu_pr(g, tol=0.0, max_iter=6, dtype=torch.float32)   # fp32 at V = 2^16
    assert_pr_close(x32, xo, fp64=False, what="rmat-s16 fp32")


@pytest.mark.parametrize("coop", ["1", "0", "1-blockmerge"])
@pytest.mark.parametrize("mode", [0, 1])
def test_sorted_stream_hot_window(coop, mode, monkeypatch):
    """Ascending-key batches concentrated in one region (NEXT-4 pattern): deep climbs through the
    device-resident level loop (coop=1: levels with windows <= 4096 slots in one cooperative
    kernel) or the host-driven one, then strict / lazy deletes of the hot keys."""
    monkeypatch.setenv("GPMA_LVL_COOP", coop[0])
    monkeypatch.setenv("GPMA_LVL_WARP", "0" if coop.endswith("blockmerge") else "1")
    V = 4096
    rng = np.random.default_rng(11)
    k0 = _keys(rng.integers(0, V, 20000), rng.integers(0, V, 20000))
    v0 = [1] * len(k0)
    g = Gpma.gpma_create(V, keys_t(k0), vals_t(v0), delete_mode=mode)
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    for b in range(6):
        ks = _keys(np.full(3000, 7 + b), np.arange(3000))
        g.insert(keys_t(ks), vals_t([b] * 3000))
        o.insert(ks, [b] * 3000)
        assert_same_layout(g, o, what=f"hot batch {b}")
    for b in range(6):
        ks = _keys(np.full(2500, 7 + b), np.arange(500, 3000))
        g.delete(keys_t(ks))
        o.delete(ks)
        assert_same_layout(g, o, what=f"hot delete {b}")
    assert g.gpma_stats()["resizes"] == o.stats()["resizes"]


def test_gpma_lock_example2_on_gpu(golden):
    """NEXT-2: GPMA (Alg. 1) on the GPU, Ex. 2 batch: same rounds and layout as the oracle."""
    g2 = golden("ex2_gpma_lock.json")
    raw = fig3_layout()
    g = Gpma.gpma_create_raw(64, 32, 4, raw.to(DEV), torch.zeros(32, dtype=torch.int32, device=DEV), algorithm=1)
    o = O.Oracle.raw(64, 32, 4, raw, algorithm=1)
    g.insert(keys_t(g2["batch"]), vals_t([0] * 5))
    o.insert(g2["batch"], [0] * 5)
    assert g.gpma_stats()["last_rounds"] == o.rounds == g2["rounds"]
    assert_same_layout(g, o, guards=False, what="ex2")


@pytest.mark.parametrize("seed", range(6))
def test_gpma_lock_sliding_window(seed):
    """NEXT-2: GPMA inserts + lazy deletes on configs[0] streams, layout parity every slide."""
    sw = config_stream(0, seed=200 + seed)
    V = 1024
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV), algorithm=1)
    o = O.Oracle(V, k0, v0, algorithm=1)
    for s in range(4):
        dk, ik, iv = sw.slide(s)
        g.delete(dk.to(DEV))
        g.insert(ik.to(DEV), iv.to(DEV))
        o.delete(dk)
        o.insert(ik, iv)
        assert g.gpma_stats()["last_rounds"] == o.rounds
        assert_same_layout(g, o, what=f"gpma seed {seed} slide {s}")
    assert_same_csr(g, o)


@pytest.mark.parametrize("seed", range(4))
def test_gpma_lock_hot_rows_and_doubling(seed):
    rng = np.random.default_rng(seed)
    V = 64
    g = Gpma.gpma_create(V, None, None, algorithm=1)
    o = O.Oracle(V, [], [], algorithm=1)
    for step in range(12):
        b = int(rng.integers(50, 400))
        ks = _keys(rng.integers(0, 8, b), rng.integers(0, V, b))
        vs = rng.integers(0, 1 << 31, len(ks)).tolist()
        g.insert(keys_t(ks), vals_t(vs))
        o.insert(ks, vs)
        assert_same_layout(g, o, what=f"gpma hot seed {seed} step {step}")
    assert g.gpma_stats()["resizes"] == o.stats()["resizes"] > 0


@pytest.mark.parametrize("split", ["0", "1"])
def test_pagerank_push_strategies(split, monkeypatch):
    """The PageRank push with and without the split (GPMA_PR_SPLIT: lower-half destinations RED'd in
    the sweep, upper half through a spill list) against the oracle, fp64 and fp32, fixed K and the
    tolerance mode (same stopping iteration)."""
    monkeypatch.setenv("GPMA_PR_SPLIT", split)
    from gpma_gen.streams import StreamConfig
    cfg = StreamConfig("rmat-s16", "rmat", 1 << 16, 1 << 20, 1 << 19, 1 << 15, 0x5EED + 3, scale=16)
    sw = config_stream(cfg, device=DEV)
    sw.keys, sw.vals = sw.keys.cpu(), sw.vals.cpu()
    V = 1 << 16
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV))
    o = O.Oracle(V, k0, v0)
    dk, ik, iv = sw.slide(0)
    g.delete(dk.to(DEV))
    g.insert(ik.to(DEV), iv.to(DEV))
    o.delete(dk)
    o.insert(ik, iv)
    xg, _ = gpu_pr(g, tol=0.0, max_iter=7)
    xo, _ = o.pagerank(tol=0.0, max_iter=7)
    assert_pr_close(xg, xo, what=f"split={split} fp64")
    x32, _ = gpu_pr(g, tol=0.0, max_iter=7, dtype=torch.float32)
    assert_pr_close(x32, xo, fp64=False, what=f"split={split} fp32")
    xg, itg = gpu_pr(g, xg, tol=1e-3, max_iter=100)
    xo2, ito = o.pagerank(x=xo, tol=1e-3, max_iter=100)
    assert itg == ito
    assert_pr_close(xg, xo2, what=f"split={split} tolerance mode")
