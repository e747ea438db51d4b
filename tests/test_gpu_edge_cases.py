"""Degenerate and extreme inputs: the CUDA path must equal the oracle bit for bit."""
import numpy as np
import pytest
import torch

import oracle as O
from tests.brute import Replay
from tests.gpu_helpers import DEV, assert_same_csr, assert_same_layout, gpu_bfs, gpu_cc, keys_t, vals_t

pytestmark = pytest.mark.gpu


def _pair(V, keys, vals, **kw):
    from paper_journals_pvldb_shalht17_b200 import Gpma
    mode = kw.pop("delete_mode", 0)
    L = kw.pop("leaf_slots", 0)
    bp = kw.pop("thresholds_bp", None)
    g = Gpma.gpma_create(V, keys_t(keys) if len(keys) else None, vals_t(vals) if len(keys) else None,
                         delete_mode=mode, leaf_slots=L, thresholds_bp=bp)
    o = O.Oracle(V, keys, vals, delete_mode=mode, leaf_slots=L)
    if bp:
        O.lib().orc_set_thresholds_bp(o._h, *bp)
    return g, o


def _apply(g, o, keys, vals=None, op=0):
    if op == 0:
        g.insert(keys_t(keys), vals_t(vals))
        o.insert(keys, vals)
    else:
        g.delete(keys_t(keys))
        o.delete(keys)
    assert_same_layout(g, o)


def test_single_vertex_self_loop():
    g, o = _pair(1, [], [])
    _apply(g, o, [0], [5])
    assert gpu_bfs(g, 0).tolist() == [0] and gpu_cc(g).tolist() == [0]
    _apply(g, o, [0], op=1)
    _apply(g, o, [0], [6])
    assert_same_csr(g, o)


def test_extreme_ids_and_values():
    V = (1 << 20) + 3
    top = V - 1
    keys = [(top << 32) | top, (top << 32), top, 0]
    vals = [0, 0x7FFFFFFF, 0xFFFFFFFE, 1]
    g, o = _pair(V, keys, vals)
    _apply(g, o, [(top << 32) | (top - 1), (1 << 32) | top], [0xFFFFFFFE, 3])
    _apply(g, o, [(top << 32) | top], op=1)
    assert_same_csr(g, o)


@pytest.mark.parametrize("mode", [0, 1])
def test_all_duplicates_and_delete_everything(mode):
    V = 64
    g, o = _pair(V, [], [], delete_mode=mode)
    k = (5 << 32) | 7
    _apply(g, o, [k] * 3000, list(range(3000)))                  # radix-sort path, one key
    rng = np.random.default_rng(2)
    ks = list({int(a) << 32 | int(b) for a, b in zip(rng.integers(0, V, 3000), rng.integers(0, V, 3000))})
    _apply(g, o, ks, [1] * len(ks))
    _apply(g, o, ks + [k], op=1)                                 # the store is empty again
    assert g.gpma_stats()["live_edges"] == 0
    _apply(g, o, ks[:100], [2] * 100)                            # re-insert (revive in lazy mode)
    assert_same_csr(g, o)


@pytest.mark.parametrize("L", [4, 8, 32])
def test_leaf_size_overrides(L):
    rng = np.random.default_rng(L)
    V = 300
    keys = [int(a) << 32 | int(b) for a, b in zip(rng.integers(0, V, 2000), rng.integers(0, V, 2000))]
    g, o = _pair(V, keys, [1] * len(keys), leaf_slots=L)
    ref = Replay(V, keys, [1] * len(keys))
    for step in range(12):
        b = int(rng.integers(1, 3000))
        ks = [int(a) << 32 | int(c) for a, c in zip(rng.integers(0, V, b), rng.integers(0, V, b))]
        if step % 3 == 2:
            _apply(g, o, ks, op=1)
            ref.delete(ks)
        else:
            vs = rng.integers(0, 1 << 31, len(ks)).tolist()
            _apply(g, o, ks, vs)
            ref.insert(ks, vs)
    assert g.gpma_stats()["leaf_slots"] == L
    assert_same_csr(g, o)


def test_threshold_overrides():
    rng = np.random.default_rng(9)
    V = 200
    bp = (1500, 3000, 7000, 6000)                                # tighter bounds: more climbs/resizes
    keys = [int(a) << 32 | int(b) for a, b in zip(rng.integers(0, V, 500), rng.integers(0, V, 500))]
    g, o = _pair(V, keys, [0] * 500, thresholds_bp=bp, delete_mode=1)
    for step in range(15):
        ks = [int(a) << 32 | int(b) for a, b in zip(rng.integers(0, V, 400), rng.integers(0, V, 400))]
        _apply(g, o, ks, [step] * len(ks), op=step % 2)


def test_halving_down_to_minimum_capacity():
    V = 4
    keys = [(a << 32) | b for a in range(V) for b in range(V)]
    g, o = _pair(V, keys, [1] * len(keys), delete_mode=1)
    for k in keys:                                               # one at a time: many halvings
        _apply(g, o, [k], op=1)
    st = g.gpma_stats()
    assert st["capacity"] == o.capacity and st["live_edges"] == 0


@pytest.mark.parametrize("n", [2047, 2048, 2049, 4095, 4096, 4097, 8191, 12288, 12289, 300_001])
def test_sort_tiles_and_stability(n):
    """Batch sizes around the small-sort limit (2048) and the onesweep tile (4096 keys), with
    heavy duplication and distinct values: the stable sort must let the LAST copy of every key
    win (R10) across tile boundaries; deletes of the same keys (keys-only sort) after that."""
    rng = np.random.default_rng(n)
    V = 1 << 12
    g, o = _pair(V, [], [])
    pool = np.unique(rng.integers(0, V, 4 * n) << 32 | rng.integers(0, V, 4 * n))[: max(n // 3, 1)]
    keys = pool[rng.integers(0, pool.size, n)].astype(np.uint64).tolist()
    vals = rng.integers(0, 1 << 31, n).tolist()
    _apply(g, o, keys, vals)
    assert_same_csr(g, o)
    _apply(g, o, keys[: n // 2], op=1)
    assert_same_csr(g, o)


@pytest.mark.parametrize("n", [1, 2, 3, 31, 33, 63, 64, 65, 127, 129, 1000, 1025, 2047, 2048])
def test_small_path_sizes_and_stability(n, monkeypatch):
    """The one-kernel small-batch insert (GPMA_SMALL=2048: every size here) across the bitonic
    sort's register / shuffle / shared-memory stride regimes and padding, with duplicated keys
    (the LAST copy wins, R10) into a populated store, then the same keys deleted."""
    monkeypatch.setenv("GPMA_SMALL", "2048")
    rng = np.random.default_rng(77 + n)
    V = 1 << 10
    k0 = np.unique(rng.integers(0, V, 3000) << 32 | rng.integers(0, V, 3000)).astype(np.uint64).tolist()
    g, o = _pair(V, k0, [1] * len(k0))
    pool = np.unique(rng.integers(0, V, 4 * n) << 32 | rng.integers(0, V, 4 * n))[: max(n // 2, 1)]
    keys = pool[rng.integers(0, pool.size, n)].astype(np.uint64).tolist()
    vals = rng.integers(0, 1 << 31, n).tolist()
    _apply(g, o, keys, vals)
    assert_same_csr(g, o)
    _apply(g, o, keys[: max(n // 2, 1)], op=1)
    assert_same_csr(g, o)


@pytest.mark.parametrize("bad_at", [0, 1500, 2999])
def test_multi_cta_small_delete_rejects_whole_batch(bad_at):
    """A 3000-key lazy delete takes the multi-CTA one-kernel path (6 CTAs): one invalid key
    anywhere -- in another CTA's slice -- must leave the store untouched (every CTA validates
    the whole batch before any marks), and the valid batch then deletes exactly the live keys."""
    from paper_journals_pvldb_shalht17_b200 import GpmaError
    rng = np.random.default_rng(5 + bad_at)
    V = 1 << 11
    k0 = np.unique(rng.integers(0, V, 20000) << 32 | rng.integers(0, V, 20000)).astype(np.uint64).tolist()
    g, o = _pair(V, k0, [1] * len(k0))
    dk = [k0[i] for i in rng.integers(0, len(k0), 3000)]
    bad = list(dk)
    bad[bad_at] = (V + 3) << 32 | 1                    # src out of range
    with pytest.raises(GpmaError):
        g.delete(keys_t(bad))
    assert_same_layout(g, o)
    _apply(g, o, dk, op=1)
    assert_same_csr(g, o)


@pytest.mark.parametrize("direct", ["1", "0"])
def test_large_device_batch_direct_vs_staged(direct, monkeypatch):
    """Batches of >= 2^16 device keys on the read-only paths (leaf-keyed insert, unsorted lazy
    delete) can be read in place without staging or graph replay (GPMA_DIRECT=1); the default
    staged / graph-replayed path (0) must give the same layouts, with duplicates (R10) and
    deletes of absent keys."""
    monkeypatch.setenv("GPMA_DIRECT", direct)
    rng = np.random.default_rng(404)
    V = 1 << 13
    k0 = np.unique(rng.integers(0, V, 150000) << 32 | rng.integers(0, V, 150000)).astype(np.uint64).tolist()
    g, o = _pair(V, k0, [1] * len(k0))
    for step in range(3):
        n = 70000 + 1000 * step
        ks = (rng.integers(0, V, n) << 32 | rng.integers(0, V, n)).astype(np.uint64).tolist()
        vs = rng.integers(0, 1 << 31, n).tolist()
        _apply(g, o, ks, vs)
        dk = [k0[i] for i in rng.integers(0, len(k0), n)]
        _apply(g, o, dk, op=1)
    assert_same_csr(g, o)


def test_torch_allocator_hooks():
    """gpma_config.alloc/free through PyTorch's caching allocator (SURVEY §8(b) "Ownership"): the
    store lives in torch's pool while the handle lives, the results are unchanged, and destroy
    hands every block back."""
    from gpma_gen import config_stream
    from paper_journals_pvldb_shalht17_b200 import Gpma
    sw = config_stream(0, seed=9)
    V = 1024
    k0, v0 = sw.initial()
    torch.cuda.synchronize()
    before = torch.cuda.memory_allocated()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV), torch_allocator=True)
    o = O.Oracle(V, k0, v0)
    cap = g.gpma_stats()["capacity"]
    assert torch.cuda.memory_allocated() - before >= cap * 12      # keys + values at least
    for s in range(3):
        dk, ik, iv = sw.slide(s)
        g.delete(dk.to(DEV))
        g.insert(ik.to(DEV), iv.to(DEV))
        o.delete(dk)
        o.insert(ik, iv)
        assert_same_layout(g, o, what=f"torch allocator slide {s}")
    assert_same_csr(g, o)
    torch.cuda.synchronize()
    mid = torch.cuda.memory_allocated()
    g.gpma_destroy()
    torch.cuda.synchronize()
    end = torch.cuda.memory_allocated()
    assert mid - end >= cap * 12                                     # the store went back to torch
    assert end <= before + (2 << 20)                                 # (torch's own lazy state aside)


@pytest.mark.parametrize("mode", [0, 1])
def test_oversized_leaf_groups(mode):
    """NEXT-4 adversarial batch: 30000 updates piling into two source rows (the leaf groups hold
    thousands of updates, heavy duplication with distinct values, so the last copy must win), mixed
    with ordinary random updates: the oversized groups take the key-sorted fallback, the rest the
    thread-per-group merge -- one layout, equal to the oracle's."""
    rng = np.random.default_rng(77)
    V = 4096
    k0 = ((rng.integers(0, V, 20000) << 32) | rng.integers(0, V, 20000)).astype(np.uint64).tolist()
    g, o = _pair(V, k0, [1] * len(k0), delete_mode=mode)
    hot = (np.repeat([7, 3001], 15000) << 32) | rng.integers(0, 6000, 30000) % V
    rnd = (rng.integers(0, V, 5000) << 32) | rng.integers(0, V, 5000)
    ks = np.concatenate([hot, rnd]).astype(np.uint64)
    perm = rng.permutation(ks.size)
    ks = ks[perm].tolist()
    vs = rng.integers(0, 1 << 31, len(ks)).tolist()
    _apply(g, o, ks, vs)
    assert_same_csr(g, o)
    _apply(g, o, ks[:8000], op=1)
    _apply(g, o, ks[4000:12000], vs[4000:12000])
    assert_same_csr(g, o)


@pytest.mark.parametrize("mode", [0, 1])
def test_dead_level_skip_intermediate_and_root(mode):
    """The dead-level skip: a hot batch from a handful of rows climbs levels where its
    one or two windows reject (nacc = 0 with >= 2^14 pending), so the skip jumps to the first level
    whose window accepts (Alg. 4 l.23-25: n_W + |U_W| is unchanged by lower levels) -- the layout,
    top level, windows and slots rewritten must equal both the oracle and the loop run level by
    level (GPMA_LVL_SKIP=0).  Then strict deletes of the same keys climb the same way."""
    import os
    V = 1 << 12
    rng = np.random.default_rng(5)
    src = rng.integers(0, V, 1 << 17, dtype=np.uint64)
    dst = rng.integers(0, V, 1 << 17, dtype=np.uint64)
    k0 = np.unique((src << np.uint64(32)) | dst)
    v0 = (np.arange(len(k0)) % 1000).astype(np.uint32)
    hot = np.array([(np.uint64(7 + r) << np.uint64(32)) | np.uint64(c) for r in range(5) for c in range(V)],
                   dtype=np.uint64)
    hot = np.setdiff1d(hot, k0)[: 3 * (1 << 13)]                    # >= 2^14 new keys, 5 rows
    hv = (np.arange(len(hot)) % 777).astype(np.uint32)
    stats = []
    for skip in ("1", "0"):
        os.environ["GPMA_LVL_SKIP"] = skip
        try:
            g, o = _pair(V, k0, v0, delete_mode=mode)
            _apply(g, o, hot, hv)
            si = g.gpma_stats()
            if mode == 1:
                _apply(g, o, hot, op=1)
            sd = g.gpma_stats()
            stats.append((si, sd))
        finally:
            os.environ.pop("GPMA_LVL_SKIP", None)
    (si1, sd1), (si0, sd0) = stats
    # (windows / slots rewritten only where no update reaches the root: a root-reaching climb jumps
    # to the root, whose rewrite supersedes the lower ones -- same layout, fewer rewrites)
    def keys(st):
        # (windows / slots rewritten differ by design: the climb plan rewrites each region once,
        # at its highest accepted window -- same layout, fewer rewrites)
        return ("last_top_level", "capacity", "resizes")
    assert {k: si1[k] for k in keys(si1)} == {k: si0[k] for k in keys(si1)}
    assert {k: sd1[k] for k in keys(sd1)} == {k: sd0[k] for k in keys(sd1)}
    assert si1["last_levels_skipped"] > 0 and si0["last_levels_skipped"] == 0
    assert si1["last_top_level"] <= si1["height"], "the hot batch should be absorbed below the root"


@pytest.mark.parametrize("knob", ["", "GPMA_GATHER_BIG=0"])
@pytest.mark.parametrize("L", [4, 16, 32])
def test_big_window_gather_paths(knob, L, monkeypatch):
    """Windows of >= 4096 slots (high levels, the resize root) are gathered by the merge-path chunk
    walk (default) or the per-slot global search: each must give the oracle's layout through
    doublings, a hot-row climb, large strict deletes and halvings of a sparse root -- with leaf sizes 4 / 16 / 32 (1024 / 256
    / 128 leaf prefixes per chunk) and chunks whose pending run is empty, within the first 32
    keys, or longer than the staging."""
    for kv in filter(None, knob.split(",")):
        k, v = kv.split("=")
        monkeypatch.setenv(k, v)
    monkeypatch.setenv("GPMA_SMALL", "0")
    V = 1 << 12
    rng = np.random.default_rng(11 + L)
    src = rng.integers(0, V, 1 << 15, dtype=np.uint64)
    dst = rng.integers(0, V, 1 << 15, dtype=np.uint64)
    k0 = np.unique((src << np.uint64(32)) | dst)
    g, o = _pair(V, k0[:4000], (np.arange(4000) % 97).astype(np.uint32), delete_mode=1, leaf_slots=L)
    rest = k0[4000:]
    for i in range(0, len(rest), 9000):                          # doublings (root-level gathers)
        ks = rest[i:i + 9000]
        _apply(g, o, ks, (np.arange(len(ks)) % 89).astype(np.uint32))
    hot = np.array([(np.uint64(3) << np.uint64(32)) | np.uint64(c) for c in range(V)], dtype=np.uint64)
    hot = np.setdiff1d(hot, k0)                                  # one row: a long pending run
    _apply(g, o, hot, np.full(len(hot), 5, np.uint32))
    _apply(g, o, hot[::2], op=1)
    live = np.setdiff1d(np.concatenate([k0, hot]), hot[::2])
    _apply(g, o, live[: len(live) * 3 // 4], op=1)
    _apply(g, o, live[len(live) * 3 // 4::3], op=1)
    cap_grown = g.gpma_stats()["capacity"]
    rest = np.setdiff1d(live[len(live) * 3 // 4:], live[len(live) * 3 // 4::3])
    _apply(g, o, rest[: len(rest) - len(rest) // 6], op=1)      # a sparse root: halvings
    assert_same_csr(g, o)
    st = g.gpma_stats()
    assert st["resizes"] >= 3 and st["capacity"] < cap_grown and cap_grown >= 1 << 15
