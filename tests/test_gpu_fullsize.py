"""Parity at BASELINE.json's full sizes, through the same C-ABI calls bench.py times.

* configs[2] (Graph500 RMAT s24, 2^27-edge window, 1M-edge slides): the complete 2^28-slot layout
  (keys, values, row offsets, leaf counts, locate heads), export_csr, BFS, CC and PageRank after
  two full slides -- element by element against the oracle.
* configs[1] (Pokec-shaped, 15M-edge window): slides of 10^2, 10^4 and 10^6 edges.
* configs[3] (uniform, strict deletes, grow then shrink): the schedule scaled down 2^8 so the
  oracle follows every step; doublings and halvings must both happen.
"""
import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import CONFIGS, bfs_root, config_stream
from gpma_gen.streams import StreamConfig, edge_values, make_stream
from tests.gpu_helpers import (DEV, assert_pr_close, assert_same_csr, assert_same_layout, gpu_bfs, gpu_cc,
                               gpu_pr)

pytestmark = [pytest.mark.gpu, pytest.mark.slow]


def _store_pair(sw, V, mode=O.LAZY):
    from paper_journals_pvldb_shalht17_b200 import Gpma
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.contiguous().to(DEV), v0.contiguous().to(DEV), delete_mode=mode)
    o = O.Oracle(V, k0.cpu(), v0.cpu(), delete_mode=mode)
    return g, o


def test_config2_full_size():
    """configs[2] at full size, on a side stream exactly as bench.py drives it: slide 0 runs the
    prefixes plainly, slide 1 captures them as CUDA graphs, slide 2 REPLAYS them (1M-key batches)."""
    cfg = CONFIGS[2]
    sw = config_stream(2, device=DEV)
    V = cfg.V
    g, o = _store_pair(sw, V)
    assert_same_layout(g, o, what="config2 create")
    x = None
    st = torch.cuda.Stream()
    for s in range(3):
        dk, ik, iv = sw.slide(s)
        with torch.cuda.stream(st):
            g.gpma_update_batch(dk.contiguous(), None, 1, stream=st)
            g.gpma_update_batch(ik.contiguous(), iv.contiguous(), 0, stream=st)
        st.synchronize()
        o.delete(dk.cpu())
        o.insert(ik.cpu(), iv.cpu())
        if s != 1:
            assert_same_layout(g, o, what=f"config2 slide {s}")
    assert_same_csr(g, o, what="config2")
    root = bfs_root(sw, cfg.seed, 1)
    assert np.array_equal(gpu_bfs(g, root), o.bfs(root))
    assert np.array_equal(gpu_cc(g), o.cc())
    xg, _ = gpu_pr(g, tol=0.0, max_iter=3)
    xo, _ = o.pagerank(tol=0.0, max_iter=3)
    assert_pr_close(xg, xo, what="config2 fp64")
    x32, _ = gpu_pr(g, tol=0.0, max_iter=3, dtype=torch.float32)
    assert_pr_close(x32, xo, fp64=False, what="config2 fp32")


def test_config1_pokec_shaped_batch_sizes():
    cfg = CONFIGS[1]
    sw = config_stream(1, device=DEV)
    g, o = _store_pair(sw, cfg.V)
    pos = 0
    for B in (100, 10_000, 1_000_000):
        dk = sw.keys[pos:pos + B]
        ik = sw.keys[sw.window + pos: sw.window + pos + B]
        iv = sw.vals[sw.window + pos: sw.window + pos + B]
        pos += B
        g.delete(dk.contiguous())
        g.insert(ik.contiguous(), iv.contiguous())
        o.delete(dk.cpu())
        o.insert(ik.cpu(), iv.cpu())
        assert_same_layout(g, o, what=f"config1 B={B}")
    assert_same_csr(g, o, what="config1")


def test_config3_resize_stress_scaled():
    """configs[3] scaled down: V=2^12, pool 2^20 uniform edges, strict deletes; grow with
    (insert 2^12 new, delete 2^10 oldest), then shrink with (insert 2^10, delete 2^12 oldest)
    until few edges are left (V guards keep the density above min_h otherwise)."""
    from paper_journals_pvldb_shalht17_b200 import Gpma
    V, pool_n = 1 << 12, 1 << 20
    pool = make_stream("uniform", V, pool_n, CONFIGS[3].seed, device=DEV)
    vals = edge_values(pool, CONFIGS[3].seed)
    live0 = 1 << 15
    g = Gpma.gpma_create(V, pool[:live0].contiguous(), vals[:live0].contiguous(), delete_mode=1)
    o = O.Oracle(V, pool[:live0].cpu(), vals[:live0].cpu(), delete_mode=O.REBALANCE)
    lo, hi = 0, live0          # live = pool[lo:hi]
    caps = [o.capacity]
    big_heads = 0
    for step in range(146):
        if step < 70:
            ni, nd = 1 << 12, 1 << 10
        else:
            ni, nd = 1 << 10, 1 << 12
        nd = min(nd, hi - lo)
        ik, iv = pool[hi:hi + ni], vals[hi:hi + ni]
        dk = pool[lo:lo + nd]
        g.insert(ik.contiguous(), iv.contiguous())
        o.insert(ik.cpu(), iv.cpu())
        g.delete(dk.contiguous())
        o.delete(dk.cpu())
        big_heads += g.gpma_stats_host()["last_big_head_windows"]
        hi += ni
        lo += nd
        assert_same_layout(g, o, what=f"config3-scaled step {step}")
        caps.append(o.capacity)
    assert max(caps) > caps[0], "no doubling happened"
    assert caps[-1] < max(caps), "no halving happened"
    assert g.gpma_stats()["resizes"] == o.stats()["resizes"]
    assert_same_csr(g, o, what="config3-scaled")
    assert big_heads > 0, "no rewritten window of >= 2048 leaves (k_heads_span) was exercised"


def _resize_pair(V, cap0, E0, seed, mode):
    """A configs[3]-shaped store (V = 2^24, uniform edges) created at capacity cap0 (override) on
    both sides, the edges' stream returned for the batches that follow."""
    from paper_journals_pvldb_shalht17_b200 import Gpma
    pool = make_stream("uniform", V, E0 + (1 << 21), seed, device=DEV)
    vals = edge_values(pool, seed)
    g = Gpma.gpma_create(V, pool[:E0].contiguous(), vals[:E0].contiguous(), delete_mode=mode, initial_capacity=cap0)
    o = O.Oracle(V, pool[:E0].cpu(), vals[:E0].cpu(), delete_mode=mode, capacity=cap0)
    return g, o, pool, vals


def test_config3_full_size_doubling():
    """configs[3] at full size (V = 2^24): a store at capacity 2^26 holding just under the root
    bound max_h (R5) takes one hot 2^20-edge insert batch whose climb reaches the root, which
    doubles to 2^27 (Alg. 4 l.16-17, R14) -- the whole 2^27-slot layout against the oracle."""
    V, cap0 = 1 << 24, 1 << 26
    mx = O.thresholds(16, 22)[1][22]
    E0 = mx - V - (1 << 18)
    g, o, pool, vals = _resize_pair(V, cap0, E0, CONFIGS[3].seed + 11, 0)
    # a hot batch (NEXT-4 shape): 2^20 new edges from 64 consecutive rows, so every window that
    # holds them is over its bound up to the root (an even one would be absorbed at the leaves)
    i = torch.arange(1 << 20, device=DEV)
    ik = (((1000 + i // (1 << 14)) << 32) | ((i % (1 << 14)) * 1021 % V)).contiguous()
    iv = (i % 1000).to(torch.int32).contiguous()
    g.insert(ik, iv)
    o.insert(ik.cpu(), iv.cpu())
    assert o.capacity == 1 << 27 and o.stats()["resizes"] == 1
    assert_same_layout(g, o, what="config3 doubling 2^26 -> 2^27")
    assert g.gpma_stats()["resizes"] == 1


def test_config3_full_size_halving():
    """configs[3] at full size, strict deletes: a store at capacity 2^28 far below the root's
    lower bound (V guards + 2^22 edges) -- every deletion climbs to the root, which halves while
    N < min_h and the half can hold N (R14): 2^28 -> 2^25 in one batch, compared slot by slot."""
    V, cap0, E0 = 1 << 24, 1 << 28, 1 << 22
    g, o, pool, vals = _resize_pair(V, cap0, E0, CONFIGS[3].seed + 12, 1)
    dk = pool[: 1 << 20].contiguous()
    g.delete(dk)
    o.delete(dk.cpu())
    assert o.capacity < cap0 and o.stats()["resizes"] >= 1
    assert_same_layout(g, o, what=f"config3 halving 2^28 -> {o.capacity}")
    assert g.gpma_stats()["capacity"] == o.capacity
