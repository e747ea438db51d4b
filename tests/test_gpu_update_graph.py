"""Update batches replayed as a CUDA graph (the prefix up to the batch's one read-back, DESIGN.md
§6) vs the oracle: same-shape batches on a side stream are captured on their second run and
replayed from the third; layouts, level traces, analytics and error statuses must equal the
plain launches' (Alg. 4; R1-R16)."""
import contextlib
import os

import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import config_stream
from tests.gpu_helpers import DEV, assert_same_csr, assert_same_layout, keys_t, vals_t

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_journals_pvldb_shalht17_b200 import DELETE_LAZY, DELETE_REBALANCE, Gpma


@contextlib.contextmanager
def env(**kv):
    old = {k: os.environ.get(k) for k in kv}
    os.environ.update({k: str(v) for k, v in kv.items()})
    try:
        yield
    finally:
        for k, v in old.items():
            if v is None:
                os.environ.pop(k, None)
            else:
                os.environ[k] = v


@pytest.mark.parametrize("mode", [0, 1])
@pytest.mark.parametrize("seed", range(4))
def test_graph_replayed_sliding_window(seed, mode):
    sw = config_stream(0, seed=seed)
    V = 1024
    k0, v0 = sw.initial()
    s = torch.cuda.Stream(DEV)
    with torch.cuda.stream(s):
        g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV), delete_mode=mode, stream=s)
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    for sl in range(sw.n_slides):
        dk, ik, iv = sw.slide(sl)
        dk, ik, iv = dk.to(DEV), ik.to(DEV), iv.to(DEV)
        torch.cuda.synchronize()
        g.gpma_update_batch(dk, None, 1, stream=s)
        g.gpma_update_batch(ik, iv, 0, stream=s)
        s.synchronize()
        o.delete(dk.cpu())
        o.insert(ik.cpu(), iv.cpu())
        assert_same_layout(g, o, what=f"seed {seed} slide {sl}")
    assert_same_csr(g, o)


def test_graph_replay_errors_and_launch_accounting():
    V = 64
    rng = np.random.default_rng(3)
    src = rng.integers(0, V, 400, dtype=np.uint64)
    dst = rng.integers(0, V, 400, dtype=np.uint64)
    keys = np.unique((src << np.uint64(32)) | dst)
    g = Gpma.gpma_create(V, keys_t(keys), vals_t(np.ones(keys.size, dtype=np.uint32)))
    o = O.Oracle(V, keys, np.ones(keys.size, dtype=np.uint32))
    s = torch.cuda.Stream(DEV)
    launches = []
    for it in range(6):
        b = np.unique((rng.integers(0, V, 8, dtype=np.uint64) << np.uint64(32)) | rng.integers(0, V, 8, dtype=np.uint64))[:5]
        while b.size < 5:
            b = np.append(b, np.uint64(b[-1] + 1))
        bad = b.copy()
        bad[2] = np.uint64(V + 3) << np.uint64(32)                  # src out of range
        kb, vb = keys_t(bad), vals_t(np.full(5, 9, dtype=np.uint32))
        l0 = g.gpma_kernel_launches()
        st = g.gpma_update_batch(kb, vb, 0, stream=s, check=False)
        s.synchronize()
        assert st == 2, f"iteration {it}: range error expected"
        assert_same_layout(g, o, what=f"rejected batch {it}")
        kg, vg = keys_t(b), vals_t(np.full(5, 7, dtype=np.uint32))
        g.gpma_update_batch(kg, vg, 0, stream=s)
        s.synchronize()
        o.insert(b, np.full(5, 7, dtype=np.uint32))
        assert_same_layout(g, o, what=f"batch {it}")
        launches.append(g.gpma_kernel_launches() - l0)
    assert min(launches) > 0
    # plain launches give the same count of kernels per batch as the replayed graph
    with env(GPMA_UPD_GRAPH="0"):
        l0 = g.gpma_kernel_launches()
        st = g.gpma_update_batch(kb, vb, 0, stream=s, check=False)
        kg2 = keys_t(b + np.uint64(1))
        g.gpma_update_batch(kg2, vg, 0, stream=s)
        s.synchronize()
        o.insert(b + np.uint64(1), np.full(5, 7, dtype=np.uint32))
        assert_same_layout(g, o, what="plain launches")


@pytest.mark.parametrize("mode", [0, 1])
@pytest.mark.parametrize("seed", range(6))
def test_graph_replay_across_resizes(seed, mode):
    """Fixed-size random insert / delete batches on a side stream (so the prefix graph is
    captured and replayed) on tiny graphs whose capacity doubles and halves: a resize changes
    the signature (store pointers, geometry), the graph is dropped and re-captured; layouts
    must equal the oracle after every batch."""
    rng = np.random.default_rng(100 + seed)
    V = int(rng.integers(16, 48))
    n0 = 4 * V
    k0 = [(int(a) << 32) | int(b) for a, b in zip(rng.integers(0, V, n0), rng.integers(0, V, n0))]
    v0 = rng.integers(0, 1 << 31, n0).tolist()
    s = torch.cuda.Stream(DEV)
    with torch.cuda.stream(s):
        g = Gpma.gpma_create(V, keys_t(k0), vals_t(v0), delete_mode=mode, stream=s)
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    live = set(k0)
    B = 2 * V                                   # one batch size for every op: replayable
    for step in range(40):
        grow = (step // 10) % 2 == 0
        if grow or not live:
            ks = [(int(a) << 32) | int(b) for a, b in zip(rng.integers(0, V, B), rng.integers(0, V, B))]
            vs = rng.integers(0, 1 << 31, B).tolist()
            g.gpma_update_batch(keys_t(ks), vals_t(vs), 0, stream=s)
            o.insert(ks, vs)
            live.update(ks)
        else:
            pres = sorted(live)
            ks = [pres[i] for i in rng.integers(0, len(pres), B)]
            g.gpma_update_batch(keys_t(ks), None, 1, stream=s)
            o.delete(ks)
            live.difference_update(ks)
        s.synchronize()
        assert_same_layout(g, o, what=f"seed {seed} step {step}")
    assert_same_csr(g, o)


@pytest.mark.parametrize("small", ["0", "1", "2"])
@pytest.mark.parametrize("mode", [0, 1])
def test_level_step_paths(small, mode):
    """Levels >= 1 through the single-CTA small-level front/back with the fused per-window
    merge (GPMA_LVL_SMALL=2, default), front/back only (1) and the multi-kernel step (0):
    layouts and per-level traces (segments, offsets,
    flags of every round, Alg. 4 l.7-25) equal the oracle's on configs[0] sliding windows and
    on random batches that climb to the root and resize."""
    from tests.test_gpu_parity import _slide_parity, test_random_small_with_resizes
    with env(GPMA_LVL_SMALL=small):
        _slide_parity(2, mode, analytics=False, trace=True)
        test_random_small_with_resizes(3, mode)
