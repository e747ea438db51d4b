"""BFS level strategies vs the oracle's textbook BFS (Alg. 2): the dense-level
sweep (active-leaf list + sweep of those leaves) and the sparse row expansion (Alg. 3,
P:679-684), each forced on every level via GPMA_BFS_SPARSE, on RMAT graphs with tombstones
(lazy deletes) and several roots.  Levels are unique: bit-exact."""
import contextlib
import os

import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import config_stream, bfs_root
from tests.gpu_helpers import DEV, gpu_bfs

pytestmark = pytest.mark.gpu

if torch.cuda.is_available():
    from paper_journals_pvldb_shalht17_b200 import Gpma


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


def _store(scale):
    if scale == 10:
        sw = config_stream(0, seed=3)
    else:
        from gpma_gen.streams import StreamConfig
        cfg = StreamConfig("rmat-s16", "rmat", 1 << 16, 1 << 20, 1 << 19, 1 << 15, 0x5EED, scale=16)
        sw = config_stream(cfg, device=DEV)
        sw.keys, sw.vals = sw.keys.cpu(), sw.vals.cpu()
    V = 1 << scale
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV))
    o = O.Oracle(V, k0, v0)
    for s in range(2):
        dk, ik, iv = sw.slide(s)
        g.delete(dk.to(DEV))
        g.insert(ik.to(DEV), iv.to(DEV))
        o.delete(dk)
        o.insert(ik, iv)
    return sw, g, o


@pytest.mark.parametrize("scale", [10, 16])
def test_bfs_every_strategy(scale):
    sw, g, o = _store(scale)
    roots = [bfs_root(sw, 7, s) for s in range(3)] + [0]
    for root in roots:
        want = o.bfs(root)
        for sparse in ("0", "1", "100000000"):          # all dense / only F=1 sparse / all sparse
            with env(GPMA_BFS_SPARSE=sparse):
                got = gpu_bfs(g, root)
            assert np.array_equal(got, want), f"root {root} sparse {sparse}"


@pytest.mark.parametrize("scale", [10, 16])
def test_cc_every_sample_strategy(scale):
    """CC (Soman et al.; R19 weak components, min-id labels) with every first-round
    sample: slot sweep (0), first one / two edges per row (1, 2)."""
    sw, g, o = _store(scale)
    want = o.cc()
    from tests.gpu_helpers import gpu_cc
    for mode in ("0", "1", "2"):
        for l1 in ("0", "1", "2"):                      # find() chains through L1: never / sample / all
            with env(GPMA_CC_SAMPLE=mode, GPMA_CC_L1=l1):
                got = gpu_cc(g)
            assert np.array_equal(got, want), f"sample mode {mode} L1 mode {l1}"
