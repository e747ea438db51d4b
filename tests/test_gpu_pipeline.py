"""NEXT-1: the transfer-hiding pipeline (Fig. 2) returns the same results as the
plain calls: layouts/analytics of every slide equal the oracle's."""
import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import bfs_root, config_stream
from tests.gpu_helpers import DEV, assert_pr_close

pytestmark = pytest.mark.gpu


@pytest.mark.parametrize("concurrent", [False, True])
def test_pipeline_matches_oracle(concurrent):
    from paper_journals_pvldb_shalht17_b200 import Gpma
    from paper_journals_pvldb_shalht17_b200.pipeline import SlidingWindowPipeline
    seed = 8
    sw = config_stream(0, seed=seed)
    V = 1024
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV))
    o = O.Oracle(V, k0, v0)
    pipe = SlidingWindowPipeline(g, V, sw.batch, sw.window + sw.batch, DEV, pr_tol=0.0, concurrent=concurrent)
    xo, _ = o.pagerank(tol=0.0, max_iter=100)
    batches = [tuple(t.contiguous().pin_memory() for t in sw.slide(s)) for s in range(4)]
    pipe.stage(0, *batches[0])
    for s in range(4):
        if s + 1 < 4:
            pipe.stage((s + 1) % 2, *batches[s + 1])
        pipe.run(s % 2, bfs_root(sw, seed, s))
        dk, ik, iv = sw.slide(s)
        o.delete(dk)
        o.insert(ik, iv)
        lv, lab, rp, col, cv, x = pipe.results(s % 2)
        assert np.array_equal(lv.numpy(), o.bfs(bfs_root(sw, seed, s)))
        assert np.array_equal(lab.numpy().view(np.uint32), o.cc())
        orp, ocol, oval = o.export_csr()
        assert np.array_equal(rp.numpy().view(np.uint64), orp)
        assert np.array_equal(col.numpy().view(np.uint32), ocol)
        assert np.array_equal(cv.numpy().view(np.uint32), oval)
        xo, _ = o.pagerank(x=xo, tol=0.0, max_iter=100)
        assert_pr_close(x.numpy(), xo, what=f"slide {s}")
    pipe.drain()
    pipe.close()
