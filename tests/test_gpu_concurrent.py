"""Concurrent read-only analytics (include/gpma.h "Concurrency"; fanout.py): BFS, CC, PageRank,
export and the query buffer run at the same time on five streams from five host threads, over
a store large enough for multi-tile scans, the dense BFS sweep and multi-round CC; every result
must equal the oracle's, repeatedly (a shared scratch buffer would corrupt one of them)."""
import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import bfs_root, config_stream
from gpma_gen.streams import StreamConfig
from tests.gpu_helpers import DEV, assert_pr_close

pytestmark = pytest.mark.gpu


def test_concurrent_analytics_match_oracle():
    from paper_journals_pvldb_shalht17_b200 import Gpma
    from paper_journals_pvldb_shalht17_b200.fanout import AnalyticsFanout
    cfg = StreamConfig("rmat-s16", "rmat", 1 << 16, 1 << 20, 1 << 19, 1 << 15, 0x5EED, scale=16)
    sw = config_stream(cfg, device=DEV)
    sw.keys, sw.vals = sw.keys.cpu(), sw.vals.cpu()
    V = 1 << 16
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV))
    o = O.Oracle(V, k0, v0)
    fan = AnalyticsFanout(DEV, n=5)
    s = torch.cuda.Stream(DEV)
    nnz_cap = sw.window + sw.batch
    lv = torch.empty(V, dtype=torch.int32, device=DEV)
    lab = torch.empty(V, dtype=torch.int32, device=DEV)
    x = torch.empty(V, dtype=torch.float64, device=DEV)
    rp = torch.empty(V + 1, dtype=torch.int64, device=DEV)
    col = torch.empty(nnz_cap, dtype=torch.int32, device=DEV)
    cv = torch.empty(nnz_cap, dtype=torch.int32, device=DEV)
    rng = np.random.default_rng(3)
    qsrc = rng.integers(0, V, 64).astype(np.uint32)
    qdst = rng.integers(0, V, 64).astype(np.uint32)
    qs = torch.as_tensor(qsrc.view(np.int32)).to(DEV)
    qd = torch.as_tensor(qdst.view(np.int32)).to(DEV)
    reach = torch.empty(64, dtype=torch.uint8, device=DEV)
    for step in range(3):
        dk, ik, iv = sw.slide(step)
        with torch.cuda.stream(s):
            g.gpma_update_batch(dk.to(DEV), None, 1, stream=s)
            g.gpma_update_batch(ik.to(DEV), iv.to(DEV), 0, stream=s)
        o.delete(dk)
        o.insert(ik, iv)
        root = bfs_root(sw, 1, step)
        for rep in range(3):
            r = fan.run(s, [
                lambda st: g.gpma_pagerank(x, warm_start=False, tol_l1=0.0, max_iter=5, stream=st),
                lambda st: g.gpma_cc(lab, stream=st),
                lambda st: g.gpma_bfs(root, lv, stream=st),
                lambda st: g.gpma_export_csr(rp, col, cv, stream=st),
                lambda st: g.gpma_query_reachable(qs, qd, reach, stream=st)])
            s.synchronize()
            ob = o.bfs(root)
            assert np.array_equal(lv.cpu().numpy(), ob), (step, rep)
            assert np.array_equal(lab.cpu().numpy().view(np.uint32), o.cc()), (step, rep)
            xo, _ = o.pagerank(tol=0.0, max_iter=5)
            assert r[0] == 5, (step, rep)
            assert_pr_close(x.cpu().numpy(), xo, what=f"{step} {rep}")
            orp, ocol, oval = o.export_csr()
            assert r[3] == len(ocol)
            assert np.array_equal(rp.cpu().numpy().view(np.uint64), orp)
            assert np.array_equal(col.cpu().numpy().view(np.uint32)[: len(ocol)], ocol)
            assert np.array_equal(cv.cpu().numpy().view(np.uint32)[: len(ocol)], oval)
            want = [(o.bfs(int(a))[int(b)] >= 0) for a, b in zip(qsrc[:8], qdst[:8])]
            assert reach.cpu().numpy()[:8].astype(bool).tolist() == want, (step, rep)
    fan.close()
