"""Query buffer (§3) on the GPU vs the oracle / brute force."""
import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import config_stream
from tests.gpu_helpers import DEV, keys_t

pytestmark = pytest.mark.gpu


def _store(seed=2, mode=0):
    from paper_journals_pvldb_shalht17_b200 import Gpma
    sw = config_stream(0, seed=seed)
    V = 1024
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.to(DEV), v0.to(DEV), delete_mode=mode)
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    dk, ik, iv = sw.slide(0)
    g.delete(dk.to(DEV))
    g.insert(ik.to(DEV), iv.to(DEV))
    o.delete(dk)
    o.insert(ik, iv)
    return sw, g, o, V


def test_edge_lookup_matches_replay():
    sw, g, o, V = _store()
    rp, col, val = o.export_csr()
    live = {}
    for u in range(V):
        for e in range(int(rp[u]), int(rp[u + 1])):
            live[(u << 32) | int(col[e])] = int(val[e])
    rng = np.random.default_rng(0)
    present = list(live)
    deleted = [int(k) for k in sw.slide(0)[0][:200]]           # tombstoned by the slide
    absent = [int(s) << 32 | int(d) for s, d in zip(rng.integers(0, V, 300), rng.integers(0, V, 300))]
    q = [present[i] for i in rng.integers(0, len(present), 500)] + deleted + absent
    vals = torch.empty(len(q), dtype=torch.int32, device=DEV)
    found = torch.empty(len(q), dtype=torch.uint8, device=DEV)
    g.gpma_query_edges(keys_t(q), vals, found)
    fv = vals.cpu().numpy().view(np.uint32)
    ff = found.cpu().numpy()
    for i, k in enumerate(q):
        assert ff[i] == (k in live)
        assert fv[i] == live.get(k, 0xFFFFFFFF)


def test_neighbors_match_csr_rows():
    sw, g, o, V = _store(seed=4)
    rp, col, val = o.export_csr()
    rng = np.random.default_rng(1)
    verts = np.concatenate([rng.integers(0, V, 200), [0, 0, V - 1]]).astype(np.uint32)
    vt = torch.as_tensor(verts.view(np.int32)).to(DEV)
    nnz = g.gpma_query_neighbors(vt)
    out_rp = torch.empty(len(verts) + 1, dtype=torch.int64, device=DEV)
    out_c = torch.empty(max(nnz, 1), dtype=torch.int32, device=DEV)
    out_v = torch.empty(max(nnz, 1), dtype=torch.int32, device=DEV)
    assert g.gpma_query_neighbors(vt, out_rp, out_c, out_v) == nnz
    grp = out_rp.cpu().numpy()
    gc = out_c.cpu().numpy().view(np.uint32)
    gv = out_v.cpu().numpy().view(np.uint32)
    for i, u in enumerate(verts):
        a, b = int(rp[u]), int(rp[u + 1])
        assert gc[grp[i]:grp[i + 1]].tolist() == col[a:b].tolist()
        assert gv[grp[i]:grp[i + 1]].tolist() == val[a:b].tolist()


@pytest.mark.parametrize("seed", [5, 6])
def test_reachability_matches_bfs(seed):
    sw, g, o, V = _store(seed=seed)
    rng = np.random.default_rng(seed)
    src = rng.integers(0, V, 150).astype(np.uint32)
    dst = rng.integers(0, V, 150).astype(np.uint32)
    dst[:5] = src[:5]                                          # reflexive pairs
    out = torch.empty(150, dtype=torch.uint8, device=DEV)
    g.gpma_query_reachable(torch.as_tensor(src.view(np.int32)).to(DEV),
                           torch.as_tensor(dst.view(np.int32)).to(DEV), out)
    got = out.cpu().numpy()
    cache = {}
    for i, (s, t) in enumerate(zip(src, dst)):
        if s not in cache:
            cache[s] = o.bfs(int(s))
        assert got[i] == (cache[s][t] >= 0), (i, s, t)


def test_reachability_closed_form_path():
    from paper_journals_pvldb_shalht17_b200 import Gpma
    n = 40                                                     # path 0 -> 1 -> ... -> n-1
    keys = [(i << 32) | (i + 1) for i in range(n - 1)]
    g = Gpma.gpma_create(n, keys_t(keys), torch.zeros(n - 1, dtype=torch.int32, device=DEV))
    src = torch.tensor([0, 5, 39, 10], dtype=torch.int32, device=DEV)
    dst = torch.tensor([39, 2, 39, 11], dtype=torch.int32, device=DEV)
    out = torch.empty(4, dtype=torch.uint8, device=DEV)
    g.gpma_query_reachable(src, dst, out)
    assert out.cpu().tolist() == [1, 0, 1, 1]
