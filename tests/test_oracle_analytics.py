"""Pin the oracle's BFS / CC / PageRank to library routines and closed forms."""
import numpy as np
import pytest
import scipy.sparse as sp
from scipy.sparse import csgraph

import oracle as O


def _csr_from_edges(V, edges):
    edges = sorted(set(edges))
    rp = np.zeros(V + 1, np.uint64)
    for s, _ in edges:
        rp[s + 1] += 1
    rp = np.cumsum(rp).astype(np.uint64)
    col = np.array([d for _, d in edges], np.uint32)
    return rp, col


def _rand_graph(V, E, seed):
    rng = np.random.default_rng(seed)
    return list({(int(a), int(b)) for a, b in zip(rng.integers(0, V, E), rng.integers(0, V, E))})


@pytest.mark.parametrize("seed", range(10))
def test_bfs_matches_scipy(seed):
    V = 60
    edges = _rand_graph(V, 90, seed)
    rp, col = _csr_from_edges(V, edges)
    A = sp.csr_matrix((np.ones(len(col)), col.astype(np.int64), rp.astype(np.int64)), shape=(V, V))
    root = int(edges[0][0])
    lv = O.bfs_csr(V, rp, col, root)
    dist = csgraph.shortest_path(A, directed=True, unweighted=True, indices=root)
    want = np.where(np.isinf(dist), -1, dist).astype(np.int32)
    assert lv.tolist() == want.tolist()


def test_bfs_closed_forms():
    n = 10
    rp, col = _csr_from_edges(n + 2, [(i, i + 1) for i in range(n - 1)])  # path 0..n-1, 2 isolated
    lv = O.bfs_csr(n + 2, rp, col, 0)
    assert lv.tolist() == list(range(n)) + [-1, -1]
    rp, col = _csr_from_edges(6, [(0, i) for i in range(1, 6)])          # out-star
    assert O.bfs_csr(6, rp, col, 0).tolist() == [0, 1, 1, 1, 1, 1]
    assert O.bfs_csr(6, rp, col, 3).tolist() == [-1, -1, -1, 0, -1, -1]


@pytest.mark.parametrize("seed", range(10))
def test_cc_matches_scipy_weak(seed):
    V = 80
    edges = _rand_graph(V, 50, seed)
    rp, col = _csr_from_edges(V, edges)
    A = sp.csr_matrix((np.ones(len(col)), col.astype(np.int64), rp.astype(np.int64)), shape=(V, V))
    ncomp, lab = csgraph.connected_components(A, directed=True, connection="weak")
    want = np.zeros(V, np.int64)
    for c in range(ncomp):
        members = np.nonzero(lab == c)[0]
        want[members] = members.min()
    assert O.cc_csr(V, rp, col).tolist() == want.tolist()


def test_cc_closed_forms():
    # three disjoint directed cliques {0,3,6}, {1,4}, {2,5,7}; vertex 8 isolated
    groups = [[6, 3, 0], [4, 1], [7, 5, 2]]
    edges = [(a, b) for g in groups for a in g for b in g if a != b]
    rp, col = _csr_from_edges(9, edges)
    assert O.cc_csr(9, rp, col).tolist() == [0, 1, 2, 0, 1, 2, 0, 2, 8]
    # direction is ignored (weak components): a chain pointing "down" the ids
    rp, col = _csr_from_edges(4, [(3, 2), (2, 1), (1, 0)])
    assert O.cc_csr(4, rp, col).tolist() == [0, 0, 0, 0]


def _google_pagerank(V, edges, d=0.85):
    """Principal eigenvector of the Google matrix (dangling mass spread uniformly)."""
    M = np.zeros((V, V))
    out = np.zeros(V)
    for s, _ in edges:
        out[s] += 1
    for s, t in edges:
        M[t, s] += 1.0 / out[s]
    for s in range(V):
        if out[s] == 0:
            M[:, s] = 1.0 / V
    G = d * M + (1 - d) / V * np.ones((V, V))
    w, vecs = np.linalg.eig(G)
    x = np.real(vecs[:, np.argmax(np.real(w))])
    return x / x.sum()


@pytest.mark.parametrize("seed", range(8))
def test_pagerank_matches_eigenvector(seed):
    V = 40
    edges = _rand_graph(V, 120, seed)
    rp, col = _csr_from_edges(V, edges)
    x, it = O.pagerank_csr(V, rp, col, tol=1e-13, max_iter=2000)
    assert it < 2000
    np.testing.assert_allclose(x, _google_pagerank(V, edges), atol=1e-10)
    assert abs(x.sum() - 1.0) < 1e-12


def test_pagerank_closed_forms():
    n = 7
    rp, col = _csr_from_edges(n, [(i, (i + 1) % n) for i in range(n)])    # directed cycle
    x, _ = O.pagerank_csr(n, rp, col, tol=0.0, max_iter=50)
    np.testing.assert_allclose(x, np.full(n, 1.0 / n), atol=1e-15)
    rp, col = _csr_from_edges(5, [])                                       # edgeless
    x, _ = O.pagerank_csr(5, rp, col, tol=0.0, max_iter=3)
    np.testing.assert_allclose(x, np.full(5, 0.2), atol=1e-15)
    # star with k leaves -> hub, hub dangling: x_leaf = (1-d)/V + d*x_hub/V,
    # x_hub = (1-d)/V + d*(k*x_leaf + x_hub/V)
    k, d = 6, 0.85
    V = k + 1
    rp, col = _csr_from_edges(V, [(i, 0) for i in range(1, V)])
    x, _ = O.pagerank_csr(V, rp, col, tol=1e-15, max_iter=5000)
    A = np.array([[1 - d / V, -d * k], [-d / V, 1.0]])
    b = np.array([(1 - d) / V, (1 - d) / V])
    hub, leaf = np.linalg.solve(A, b)
    np.testing.assert_allclose(x[0], hub, atol=1e-12)
    np.testing.assert_allclose(x[1:], leaf, atol=1e-12)


def test_pagerank_tolerance_and_warm_start():
    """Stop after the first iteration whose L1 change < tol; warm start."""
    V = 50
    edges = _rand_graph(V, 200, 1)
    rp, col = _csr_from_edges(V, edges)
    x_cold, it_cold = O.pagerank_csr(V, rp, col, tol=1e-3, max_iter=100)
    # recompute the L1 changes by hand: the iteration count is the first below tol
    xs, it = [np.full(V, 1.0 / V)], 0
    while True:
        xn, _ = O.pagerank_csr(V, rp, col, x=xs[-1], tol=0.0, max_iter=1)
        it += 1
        err = np.abs(xn - xs[-1]).sum()
        xs.append(xn)
        if err < 1e-3:
            break
    assert it == it_cold
    np.testing.assert_allclose(x_cold, xs[-1], atol=0)
    x_warm, it_warm = O.pagerank_csr(V, rp, col, x=x_cold, tol=1e-3, max_iter=100)
    assert it_warm <= it_cold


def test_oracle_store_analytics_use_live_edges():
    V = 6
    keys = [(0 << 32) | 1, (1 << 32) | 2, (2 << 32) | 3, (4 << 32) | 5]
    o = O.Oracle(V, keys, [1, 1, 1, 1])
    o.delete([(1 << 32) | 2])                     # tombstone breaks the path
    assert o.bfs(0).tolist() == [0, 1, -1, -1, -1, -1]
    assert o.cc().tolist() == [0, 0, 2, 2, 4, 4]
