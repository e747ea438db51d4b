"""Sharded (multi-GPU) path on the GPU: CUDA shards + DistGpma orchestration.

Two processes share one B200 through a gloo group (NCCL refuses two ranks on one device);
every shard's layout must equal an oracle shard fed the same owned batches (bit-exact), and
the distributed BFS / CC / PageRank must equal the single-store oracle.  A world-size-1 run
covers the P = 1 path of the same code.
"""
import os
import socket

import numpy as np
import pytest
import torch

import oracle as O
from gpma_gen import bfs_root, config_stream

pytestmark = pytest.mark.gpu


def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def _owned(keys, vals, V, P, r):
    src = keys >> 32
    m = (src // ((V + P - 1) // P)) == r
    return keys[m], (None if vals is None else vals[m])


def _run(rank, world, port, mode, seed, fails):
    import torch.distributed as dist
    from paper_journals_pvldb_shalht17_b200.dist import CudaShard, DistGpma, batch_slice, row_range
    from tests.gpu_helpers import DEV, assert_pr_close, assert_same_layout
    try:
        if world > 1:
            os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
            dist.init_process_group("gloo", rank=rank, world_size=world)
        torch.cuda.set_device(0)
        sw = config_stream(0, seed=seed)
        V, W, B = 1024, sw.window, sw.batch
        k0, v0 = sw.initial()
        rows = row_range(V, world, rank)
        lo, hi = batch_slice(W, world, rank)
        shard = CudaShard(V, rows, DEV, delete_mode=mode)
        dg = DistGpma(V, k0[lo:hi].contiguous().to(DEV), v0[lo:hi].contiguous().to(DEV), shard)
        ok0, ov0 = _owned(k0, v0, V, world, rank)
        osh = O.Oracle(V, ok0, ov0, rows=rows, delete_mode=mode)
        ref = O.Oracle(V, k0, v0, delete_mode=mode)
        assert_same_layout(shard.g, osh, what=f"rank {rank} create")
        x = None
        for s in range(3):
            dk, ik, iv = sw.slide(s)
            a, b = batch_slice(B, world, rank)
            dg.delete(dk[a:b].contiguous().to(DEV))
            dg.insert(ik[a:b].contiguous().to(DEV), iv[a:b].contiguous().to(DEV))
            osh.delete(_owned(dk, None, V, world, rank)[0])
            osh.insert(*_owned(ik, iv, V, world, rank))
            ref.delete(dk)
            ref.insert(ik, iv)
            assert_same_layout(shard.g, osh, what=f"rank {rank} slide {s}")
            root = bfs_root(sw, seed, s)
            assert dg.bfs(root).cpu().numpy().tolist() == ref.bfs(root).tolist(), "BFS"
            assert dg.cc().cpu().numpy().view(np.uint32).tolist() == ref.cc().tolist(), "CC"
            xt = None if x is None else torch.from_numpy(x.copy()).to(DEV)
            xg, it = dg.pagerank(xt, warm=x is not None, tol=0.0, max_iter=6)
            xo, _ = ref.pagerank(x=x, tol=0.0, max_iter=6)
            assert it == 6
            assert_pr_close(xg.cpu().numpy(), xo, what="dist PR")
            x = xo
        if world > 1:
            dist.destroy_process_group()
    except Exception as e:
        import traceback
        fails.put(f"rank {rank}: {e!r}\n{traceback.format_exc()}")
        raise


@pytest.mark.parametrize("mode,seed", [(0, 5), (1, 6)])
def test_two_shards_one_gpu(mode, seed):
    import torch.multiprocessing as mp
    ctx = mp.get_context("spawn")
    fails = ctx.Queue()
    mp.spawn(_run, args=(2, _free_port(), mode, seed, fails), nprocs=2, join=True)
    assert fails.empty()


def test_world_size_one_path():
    import queue
    q = queue.Queue()
    _run(0, 1, 0, 0, 9, q)
    assert q.empty()


def test_exchange_primitives_against_their_definitions():
    """gpma_bfs_bits / gpma_bfs_merge / gpma_pr_update_rows (include/gpma.h) on a shard handle,
    element by element against their plain definitions."""
    from paper_journals_pvldb_shalht17_b200 import Gpma
    from tests.gpu_helpers import DEV, keys_t, vals_t
    V, P, r = 1000, 3, 1                                  # ragged: V not a multiple of 32 or P
    chunk = (V + P - 1) // P
    lo, hi = r * chunk, min(V, (r + 1) * chunk)
    rng = np.random.default_rng(9)
    src = rng.integers(lo, hi, 3000, dtype=np.uint64)
    dst = rng.integers(0, V, 3000, dtype=np.uint64)
    keys = np.unique((src << np.uint64(32)) | dst)
    g = Gpma.gpma_create(V, keys_t(keys), vals_t(np.zeros(keys.size, np.uint32)), rows=(lo, hi))
    words = (V + 31) // 32
    # bits: levels == depth
    lv = rng.integers(-1, 4, V).astype(np.int32)
    bm = torch.zeros(words, dtype=torch.int32, device=DEV)
    g.gpma_bfs_bits(torch.from_numpy(lv).to(DEV), 2, bm)
    want = np.packbits(np.concatenate([lv == 2, np.zeros(words * 32 - V, bool)]), bitorder="little")
    assert np.array_equal(bm.cpu().numpy().view(np.uint8), want)
    # merge: unreached and set in any bitmap -> depth
    bms = rng.integers(0, 1 << 32, (P, words), dtype=np.uint64).astype(np.uint32)
    lvt = torch.from_numpy(lv).to(DEV)
    g.gpma_bfs_merge(lvt, torch.from_numpy(bms.view(np.int32)).to(DEV), P, 7)
    anyb = np.unpackbits(np.bitwise_or.reduce(bms, axis=0).view(np.uint8), bitorder="little")[:V].astype(bool)
    exp = lv.copy()
    exp[anyb & (lv == -1)] = 7
    assert np.array_equal(lvt.cpu().numpy(), exp)
    # owned-rows PageRank update from reduced sums (2^-62 fixed point) + the dangling total
    S = float(2 ** 62)
    x = rng.random(V)
    yr = rng.integers(0, 1 << 50, hi - lo + 1, dtype=np.uint64)
    xt = torch.from_numpy(x.copy()).to(DEV)
    err = g.gpma_pr_update_rows(xt, torch.from_numpy(yr.view(np.int64)).to(DEV), 0.85)
    nx = (1 - 0.85) / V + 0.85 * (yr[:-1].astype(np.float64) / S + float(yr[-1]) / S / V)
    got = xt.cpu().numpy()
    assert np.abs(got[lo:hi] - nx).max() <= 1e-15
    assert np.array_equal(got[:lo], x[:lo]) and np.array_equal(got[hi:], x[hi:])
    assert abs(err - np.abs(nx - x[lo:hi]).sum()) <= 1e-9


@pytest.mark.parametrize("mode", [0, 1])
def test_dist_handle_nccl_world_one(mode):
    """gpma_dist_create: the library's own NCCL communicator at world size 1 -- the
    validated routing, the collective BFS / CC / PageRank, the all-gather of x -- through the
    C ABI, against the single-store oracle (bit-exact layout; PR scale-aware), and a batch with
    one bad key rejected before anything mutates."""
    from paper_journals_pvldb_shalht17_b200 import Gpma, GpmaError
    from tests.gpu_helpers import DEV, assert_pr_close, assert_same_layout, keys_t, vals_t
    sw = config_stream(0, seed=31 + mode)
    V = 1024
    k0, v0 = sw.initial()
    uid = Gpma.gpma_dist_unique_id()
    g = Gpma.gpma_dist_create(uid, 0, 1, V, k0.to(DEV), v0.to(DEV), delete_mode=mode)
    assert g.gpma_dist_info() == {"rank": 0, "nranks": 1, "row_begin": 0, "row_end": V}
    o = O.Oracle(V, k0, v0, delete_mode=mode)
    assert_same_layout(g, o, what="dist create")
    x = None
    for s in range(3):
        dk, ik, iv = sw.slide(s)
        g.delete(dk.to(DEV))
        g.insert(ik.to(DEV), iv.to(DEV))
        o.delete(dk)
        o.insert(ik, iv)
        assert_same_layout(g, o, what=f"dist slide {s}")
        root = bfs_root(sw, 31, s)
        lv = torch.empty(V, dtype=torch.int32, device=DEV)
        g.gpma_bfs(root, lv)
        assert np.array_equal(lv.cpu().numpy(), o.bfs(root)), "dist BFS"
        lab = torch.empty(V, dtype=torch.int32, device=DEV)
        g.gpma_cc(lab)
        assert np.array_equal(lab.cpu().numpy().view(np.uint32), o.cc()), "dist CC"
        xt = torch.empty(V, dtype=torch.float64, device=DEV) if x is None else torch.from_numpy(x.copy()).to(DEV)
        it = g.gpma_pagerank(xt, warm_start=x is not None, tol_l1=0.0, max_iter=6)
        xo, _ = o.pagerank(x=x, tol=0.0, max_iter=6)
        assert it == 6
        assert_pr_close(xt.cpu().numpy(), xo, what="dist PR")
        x = xo
    bad = keys_t([(3 << 32) | 5, (V + 7) << 32])
    assert g.gpma_update_batch(bad, vals_t([1, 2]), 0, check=False) == 2     # RANGE, nothing applied
    assert_same_layout(g, o, what="after a rejected dist batch")
    g.gpma_destroy()
