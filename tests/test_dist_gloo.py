"""World-size-2 gloo tests of the sharded (multi-GPU) path on CPU.

The orchestration and collectives of `DistGpma` (routing all-to-all-v, MAX/MIN/SUM all-reduces,
loop termination) run for real over a 2-rank gloo group; each rank's compute is the oracle-backed
emulation of tests/dist_oracle.py.  Results must equal the single-store oracle: edge set (union of
the shard CSRs), BFS levels, CC labels (bit-exact) and PageRank (fixed K, 1e-12).
"""
import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle as O
from gpma_gen import bfs_root, config_stream
from paper_journals_pvldb_shalht17_b200.dist import DistGpma, batch_slice, owner_of, row_range


def _free_port():
    with socket.socket() as s:
        s.bind(("127.0.0.1", 0))
        return s.getsockname()[1]


def _worker(rank, world, port, mode, seed, fails):
    try:
        os.environ.update(MASTER_ADDR="127.0.0.1", MASTER_PORT=str(port))
        dist.init_process_group("gloo", rank=rank, world_size=world)
        from tests.dist_oracle import OracleShard
        sw = config_stream(0, seed=seed)
        V = 1024
        W, B = sw.window, sw.batch
        k0, v0 = sw.initial()
        lo, hi = batch_slice(W, world, rank)
        shard = OracleShard(V, row_range(V, world, rank), delete_mode=mode)
        dg = DistGpma(V, k0[lo:hi].contiguous(), v0[lo:hi].contiguous(), shard)
        ref = O.Oracle(V, k0, v0, delete_mode=mode)
        x = None
        for s in range(3):
            dk, ik, iv = sw.slide(s)
            a, b = batch_slice(B, world, rank)
            dg.delete(dk[a:b].contiguous())
            dg.insert(ik[a:b].contiguous(), iv[a:b].contiguous())
            ref.delete(dk)
            ref.insert(ik, iv)
            # edge set: the shards' rows concatenate to the single-store CSR
            rp, col, val = shard.o.export_csr()
            parts = [None] * world
            dist.all_gather_object(parts, (rp.tolist(), col.tolist(), val.tolist()))
            grp, gcol, gval = ref.export_csr()
            cat_col = sum((p[1] for p in parts), [])
            cat_val = sum((p[2] for p in parts), [])
            assert cat_col == gcol.tolist() and cat_val == gval.tolist()
            lo_r, hi_r = row_range(V, world, rank)
            assert (np.array(rp) + grp[lo_r]).tolist() == grp[lo_r:hi_r + 1].tolist()
            root = bfs_root(sw, seed, s)
            assert dg.bfs(root).numpy().tolist() == ref.bfs(root).tolist()
            assert dg.cc().numpy().view(np.uint32).tolist() == ref.cc().tolist()
            xt = None if x is None else torch.from_numpy(x.copy())
            xg, it = dg.pagerank(xt, warm=x is not None, tol=0.0, max_iter=6)
            xo, _ = ref.pagerank(x=x, tol=0.0, max_iter=6)
            assert it == 6 and np.abs(xg.numpy() - xo).max() < 1e-12
            x = xo
        # a bad key on ONE rank rejects the batch on every rank, nothing applied anywhere
        before = shard.o.dump()
        bad = torch.tensor([(V + 3) << 32 | 1] if rank == world - 1 else [], dtype=torch.int64)
        from paper_journals_pvldb_shalht17_b200.gpma import GpmaError
        try:
            dg.insert(bad, torch.ones(bad.numel(), dtype=torch.int32))
            raise AssertionError("the bad batch was accepted")
        except GpmaError as e:
            assert e.status == 2
        after = shard.o.dump()
        assert (before[0] == after[0]).all() and (before[1] == after[1]).all()
        # tolerance mode: the same stopping iteration as the single store
        xg, it = dg.pagerank(None, warm=False, tol=1e-3, max_iter=100)
        xo, ito = ref.pagerank(tol=1e-3, max_iter=100)
        assert it == ito and np.abs(xg.numpy() - xo).max() < 1e-12
        dist.destroy_process_group()
    except Exception as e:  # surface the failure to the parent
        import traceback
        fails.put(f"rank {rank}: {e!r}\n{traceback.format_exc()}")
        raise


@pytest.mark.parametrize("mode,seed", [(O.LAZY, 3), (O.REBALANCE, 4)])
def test_two_rank_gloo_matches_single_store(mode, seed):
    ctx = mp.get_context("spawn")
    fails = ctx.Queue()
    mp.spawn(_worker, args=(2, _free_port(), mode, seed, fails), nprocs=2, join=True)
    assert fails.empty()


@pytest.mark.parametrize("world,seed", [(3, 7), (4, 8)])
def test_ragged_shards_gloo_matches_single_store(world, seed):
    """World size 3 and 4: V = 1024 splits into unequal row ranges (342/342/340, 256 x 4), batch
    slices of unequal length; lazy deletes."""
    ctx = mp.get_context("spawn")
    fails = ctx.Queue()
    mp.spawn(_worker, args=(world, _free_port(), O.LAZY, seed, fails), nprocs=world, join=True)
    assert fails.empty()


def test_owner_and_slices():
    V, P = 1000, 3
    assert [row_range(V, P, r) for r in range(P)] == [(0, 334), (334, 668), (668, 1000)]
    assert int(owner_of(torch.tensor([0, 333, 334, 999]), V, P).tolist()[-1]) == 2
    assert [batch_slice(10, 3, r) for r in range(3)] == [(0, 3), (3, 6), (6, 10)]
