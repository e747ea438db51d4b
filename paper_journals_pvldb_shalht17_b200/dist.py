"""Source-range sharded GPMA+ over P ranks, one process per GPU.

PAPER.md P:1693-1705 (§6.4): "We evenly partition graphs according to the vertex index and
synchronize all devices after each iteration."  R24: owner(u) = floor(u / ceil(V/P)); rank r
holds an independent GPMA+ store over its rows (its own guards, capacity, resizes).

Every step of the method runs in libgpma kernels on the rank's shard (`gpma_route`,
`gpma_update_batch`, `gpma_bfs_level`, `gpma_cc_round`, `gpma_pr_push`, `gpma_pr_update`);
this module only sequences them and runs the exchanges, which are collectives of the
caller's torch.distributed process group (NCCL over NVLink on B200; gloo in the CPU tests):

* update: each rank routes its contiguous slice of the global batch by owner (stable) and an
  all-to-all-v delivers the pieces; the rank-order concatenation keeps the global batch order,
  so "last occurrence wins" (R10) is preserved.
* BFS: levels are replicated; each level expands the owned frontier rows, then the ranks
  all-gather their discoveries as bitmaps (V/8 bytes each) and merge them into levels.
* CC: labels are replicated; each round hooks the owned edges on top of them, then
  MIN-all-reduce; stop when no rank changed anything (fixpoint = min-id labels, R19).
* PageRank: each iteration pushes the owned rows into an exact 64-bit fixed-point y (plus the
  owned dangling mass), REDUCE-SCATTERs y to the owners (half an all-reduce's traffic), and
  each rank updates only its owned slice of x (the only one its next push reads); the error
  and the dangling mass are two-word all-reduces; an all-gather of the owned slices returns the
  full vector at the end.
"""
from __future__ import annotations

import math

import torch
import torch.distributed as dist

INSERT, DELETE = 0, 1


def row_range(V: int, P: int, r: int) -> tuple[int, int]:
    """Rows [lo, hi) owned by rank r (R24)."""
    chunk = (V + P - 1) // P
    lo = min(V, r * chunk)
    return lo, min(V, lo + chunk)


def owner_of(src, V: int, P: int):
    return src // ((V + P - 1) // P)


def batch_slice(n: int, P: int, r: int) -> tuple[int, int]:
    """The contiguous slice of a global batch of n keys that rank r ingests."""
    return n * r // P, n * (r + 1) // P


class CudaShard:
    """Per-rank compute: one sharded libgpma store (all method steps in its kernels)."""

    def __init__(self, V: int, rows: tuple[int, int], device, stream=None, **cfg):
        from .gpma import Gpma
        self.Gpma = Gpma
        self.V, self.rows, self.device, self.stream, self.cfg = V, rows, torch.device(device), stream, cfg
        self.g = None
        # a one-row handle serves the routing before the shard exists
        self.router = Gpma.gpma_create(V, None, None, rows=(0, 1), stream=stream)

    def create(self, keys, vals):
        self.g = self.Gpma.gpma_create(self.V, keys, vals, rows=self.rows, stream=self.stream, **self.cfg)

    def route(self, keys, vals, P: int):
        n = keys.numel()
        ok = torch.empty(max(n, 1), dtype=torch.int64, device=self.device)[:n]
        ov = torch.empty(max(n, 1), dtype=torch.int32, device=self.device)[:n]
        h = self.g or self.router
        counts = h.gpma_route(keys, vals, P, ok, ov, stream=self.stream)
        return ok, ov, counts

    def validate(self, keys, vals, op) -> int:
        return (self.g or self.router).gpma_validate_batch(keys, vals if op == INSERT else None, op,
                                                           stream=self.stream)

    def update(self, keys, vals, op):
        self.g.gpma_update_batch(keys, vals if op == INSERT else None, op, stream=self.stream)

    def vertex_array(self, n, dtype):
        return torch.empty(n, dtype=dtype, device=self.device)

    def bfs_init(self, root, levels):
        self.g.gpma_bfs_init(root, levels, stream=self.stream)

    def bfs_level(self, levels, depth) -> int:
        return self.g.gpma_bfs_level(levels, depth, stream=self.stream)

    def cc_round(self, labels, init) -> int:
        return self.g.gpma_cc_round(labels, init, stream=self.stream)

    def pr_push(self, x, init, y):
        self.g.gpma_pr_push(x, init, y, stream=self.stream)

    def pr_update(self, x, y, damping) -> float:
        return self.g.gpma_pr_update(x, y, damping, stream=self.stream)

    def pr_update_rows(self, x, y_rows, damping) -> float:
        return self.g.gpma_pr_update_rows(x, y_rows, damping, stream=self.stream)

    def pr_update_rows_dev(self, x, y_rows, damping, err_dev):
        """err_dev (device double[1]) += the owned rows' L1 change; no host synchronisation."""
        self.g.gpma_pr_update_rows_dev(x, y_rows, err_dev, damping, stream=self.stream)

    def bfs_bits(self, levels, depth, bitmap):
        self.g.gpma_bfs_bits(levels, depth, bitmap, stream=self.stream)

    def bfs_merge(self, levels, bitmaps, n, depth):
        self.g.gpma_bfs_merge(levels, bitmaps, n, depth, stream=self.stream)

    def sync(self):
        if self.device.type == "cuda":
            (self.stream or torch.cuda.current_stream(self.device)).synchronize()


class DistGpma:
    """One rank's view of a source-range sharded GPMA+ store.  All methods are collective."""

    def __init__(self, V: int, init_keys, init_vals, shard, group=None):
        self.V = V
        self.group = group
        self.P = dist.get_world_size(group) if dist.is_initialized() else 1
        self.r = dist.get_rank(group) if dist.is_initialized() else 0
        self.rows = row_range(V, self.P, self.r)
        self.shard = shard
        self._cpu_coll = self.P > 1 and dist.get_backend(group) == "gloo"
        k, v = self._exchange(init_keys, init_vals)
        shard.create(k, v)

    # ---- collectives (gloo runs them on host copies)
    def _dev(self, t):
        return t.cpu() if self._cpu_coll else t

    def _back(self, t, like):
        if t is like:
            return like
        like.copy_(t.to(like.device))
        return like

    def _all_reduce(self, t, op):
        if self.P == 1:
            return t
        h = self._dev(t)
        dist.all_reduce(h, op=op, group=self.group)
        return self._back(h, t)

    def _all_gather(self, out, t):
        """out (P * t.numel()) := the ranks' t, back to back."""
        if self.P == 1:
            out.copy_(t)
            return out
        if self._cpu_coll:                  # gloo: list all-gather of host copies
            parts = [torch.empty_like(self._dev(t)) for _ in range(self.P)]
            dist.all_gather(parts, self._dev(t).contiguous(), group=self.group)
            return self._back(torch.cat(parts), out)
        dist.all_gather_into_tensor(out, t.contiguous(), group=self.group)
        return out

    def _reduce_scatter(self, out, t):
        """out (t.numel() / P) := this rank's slice of the element-wise SUM of the ranks' t."""
        if self._cpu_coll:                  # gloo has no reduce-scatter: all-reduce, keep the slice
            h = self._dev(t).clone()
            dist.all_reduce(h, group=self.group)
            n = out.numel()
            return self._back(h[self.r * n:(self.r + 1) * n], out)
        dist.reduce_scatter_tensor(out, t, group=self.group)
        return out

    def _exchange(self, keys, vals):
        """Route this rank's slice by owner and all-to-all-v it: returns the owned batch."""
        if self.P == 1:
            return keys, vals
        ok, ov, counts = self.shard.route(keys, vals, self.P)
        self.shard.sync()
        send = torch.tensor(counts, dtype=torch.int64)
        recv = torch.empty(self.P, dtype=torch.int64)
        if not self._cpu_coll:
            send, recv = send.to(ok.device), recv.to(ok.device)
        dist.all_to_all_single(recv, send, group=self.group)
        rc = [int(c) for c in recv.tolist()]
        sk, sv = self._dev(ok), self._dev(ov)
        rk = torch.empty(sum(rc), dtype=torch.int64, device=sk.device)
        rv = torch.empty(sum(rc), dtype=torch.int32, device=sv.device)
        dist.all_to_all_single(rk, sk, rc, counts, group=self.group)
        dist.all_to_all_single(rv, sv, rc, counts, group=self.group)
        return rk.to(ok.device), rv.to(ok.device)

    # ---- API
    def update_batch(self, keys, vals=None, op: int = INSERT):
        """Apply this rank's contiguous slice of a global batch (collective).  Every rank validates
        its slice and the ranks agree on the worst status (MAX all-reduce) BEFORE anything is
        routed or applied: a bad key anywhere rejects the batch on every rank with the same
        GpmaError, as the single-store contract rejects the whole batch (include/gpma.h)."""
        st = self.shard.validate(keys, vals, op) if self.P > 1 else 0
        if self.P > 1:
            t = torch.tensor([st], dtype=torch.int32)
            if not self._cpu_coll:
                t = t.to(self.shard.device)
            dist.all_reduce(t, op=dist.ReduceOp.MAX, group=self.group)
            st = int(t.item())
            if st:
                from .gpma import GpmaError
                raise GpmaError(st, "distributed update_batch: a rank's slice was rejected (nothing applied)")
        k, v = self._exchange(keys, vals)
        self.shard.update(k, v, op)

    def insert(self, keys, vals):
        self.update_batch(keys, vals, INSERT)

    def delete(self, keys):
        self.update_batch(keys, None, DELETE)

    def bfs(self, root: int, levels=None):
        levels = self.shard.vertex_array(self.V, torch.int32) if levels is None else levels
        self.shard.bfs_init(root, levels)
        words = (self.V + 31) // 32
        bm = self.shard.vertex_array(words, torch.int32)
        bms = self.shard.vertex_array(self.P * words, torch.int32)
        depth = 1
        while True:
            F = self.shard.bfs_level(levels, depth)      # |frontier| of the replicated levels
            if F == 0:
                break
            if self.P > 1:
                self.shard.bfs_bits(levels, depth, bm)   # this rank's discoveries
                self._all_gather(bms, bm)
                self.shard.bfs_merge(levels, bms, self.P, depth)
            depth += 1
        return levels

    def cc(self, labels=None):
        labels = self.shard.vertex_array(self.V, torch.int32) if labels is None else labels
        init = True
        while True:
            changed = self.shard.cc_round(labels, init)
            init = False
            if self.P == 1:
                break                       # one local round is the full answer
            self._all_reduce(labels, dist.ReduceOp.MIN)
            c = torch.tensor([changed], dtype=torch.int64)
            if not self._cpu_coll:
                c = c.to(labels.device)
            dist.all_reduce(c, group=self.group)
            if int(c.item()) == 0:
                break
        return labels

    def pagerank(self, x=None, warm: bool = False, damping: float = 0.85, tol: float = 1e-3,
                 max_iter: int = 100):
        x = self.shard.vertex_array(self.V, torch.float64) if x is None else x
        it = 0
        if self.P == 1:
            y = self.shard.vertex_array(self.V + 1, torch.int64)
            y.zero_()
            while it < max_iter:
                self.shard.pr_push(x, (not warm) and it == 0, y)
                err = self.shard.pr_update(x, y, damping)
                it += 1
                if err < tol:
                    break
            return x, it
        chunk = (self.V + self.P - 1) // self.P
        lo, hi = self.rows
        y = self.shard.vertex_array(chunk * self.P + 1, torch.int64)   # y[V] = dangling mass
        yr = self.shard.vertex_array(chunk + 1, torch.int64)          # owned sums, then the dangling total
        e = self.shard.vertex_array(1, torch.float64)
        y.zero_()
        while it < max_iter:
            self.shard.pr_push(x, (not warm) and it == 0, y)
            self._reduce_scatter(yr[:chunk], y[:chunk * self.P])
            dang = y[self.V:self.V + 1].clone()
            self._all_reduce(dang, dist.ReduceOp.SUM)
            yr[hi - lo:hi - lo + 1].copy_(dang)
            e.zero_()
            self.shard.pr_update_rows_dev(x, yr, damping, e)          # the local error stays on the device
            self._all_reduce(e, dist.ReduceOp.SUM)
            y.zero_()
            it += 1
            if float(e.item()) < tol:                                 # the iteration's one host read
                break
        # replicate x: the owned slices, back to back (the last one padded to chunk)
        xs = self.shard.vertex_array(chunk * self.P, torch.float64)
        mine = self.shard.vertex_array(chunk, torch.float64)
        mine.zero_()
        mine[:hi - lo].copy_(x[lo:hi])
        self._all_gather(xs, mine)
        x.copy_(xs[:self.V])
        return x, it
