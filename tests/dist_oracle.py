"""CPU emulation of one rank's compute for the sharded store (test infrastructure).

It implements the per-rank steps that `paper_journals_pvldb_shalht17_b200.dist.CudaShard`
runs in libgpma kernels, plainly, on top of an oracle shard (`Oracle(..., rows=(lo, hi))`), so
that the orchestration and collectives of `DistGpma` can be exercised by world_size-2 gloo
tests without a GPU.
"""
from __future__ import annotations

import numpy as np
import torch

import oracle as O

SCALE = float(2 ** 62)


class OracleShard:
    def __init__(self, V, rows, delete_mode=O.LAZY):
        self.V, self.rows, self.mode = V, rows, delete_mode
        self.o = None
        self.device = torch.device("cpu")

    def create(self, keys, vals):
        self.o = O.Oracle(self.V, keys.numpy(), vals.numpy(), rows=self.rows, delete_mode=self.mode)

    def route(self, keys, vals, P):
        k = keys.numpy().view(np.uint64)
        v = np.zeros(k.size, np.int32) if vals is None else vals.numpy()
        chunk = (self.V + P - 1) // P
        owner = (k >> np.uint64(32)) // np.uint64(chunk)
        order = np.argsort(owner, kind="stable")
        counts = [int((owner == r).sum()) for r in range(P)]
        return (torch.from_numpy(k[order].view(np.int64).copy()), torch.from_numpy(v[order].copy()), counts)

    def validate(self, keys, vals, op) -> int:
        """gpma_validate_batch: RESERVED (3) beats RANGE (2); global vertex range."""
        k = keys.numpy().view(np.uint64)
        src, dst = k >> np.uint64(32), k & np.uint64(0xFFFFFFFF)
        if (dst == np.uint64(0xFFFFFFFF)).any():
            return 3
        if op == 0 and vals is not None and (vals.numpy().view(np.uint32) == np.uint32(0xFFFFFFFF)).any():
            return 3
        return 2 if ((src >= np.uint64(self.V)) | (dst >= np.uint64(self.V))).any() else 0

    def update(self, keys, vals, op):
        if op == 0:
            self.o.insert(keys.numpy(), vals.numpy())
        else:
            self.o.delete(keys.numpy())

    def vertex_array(self, n, dtype):
        return torch.empty(n, dtype=dtype)

    def sync(self):
        pass

    def _csr(self):
        rp, col, _ = self.o.export_csr()
        return rp.astype(np.int64), col.astype(np.int64)

    def bfs_init(self, root, levels):
        levels.fill_(-1)
        levels[root] = 0

    def bfs_level(self, levels, depth):
        lv = levels.numpy()
        front = np.nonzero(lv == depth - 1)[0]
        rp, col = self._csr()
        lo, hi = self.rows
        for u in front:
            if lo <= u < hi:
                for v in col[rp[u - lo]:rp[u - lo + 1]]:
                    if lv[v] == -1:
                        lv[v] = depth
        return int(front.size)

    def cc_round(self, labels, init):
        p = labels.numpy().view(np.uint32)
        if init:
            p[:] = np.arange(self.V, dtype=np.uint32)
        prev = p.copy()

        def find(x):
            while p[x] != x:
                x = p[x]
            return x

        rp, col = self._csr()
        lo, _ = self.rows
        for i in range(rp.size - 1):
            for v in col[rp[i]:rp[i + 1]]:
                a, b = find(lo + i), find(int(v))
                if a < b:
                    p[b] = a
                elif b < a:
                    p[a] = b
        for x in range(self.V):
            p[x] = find(x)
        return int((p != prev).sum())

    def pr_push(self, x, init, y):
        xv = x.numpy()
        if init:
            xv[:] = 1.0 / self.V
        yy = y.numpy().view(np.uint64)
        rp, col = self._csr()
        lo, _ = self.rows
        for i in range(rp.size - 1):
            deg = rp[i + 1] - rp[i]
            if deg == 0:
                yy[self.V] += np.uint64(round(xv[lo + i] * SCALE))
                continue
            c = np.uint64(round(xv[lo + i] / deg * SCALE))
            for v in col[rp[i]:rp[i + 1]]:
                yy[v] += c

    def pr_update(self, x, y, damping):
        xv = x.numpy()
        yy = y.numpy().view(np.uint64)
        D = float(yy[self.V]) / SCALE
        nx = (1 - damping) / self.V + damping * (yy[: self.V].astype(np.float64) / SCALE + D / self.V)
        err = float(np.abs(nx - xv).sum())
        xv[:] = nx
        yy[:] = 0
        return err

    def pr_update_rows(self, x, y_rows, damping):
        """gpma_pr_update_rows: the owned rows from their reduced sums (+ y_rows[nr] = dangling)."""
        xv = x.numpy()
        yr = y_rows.numpy().view(np.uint64)
        lo, hi = self.rows
        nr = hi - lo
        D = float(yr[nr]) / SCALE
        nx = (1 - damping) / self.V + damping * (yr[:nr].astype(np.float64) / SCALE + D / self.V)
        err = float(np.abs(nx - xv[lo:hi]).sum())
        xv[lo:hi] = nx
        return err

    def pr_update_rows_dev(self, x, y_rows, damping, err_dev):
        err_dev += self.pr_update_rows(x, y_rows, damping)

    def bfs_bits(self, levels, depth, bitmap):
        """gpma_bfs_bits: bit v of bitmap = (levels[v] == depth)."""
        lv = levels.numpy()
        bits = np.zeros(bitmap.numel() * 32, dtype=np.uint8)
        bits[: self.V] = lv == depth
        bitmap.numpy().view(np.uint32)[:] = np.packbits(bits, bitorder="little").view(np.uint32)

    def bfs_merge(self, levels, bitmaps, n, depth):
        """gpma_bfs_merge: levels[v] := depth where unreached and set in any bitmap."""
        lv = levels.numpy()
        words = (self.V + 31) // 32
        b = bitmaps.numpy().view(np.uint32).reshape(n, words)
        anyb = np.bitwise_or.reduce(b, axis=0)
        bits = np.unpackbits(anyb.view(np.uint8), bitorder="little")[: self.V].astype(bool)
        lv[bits & (lv == -1)] = depth
