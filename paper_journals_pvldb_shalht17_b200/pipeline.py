"""Transfer-hiding sliding-window driver (§3 Fig. 2).

"by repeating the aforementioned process, all data transfers are overlapped with concurrent
device computations".  Slide i's update + analytics run on the compute stream
through the C ABI (device buffers), while a copy stream moves slide i+1's batches host->device
and slide i-1's results device->host; events order the two streams.  Pure plumbing: every
step of the method still runs in libgpma's kernels.

When the copies run matters on B200: a PCIe-saturating D2H delays the GPU's own command fetch,
so every kernel launch and host read-back of the launch-dense phases (update, BFS, CC: dozens
of short kernels and one host round trip per level) slowed by ~0.1 ms while it ran
(tools/interference_probe.py).  The copies are therefore issued when the slide reaches its
long-kernel phases (CC + PageRank + export, ~6.5 ms of few, long launches; the ~5 ms D2H
fits inside): slide i-1's results D2H and slide i+1's batches H2D start there.
"""
from __future__ import annotations

import torch

from .fanout import AnalyticsFanout


class SlidingWindowPipeline:
    def __init__(self, g, V: int, max_batch: int, nnz_capacity: int, device, rows: int | None = None,
                 pr_tol: float = 1e-3, concurrent: bool = False, copy_csr: bool = True,
                 copy_results: bool = True):
        self.g, self.V, self.dev, self.pr_tol = g, V, torch.device(device), pr_tol
        self.copy_csr = copy_csr              # False: the exported CSR stays in HBM (device users)
        self.copy_results = copy_results      # False: no D2H at all (diagnostics)
        self.fan = AnalyticsFanout(self.dev, priorities=[0, -1, -2, 0]) if concurrent else None
        self.cs = torch.cuda.Stream(self.dev)      # compute
        self.xs = torch.cuda.Stream(self.dev)      # copies
        nr = V if rows is None else rows
        B = max_batch
        mk = lambda n, dt: torch.empty(n, dtype=dt, device=self.dev)
        self.d_in = [(mk(B, torch.int64), mk(B, torch.int64), mk(B, torch.int32)) for _ in range(2)]
        self.n_in = [(0, 0), (0, 0)]
        self.ev_in = [torch.cuda.Event() for _ in range(2)]
        self.pending_in = [None, None]                # staged batches whose H2D is not issued yet
        self.pending_out = [False, False]             # results whose D2H is not issued yet
        self.ev_long = torch.cuda.Event()
        # results of the previous slide are read from the second buffer while this one is written
        self.d_out = [(mk(V, torch.int32), mk(V, torch.int32), mk(nr + 1, torch.int64),
                       mk(nnz_capacity, torch.int32), mk(nnz_capacity, torch.int32)) for _ in range(2)]
        self.x = mk(V, torch.float64)
        self.d_x = [mk(V, torch.float64) for _ in range(2)]
        self.ev_done = [torch.cuda.Event() for _ in range(2)]
        self.ev_out = [torch.cuda.Event() for _ in range(2)]
        pin = lambda t: torch.empty(t.shape, dtype=t.dtype, pin_memory=True)
        self.h_out = [tuple(pin(t) for t in self.d_out[0]) + (pin(self.x),) for _ in range(2)]
        self.nnz = [0, 0]
        self.pr_iters = []
        self.i = 0
        with torch.cuda.stream(self.cs):
            g.gpma_pagerank(self.x, warm_start=False, tol_l1=pr_tol, stream=self.cs)

    def stage(self, slot: int, dk, ik, iv):
        """Queue one slide's batches (pinned host tensors) for its buffer; the H2D is issued on
        the copy stream at the next slide's long-kernel phase (or when the slide runs)."""
        self._flush_in(slot)
        self.pending_in[slot] = (dk, ik, iv)
        self.n_in[slot] = (dk.numel(), ik.numel())

    def _flush_in(self, slot: int):
        p = self.pending_in[slot]
        if p is None:
            return
        self.pending_in[slot] = None
        dk, ik, iv = p
        kd, ki, vi = self.d_in[slot]
        self.xs.wait_event(self.ev_done[slot])       # the buffer's previous slide is consumed
        with torch.cuda.stream(self.xs):
            kd[: dk.numel()].copy_(dk, non_blocking=True)
            ki[: ik.numel()].copy_(ik, non_blocking=True)
            vi[: iv.numel()].copy_(iv, non_blocking=True)
            self.ev_in[slot].record(self.xs)

    def _flush_out(self, slot: int):
        """Queue the D2H of the results of the slide that last ran in `slot`."""
        if not self.pending_out[slot]:
            return
        self.pending_out[slot] = False
        self.xs.wait_event(self.ev_done[slot])
        if not self.copy_results:
            self.ev_out[slot].record(self.xs)
            return
        lv, lab, rp, col, cv = self.d_out[slot]
        h = self.h_out[slot]
        n = self.nnz[slot]
        with torch.cuda.stream(self.xs):
            h[0].copy_(lv, non_blocking=True)
            h[1].copy_(lab, non_blocking=True)
            if self.copy_csr:
                h[2].copy_(rp, non_blocking=True)
                h[3][:n].copy_(col[:n], non_blocking=True)
                h[4][:n].copy_(cv[:n], non_blocking=True)
            h[5].copy_(self.d_x[slot], non_blocking=True)
            self.ev_out[slot].record(self.xs)

    def run(self, slot: int, root: int):
        """Slide on the compute stream; the previous slide's D2H and the next slide's H2D go
        on the copy stream once this slide reaches CC."""
        g, s = self.g, self.cs
        kd, ki, vi = self.d_in[slot]
        self._flush_in(slot)                         # normally already issued
        nd, ni = self.n_in[slot]
        lv, lab, rp, col, cv = self.d_out[slot]
        s.wait_event(self.ev_in[slot])
        other = slot ^ 1
        with torch.cuda.stream(s):
            g.gpma_update_batch(kd[:nd], None, 1, stream=s)
            g.gpma_update_batch(ki[:ni], vi[:ni], 0, stream=s)
            s.wait_event(self.ev_out[slot])          # host copy of this buffer's last results is done
            dx = self.d_x[slot]

            def pr(st):
                it = g.gpma_pagerank(self.x, warm_start=True, tol_l1=self.pr_tol, stream=st)
                # snapshot for the D2H by an SM copy (x * 1.0 is exact), not a D2D cudaMemcpy:
                # that would queue on a copy engine behind the previous slide's result D2H
                torch.mul(self.x, 1.0, out=dx)
                return it

            def copies_now(st, overlap=None):
                self.ev_long.record(st)
                if overlap is not None:    # enqueue the next (sync-free) kernels first: the copy
                    overlap(st)            # issuing below then runs on the host while they do
                self.xs.wait_event(self.ev_long)
                self._flush_out(other)
                self._flush_in(other)

            if self.fan is not None:          # the read-only analytics side by side (fanout.py)
                copies_now(s)
                r = self.fan.run(s, [pr, lambda st: g.gpma_cc(lab, stream=st),
                                     lambda st: g.gpma_bfs(root, lv, stream=st),
                                     lambda st: g.gpma_export_csr(rp, col, cv, stream=st)])
                it, n = r[0], r[3]
            else:
                g.gpma_bfs(root, lv, stream=s)
                copies_now(s, overlap=lambda st: g.gpma_cc(lab, stream=st))
                it = pr(s)
                n = g.gpma_export_csr(rp, col, cv, stream=s)
            self.pr_iters.append(it)
            self.nnz[slot] = n
            self.ev_done[slot].record(s)
        self.pending_out[slot] = True

    def results(self, slot: int):
        """Host results of the slide that last ran in `slot` (waits for their copies)."""
        self._flush_out(slot)
        self.ev_out[slot].synchronize()
        lv, lab, rp, col, cv, x = self.h_out[slot]
        n = self.nnz[slot]
        return lv, lab, rp, col[:n], cv[:n], x

    def flush(self):
        """Issue every deferred copy now (no wait): the last slide's results D2H."""
        for slot in range(2):
            self._flush_out(slot)
            self._flush_in(slot)

    def drain(self):
        self.flush()
        torch.cuda.synchronize(self.dev)

    def close(self):
        if self.fan is not None:
            self.fan.close()
