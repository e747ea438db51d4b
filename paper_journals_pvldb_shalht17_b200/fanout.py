"""Concurrent analytics after an update (include/gpma.h, "Concurrency").

BFS, CC, PageRank and export only read the store (§5 P:1090-1108 runs each of them on the
same GPMA+ snapshot) and each is bound by something different -- BFS and CC by dependent
loads and per-level host round trips, PageRank by random REDs, export by write bandwidth --
so the step runs them side by side: one stream and one host thread per analytic (ctypes
releases the GIL inside every C call), fenced by events after the update and before the
next one.  Plumbing only: every kernel is libgpma's.
"""
from __future__ import annotations

from concurrent.futures import ThreadPoolExecutor

import torch


class AnalyticsFanout:
    def __init__(self, device, n: int = 4, timing: bool = False, priorities=None):
        self.dev = torch.device(device)
        pr = list(priorities) if priorities is not None else [0] * n
        self.streams = [torch.cuda.Stream(self.dev, priority=pr[k]) for k in range(n)]
        self.pool = ThreadPoolExecutor(n, initializer=torch.cuda.set_device, initargs=(self.dev,))
        self.ev_fork = torch.cuda.Event()
        self.ev_join = [torch.cuda.Event() for _ in range(n)]
        self.timing = timing
        self.history = []           # per run: [(start, end) event per job] when timing

    def _one(self, k, fn, ev):
        st = self.streams[k]
        with torch.cuda.stream(st):
            if ev:
                ev[0].record(st)
            r = fn(st)
            if ev:
                ev[1].record(st)
            self.ev_join[k].record(st)
        return r

    def run(self, s, jobs):
        """Run jobs[k](stream_k) concurrently after the work queued on `s`; `s` then waits
        for all of them.  Returns the jobs' results in order."""
        assert len(jobs) <= len(self.streams)
        self.ev_fork.record(s)
        for st in self.streams[: len(jobs)]:
            st.wait_event(self.ev_fork)
        evs = [[torch.cuda.Event(enable_timing=True) for _ in range(2)] if self.timing else None
               for _ in jobs]
        if self.timing:
            self.history.append(evs)
        futs = [self.pool.submit(self._one, k, fn, evs[k]) for k, fn in enumerate(jobs)]
        res = [f.result() for f in futs]
        for k in range(len(jobs)):
            s.wait_event(self.ev_join[k])
        return res

    def history_ms(self):
        """Per-run, per-job device times (timing=True; call after synchronising)."""
        return [[a.elapsed_time(b) for a, b in run] for run in self.history]

    def close(self):
        self.pool.shutdown(wait=True)
