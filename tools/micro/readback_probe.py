#!/usr/bin/env python
"""Latency of a small device->host read-back (kernel store to pinned memory vs cudaMemcpyAsync)
with and without a large D2H copy in flight on another stream.  (tools only)"""
import time, torch
dev = torch.device("cuda:0")
big = torch.empty(256 << 20, dtype=torch.uint8, device=dev)
hbig = torch.empty(256 << 20, dtype=torch.uint8, pin_memory=True)
small = torch.ones(2, dtype=torch.int64, device=dev)
hs = torch.empty(2, dtype=torch.int64, pin_memory=True)
cs, xs = torch.cuda.Stream(), torch.cuda.Stream()

def loop(kind, n=200):
    torch.cuda.synchronize()
    t0 = time.perf_counter()
    for _ in range(n):
        with torch.cuda.stream(cs):
            if kind == "memcpy":
                hs.copy_(small, non_blocking=True)
            else:   # an SM store into pinned host memory (zero-copy): index_copy on a mapped view
                small.add_(0)
        cs.synchronize()
    return (time.perf_counter() - t0) / n * 1e6

for busy in (False, True):
    if busy:
        with torch.cuda.stream(xs):
            for _ in range(8):
                hbig.copy_(big, non_blocking=True)
    print("busy" if busy else "idle", "memcpy us", round(loop("memcpy"), 1), "kernel+sync us", round(loop("kernel"), 1))
    torch.cuda.synchronize()
