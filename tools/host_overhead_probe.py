"""Host-side cost of one C-ABI update call (tools only): Python binding + ctypes for an empty
batch, the raw ctypes call, and B=100 lazy delete / insert calls with their device time."""
import os
import sys
import time

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from gpma_gen import config_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402
from paper_journals_pvldb_shalht17_b200.gpma import lib, _stream  # noqa: E402

dev = torch.device("cuda:0")
sw = config_stream(1, device=dev)
k0, v0 = sw.initial()
g = Gpma.gpma_create(1_600_000, k0.contiguous(), v0.contiguous())
empty_k = torch.empty(0, dtype=torch.int64, device=dev)
empty_v = torch.empty(0, dtype=torch.int32, device=dev)


def t_us(f, n=200):
    for _ in range(10):
        f()
    t0 = time.perf_counter()
    for _ in range(n):
        f()
    return (time.perf_counter() - t0) / n * 1e6


print("python binding, n=0 insert: %.2f us" % t_us(lambda: g.gpma_update_batch(empty_k, empty_v, 0)))
s = _stream(None)
print("raw ctypes, n=0 insert: %.2f us" % t_us(lambda: lib().gpma_update_batch(g._h, None, None, 0, 0, s)))
print("torch.cuda.synchronize: %.2f us" % t_us(torch.cuda.synchronize))
B = 100
pos = [0]


def slide_del():
    p = pos[0]
    g.gpma_update_batch(sw.keys[p:p + B], None, 1)


def slide_ins():
    p = pos[0]
    g.gpma_update_batch(sw.keys[sw.window + p: sw.window + p + B], sw.vals[sw.window + p: sw.window + p + B], 0)
    pos[0] += B


print("B=100 lazy delete call: %.2f us" % t_us(slide_del, 100))
print("B=100 insert call: %.2f us" % t_us(slide_ins, 100))
dk = sw.keys[0:B].clone()
print("raw ctypes B=100 delete (same keys): %.2f us" % t_us(lambda: lib().gpma_update_batch(g._h, dk.data_ptr(), None, B, 1, s)))
