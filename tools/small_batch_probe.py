"""Small-batch slide anatomy (tools only): for B in (100, 1000) on configs[1], the per-slide
device time (CUDA events), host wall time of each C-ABI call, and the kernels one slide
launches with their device times (the library's event profiler)."""
import sys
import time

import numpy as np
import torch

sys.path.insert(0, __import__("os").path.dirname(__import__("os").path.dirname(__import__("os").path.abspath(__file__))))
from gpma_gen import config_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402

dev = torch.device("cuda:0")
sw = config_stream(1, device=dev)
k0, v0 = sw.initial()
s = torch.cuda.Stream(dev)
with torch.cuda.stream(s):
    for B in [int(b) for b in (sys.argv[1:] or ["100", "1000", "10000"])]:
        g = Gpma.gpma_create(1_600_000, k0.contiguous(), v0.contiguous(), stream=s)
        pos = 0
        ev, hd, hi = [], [], []
        for it in range(min(60, (sw.keys.numel() - sw.window) // B - 1)):
            dk = sw.keys[pos:pos + B]
            ik = sw.keys[sw.window + pos: sw.window + pos + B]
            iv = sw.vals[sw.window + pos: sw.window + pos + B]
            pos += B
            if it == min(50, (sw.keys.numel() - sw.window) // B - 3):
                g.gpma_debug_profile("*")
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(s)
            t0 = time.perf_counter()
            g.gpma_update_batch(dk, None, 1, stream=s)
            t1 = time.perf_counter()
            g.gpma_update_batch(ik, iv, 0, stream=s)
            t2 = time.perf_counter()
            e1.record(s)
            e1.synchronize()
            if it == min(50, (sw.keys.numel() - sw.window) // B - 3):
                prof = g.gpma_debug_profile_read()
                g.gpma_debug_profile(None)
            elif it >= 3:
                ev.append(e0.elapsed_time(e1))
                hd.append((t1 - t0) * 1e3)
                hi.append((t2 - t1) * 1e3)
        print(f"B={B}: levels climbed by the last insert {g.gpma_stats()['last_top_level']}; slide {np.mean(ev):.4f} ms (events), host delete call {np.mean(hd):.4f} ms, "
              f"host insert call {np.mean(hi):.4f} ms")
        tot = sum(v[1] for v in prof.values())
        n = sum(v[0] for v in prof.values())
        print(f"  profiled slide: {n} launches, {tot:.4f} ms of kernel time (event-bracketed)")
        for k, v in sorted(prof.items(), key=lambda kv: -kv[1][1]):
            print(f"    {k:24s} {v[0]:3d} {v[1]:.4f}")
        del g
