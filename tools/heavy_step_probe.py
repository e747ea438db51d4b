"""Kernel table of one heavy configs[3] grow step (tools only): the resize stress schedule on a
fresh store (second pass, warm pool), the library profiler on the insert of the step whose
pending count after level 0 is largest below the first doubling; prints the insert's CUDA-event
time, the level trace summary and every kernel (launches, ms)."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from gpma_gen import CONFIGS  # noqa: E402
from gpma_gen.streams import edge_values, make_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402

dev = torch.device("cuda:0")
torch.cuda.set_device(dev)
cfg = CONFIGS[3]
pool = make_stream("uniform", cfg.V, cfg.E, cfg.seed, device=dev)
vals = edge_values(pool, cfg.seed)
N = pool.numel()


def seq(a, b):
    idx = torch.arange(a, b, device=dev) % N
    return pool[idx].contiguous(), vals[idx].contiguous()


s = torch.cuda.Stream(dev)
target = int(sys.argv[1]) if len(sys.argv) > 1 else 37
for rep in range(2):
    f, b = 0, 1 << 23
    with torch.cuda.stream(s):
        k0, v0 = seq(f, b)
        g = Gpma.gpma_create(cfg.V, k0, v0, delete_mode=1, stream=s)
        del k0, v0
        for step in range(target + 1):
            ni, nd = 1 << 20, 1 << 18
            ik, iv = seq(b, b + ni)
            dk, _ = seq(f, f + nd)
            prof = rep == 1 and step == target
            if prof:
                g.gpma_debug_profile("*")
            s.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            e0.record(s)
            g.gpma_update_batch(ik, iv, 0, stream=s)
            e1.record(s)
            e1.synchronize()
            if prof:
                st = g.gpma_stats_host()
                tab = g.gpma_debug_profile_read()
                ksum = sum(v[1] for v in tab.values())
                print(f"step {step}: insert {e0.elapsed_time(e1):.3f} ms, kernels {ksum:.3f} ms, pending level 1 "
                      f"{st['last_pending_level1']}, top level {st['last_top_level']}, launches "
                      f"{sum(v[0] for v in tab.values())}")
                for k, v in sorted(tab.items(), key=lambda kv: -kv[1][1]):
                    print(f"    {k:28s} {v[0]:4d} {v[1]:.3f}")
            g.gpma_update_batch(dk, None, 1, stream=s)
            b += ni
            f += nd
        del g
