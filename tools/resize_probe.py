"""Kernel times of one root resize (tools only): configs[3]-shaped store (V = 2^24, uniform,
strict deletes), inserts of 2^20 until the capacity doubles; the library profiler records the
resizing batch."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from gpma_gen.streams import CONFIGS, edge_values, make_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402

dev = torch.device("cuda:0")
cfg = CONFIGS[3]
pool = make_stream("uniform", cfg.V, 1 << 27, cfg.seed, device=dev)
vals = edge_values(pool, cfg.seed)
s = torch.cuda.Stream(dev)
with torch.cuda.stream(s):
    live = 1 << 23
    g = Gpma.gpma_create(cfg.V, pool[:live].contiguous(), vals[:live].contiguous(), delete_mode=1, stream=s)
    cap = g.gpma_stats()["capacity"]
    for step in range(200):
        ik, iv = pool[live:live + (1 << 20)].contiguous(), vals[live:live + (1 << 20)].contiguous()
        g.gpma_debug_profile("*")
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(s)
        g.gpma_update_batch(ik, iv, 0, stream=s)
        e1.record(s)
        e1.synchronize()
        prof = g.gpma_debug_profile_read()
        live += 1 << 20
        st = g.gpma_stats()
        if st["capacity"] != cap:
            print(f"resize {cap} -> {st['capacity']} at step {step}: {e0.elapsed_time(e1):.2f} ms")
            for k, v in sorted(prof.items(), key=lambda kv: -kv[1][1])[:15]:
                print(f"  {k:24s} {v[0]:4d} {v[1]:.3f}")
            break
