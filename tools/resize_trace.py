"""Where a resizing step of bench.py's configs[3] stress spends its time (tools only): the
same schedule (two passes on fresh stores), the library profiler on every step of the second
pass; for each resizing step print the CUDA-event time, host wall time, the sum of kernel times
and the top kernels (the remainder is allocation / host sync gaps)."""
import os
import sys
import time

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
for rep in range(int(sys.argv[1]) if len(sys.argv) > 1 else 3):  # noqa: C901
    f, b = 0, 1 << 23
    with torch.cuda.stream(s):
        k0, v0 = seq(f, b)
        g = Gpma.gpma_create(cfg.V, k0, v0, delete_mode=1, stream=s)
        del k0, v0
        res0 = g.gpma_stats()["resizes"]
        for step in range(490):
            ni, nd = (1 << 20, 1 << 18) if step < 242 else (1 << 18, 1 << 20)
            nd = min(nd, b + ni - f)
            ik, iv = seq(b, b + ni)
            dk, _ = seq(f, f + nd)
            if rep > 0:
                g.gpma_debug_profile("*")
            s.synchronize()
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            w0 = time.perf_counter()
            e0.record(s)
            nv = rep == 0 and str(step) in os.environ.get("RT_NVTX_STEPS", "").split(",")
            if nv:                                   # (ncu --nvtx --nvtx-include rzstep/)
                torch.cuda.nvtx.range_push("rzstep")
            g.gpma_update_batch(ik, iv, 0, stream=s)
            w1 = time.perf_counter()
            g.gpma_update_batch(dk, None, 1, stream=s)
            if nv:
                torch.cuda.nvtx.range_pop()
            e1.record(s)
            e1.synchronize()
            w2 = time.perf_counter()
            b += ni
            f += nd
            st = g.gpma_stats()
            prof = g.gpma_debug_profile_read() if rep > 0 else {}
            if st["resizes"] != res0:
                res0 = st["resizes"]
                ksum = sum(v[1] for v in prof.values())
                print(f"rep {rep} step {step} cap {st['capacity']}: events {e0.elapsed_time(e1):.2f} ms, "
                      f"wall insert {1e3 * (w1 - w0):.2f} delete {1e3 * (w2 - w1):.2f} ms, kernels {ksum:.2f} ms "
                      f"(levels skipped {st.get('last_levels_skipped', 0)} in the last call, top level "
                      f"{st['last_top_level']})", flush=True)
                for k, v in sorted(prof.items(), key=lambda kv: -kv[1][1])[:8]:
                    print(f"    {k:24s} {v[0]:4d} {v[1]:.3f}", flush=True)
        del g
