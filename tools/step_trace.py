"""Per-step times of the configs[3] resize stress (tools only), second pass: prints a marker on
stderr before every step (so GPMA_TRACE_LEVELS / GPMA_TRACE_ALLOC output can be attributed) and
the insert / delete CUDA-event times of the steps in [lo, hi] (argv)."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from gpma_gen import CONFIGS  # noqa: E402
from gpma_gen.streams import edge_values, make_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402

lo, hi = int(sys.argv[1]), int(sys.argv[2])
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
for rep in range(2):
    f, b = 0, 1 << 23
    with torch.cuda.stream(s):
        k0, v0 = seq(f, b)
        g = Gpma.gpma_create(cfg.V, k0, v0, delete_mode=1, stream=s)
        del k0, v0
        for step in range(490):
            ni, nd = (1 << 20, 1 << 18) if step < 242 else (1 << 18, 1 << 20)
            nd = min(nd, b + ni - f)
            ik, iv = seq(b, b + ni)
            dk, _ = seq(f, f + nd)
            show = rep == 1 and lo <= step <= hi
            if show:
                print(f"=== step {step}", file=sys.stderr, flush=True)
            s.synchronize()
            e = [torch.cuda.Event(enable_timing=True) for _ in range(3)]
            e[0].record(s)
            g.gpma_update_batch(ik, iv, 0, stream=s)
            if show:
                print("=== delete", file=sys.stderr, flush=True)
            e[1].record(s)
            g.gpma_update_batch(dk, None, 1, stream=s)
            e[2].record(s)
            e[2].synchronize()
            b += ni
            f += nd
            if show:
                st = g.gpma_stats_host()
                print(f"step {step}: insert {e[0].elapsed_time(e[1]):.3f} ms, delete {e[1].elapsed_time(e[2]):.3f} ms, "
                      f"cap {st['capacity']}, top level {st['last_top_level']}, skipped {st['last_levels_skipped']}",
                      flush=True)
        del g
