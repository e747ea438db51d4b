"""configs[3] ordinary steps A/B (tools only): the first `--grow` grow steps (INSERT 2^20, strict
DELETE 2^18) and `--shrink` steps of the shrink phase started from a grown store, insert and
delete CUDA-event times separately; the library knobs in the environment apply."""
import argparse
import json
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from gpma_gen import CONFIGS  # noqa: E402
from gpma_gen.streams import edge_values, make_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--grow", type=int, default=40)
ap.add_argument("--shrink", type=int, default=30)
a = ap.parse_args()
dev = torch.device("cuda:0")
cfg = CONFIGS[3]
pool = make_stream("uniform", cfg.V, 1 << 26, cfg.seed, device=dev)
vals = edge_values(pool, cfg.seed)
s = torch.cuda.Stream(dev)
ins, dels, resz = [], [], 0
with torch.cuda.stream(s):
    f, b = 0, 1 << 23
    g = Gpma.gpma_create(cfg.V, pool[f:b].contiguous(), vals[f:b].contiguous(), delete_mode=1, stream=s)
    r0 = g.gpma_stats()["resizes"]
    for step in range(a.grow):
        ik, iv = pool[b:b + (1 << 20)].contiguous(), vals[b:b + (1 << 20)].contiguous()
        dk = pool[f:f + (1 << 18)].contiguous()
        e = [torch.cuda.Event(enable_timing=True) for _ in range(3)]
        e[0].record(s)
        g.gpma_update_batch(ik, iv, 0, stream=s)
        e[1].record(s)
        g.gpma_update_batch(dk, None, 1, stream=s)
        e[2].record(s)
        e[2].synchronize()
        b += 1 << 20
        f += 1 << 18
        r = g.gpma_stats()["resizes"]
        if r != r0:
            r0 = r
            resz += 1
            continue
        ins.append(e[0].elapsed_time(e[1]))
        dels.append(e[1].elapsed_time(e[2]))
    sins, sdel = [], []
    for step in range(a.shrink):
        ik, iv = pool[b:b + (1 << 18)].contiguous(), vals[b:b + (1 << 18)].contiguous()
        dk = pool[f:f + (1 << 20)].contiguous()
        e = [torch.cuda.Event(enable_timing=True) for _ in range(3)]
        e[0].record(s)
        g.gpma_update_batch(ik, iv, 0, stream=s)
        e[1].record(s)
        g.gpma_update_batch(dk, None, 1, stream=s)
        e[2].record(s)
        e[2].synchronize()
        b += 1 << 18
        f += 1 << 20
        r = g.gpma_stats()["resizes"]
        if r != r0:
            r0 = r
            resz += 1
            continue
        sins.append(e[0].elapsed_time(e[1]))
        sdel.append(e[1].elapsed_time(e[2]))
h = len(ins) // 4
print(json.dumps({"knobs": {k: v for k, v in os.environ.items() if k.startswith("GPMA_")},
                  "grow_insert_ms": float(np.mean(ins[h:])), "grow_delete_ms": float(np.mean(dels[h:])),
                  "shrink_insert_ms": float(np.mean(sins)) if sins else None,
                  "shrink_delete_ms": float(np.mean(sdel)) if sdel else None,
                  "steps": len(ins) + len(sins), "resizing_steps": resz}))
