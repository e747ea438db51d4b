"""Update-path probe (tools only): configs[2] store, `--slides` sliding-window slides (DELETE
2^20 + INSERT 2^20) with no analytics -- short enough to run under ncu.  Prints the CUDA-event
time of delete / insert per slide and the mean over the last half.  Env knobs of the library
(GPMA_DEL_SORT, GPMA_INS_FUSED, ...) apply."""
import argparse
import json
import os
import sys

import numpy as np
import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
from gpma_gen import config_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--slides", type=int, default=8)
ap.add_argument("--config", type=int, default=2)
ap.add_argument("--batch", type=int, default=0)
a = ap.parse_args()
dev = torch.device("cuda:0")
sw = config_stream(a.config, device=dev)
if a.batch:
    sw.batch = a.batch
s = torch.cuda.Stream(dev)
out = []
with torch.cuda.stream(s):
    k0, v0 = sw.initial()
    from gpma_gen import CONFIGS
    V = CONFIGS[a.config].V
    g = Gpma.gpma_create(V, k0.contiguous(), v0.contiguous(), stream=s)
    for i in range(a.slides):
        dk, ik, iv = sw.slide(i)
        e = [torch.cuda.Event(enable_timing=True) for _ in range(3)]
        e[0].record(s)
        g.gpma_update_batch(dk, None, 1, stream=s)
        e[1].record(s)
        g.gpma_update_batch(ik, iv, 0, stream=s)
        e[2].record(s)
        e[2].synchronize()
        out.append((e[0].elapsed_time(e[1]), e[1].elapsed_time(e[2])))
h = np.array(out[len(out) // 2:])
print(json.dumps({"batch": sw.batch, "delete_ms": float(h[:, 0].mean()), "insert_ms": float(h[:, 1].mean()),
                  "per_slide": [[round(x, 4) for x in r] for r in out]}))
