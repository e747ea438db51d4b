"""The device level loop under a dense store (tools only): configs[3]-shaped (V = 2^24, uniform
edges) at capacity 2^27 filled to just under the root bound, then one uniform 2^20-edge insert
batch -- ~0.6M updates climb past the leaves, the regime of the grow phase of the resize stress.
Prints the insert's CUDA-event time; GPMA_TRACE_LEVELS=1 adds the level trace."""
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import oracle as O  # noqa: E402
from gpma_gen import CONFIGS  # noqa: E402
from gpma_gen.streams import edge_values, make_stream  # noqa: E402
from paper_journals_pvldb_shalht17_b200 import Gpma  # noqa: E402

dev = torch.device("cuda:0")
torch.cuda.set_device(dev)
V, cap0 = 1 << 24, 1 << 27
mx = O.thresholds(16, 23)[1][23]
E0 = mx - V - (1 << 22)
reps = int(sys.argv[1]) if len(sys.argv) > 1 else 3
pool = make_stream("uniform", V, E0 + reps * (1 << 20), CONFIGS[3].seed + 5, device=dev)
vals = edge_values(pool, CONFIGS[3].seed + 5)
g = Gpma.gpma_create(V, pool[:E0].contiguous(), vals[:E0].contiguous(), delete_mode=1, initial_capacity=cap0)
for r in range(reps):
    a, b = E0 + r * (1 << 20), E0 + (r + 1) * (1 << 20)
    ik, iv = pool[a:b].contiguous(), vals[a:b].contiguous()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    e0.record()
    g.insert(ik, iv)
    e1.record()
    e1.synchronize()
    st = g.gpma_stats_host()
    print(f"insert {r}: {e0.elapsed_time(e1):.3f} ms, pending level 1 {st['last_pending_level1']}, "
          f"top level {st['last_top_level']}, capacity {st['capacity']}", flush=True)
