"""Run bench.py's configs[3] resize stress several times in one process (tools only) and print
each run's per-resizing-step times, to separate run-to-run variance from a regression."""
import json
import os
import sys

import torch

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import bench  # noqa: E402

dev = torch.device("cuda:0")
torch.cuda.set_device(dev)
for r in range(int(sys.argv[1]) if len(sys.argv) > 1 else 3):
    out = bench.resize_stress(dev)
    print(json.dumps({k: out[k] for k in ("updates_per_s", "ms_other_step_mean", "ms_resize_steps")}),
          flush=True)
