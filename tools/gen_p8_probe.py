"""Memory / time of generating the P = 8 weak-scaled stream (configs[4] size, 2^31 edges) on
one GPU (tools only): peak allocation per generator phase."""
import sys
import time

import torch

sys.path.insert(0, __import__("os").path.dirname(__import__("os").path.dirname(__import__("os").path.abspath(__file__))))
import gpma_gen.streams as S  # noqa: E402

marks = []
_unique = torch.unique


def unique_traced(x, *a, **k):
    r = _unique(x, *a, **k)
    marks.append(("unique n=%d" % x.numel(), torch.cuda.max_memory_allocated() / 1e9))
    torch.cuda.reset_peak_memory_stats()
    return r


torch.unique = unique_traced
t = time.time()
sw = S.config_stream(S.weak_scaled(2, 8), device="cuda:0")
torch.cuda.synchronize()
print("P=8 stream", sw.keys.numel(), "gen s", round(time.time() - t, 2), "peak GB after last unique",
      torch.cuda.max_memory_allocated() / 1e9, flush=True)
worst = sorted(marks, key=lambda m: -m[1])[:6]
for m in worst:
    print("  peak before", m[0], round(m[1], 1), "GB")
