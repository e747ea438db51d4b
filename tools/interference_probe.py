#!/usr/bin/env python
"""Does a concurrent large D2H (copy engine) slow the device step?  (tools only)"""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from gpma_gen import config_stream, bfs_root, CONFIGS
from paper_journals_pvldb_shalht17_b200 import Gpma

dev = torch.device("cuda:0")
torch.cuda.set_device(dev)
cfg = CONFIGS[2]
sw = config_stream(2, device=dev)
V, B = cfg.V, sw.batch
s = torch.cuda.Stream(dev)
xs = torch.cuda.Stream(dev)
with torch.cuda.stream(s):
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.contiguous(), v0.contiguous(), stream=s)
nnz_cap = sw.window + B
levels = torch.empty(V, dtype=torch.int32, device=dev); labels = torch.empty(V, dtype=torch.int32, device=dev)
xx = torch.empty(V, dtype=torch.float64, device=dev)
rp = torch.empty(V + 1, dtype=torch.int64, device=dev); col = torch.empty(nnz_cap, dtype=torch.int32, device=dev)
cv = torch.empty(nnz_cap, dtype=torch.int32, device=dev)
big = torch.empty(256 << 20, dtype=torch.uint8, device=dev)
hbig = torch.empty(256 << 20, dtype=torch.uint8, pin_memory=True)
with torch.cuda.stream(s):
    g.gpma_pagerank(xx, warm_start=False, tol_l1=1e-3, stream=s)
torch.cuda.synchronize()
i = [0]


def steps(n, busy):
    slides = [sw.slide(i[0] + j) for j in range(n)]
    roots = [bfs_root(sw, cfg.seed, i[0] + j) for j in range(n)]   # host values before the copies start
    torch.cuda.synchronize()
    if busy:
        with torch.cuda.stream(xs):
            for _ in range(3 * n):
                hbig.copy_(big, non_blocking=True)
    ph = {"upd": 0.0, "bfs": 0.0, "cc": 0.0, "pr": 0.0, "exp": 0.0}
    for j in range(n):
        dk, ik, iv = slides[j]
        e = [torch.cuda.Event(enable_timing=True) for _ in range(6)]
        with torch.cuda.stream(s):
            e[0].record(s)
            g.gpma_update_batch(dk, None, 1, stream=s); g.gpma_update_batch(ik, iv, 0, stream=s)
            e[1].record(s)
            g.gpma_bfs(roots[j], levels, stream=s)
            e[2].record(s)
            g.gpma_cc(labels, stream=s)
            e[3].record(s)
            g.gpma_pagerank(xx, warm_start=True, tol_l1=1e-3, max_iter=3, stream=s)
            e[4].record(s)
            g.gpma_export_csr(rp, col, cv, stream=s)
            e[5].record(s)
        s.synchronize()
        for k, name in enumerate(ph):
            ph[name] += e[k].elapsed_time(e[k + 1]) / n
    i[0] += n
    torch.cuda.synchronize()
    return {k: round(v, 3) for k, v in ph.items()}


steps(2, False)
print("idle ", steps(4, False))
print("busy ", steps(4, True))
print("idle ", steps(4, False))

# which BFS kernels stretch under the concurrent D2H?
for busy in (False, True):
    dk, ik, iv = sw.slide(i[0]); i[0] += 1
    root = bfs_root(sw, cfg.seed, i[0])
    torch.cuda.synchronize()
    if busy:
        with torch.cuda.stream(xs):
            for _ in range(6):
                hbig.copy_(big, non_blocking=True)
    g.gpma_debug_profile("*")
    t0 = time.perf_counter()
    with torch.cuda.stream(s):
        g.gpma_bfs(root, levels, stream=s)
    s.synchronize()
    wall = (time.perf_counter() - t0) * 1e3
    prof = g.gpma_debug_profile_read()
    g.gpma_debug_profile(None)
    torch.cuda.synchronize()
    print("busy" if busy else "idle", "bfs wall ms", round(wall, 3),
          {k: (v[0], round(v[1], 3)) for k, v in sorted(prof.items(), key=lambda kv: -kv[1][1])})
