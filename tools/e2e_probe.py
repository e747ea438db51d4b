#!/usr/bin/env python
"""Where does the e2e step lose time against the device step?  (tools only)
Times on configs[2]: (a) the pipelined e2e slide, (b) the same with the D2H copies skipped,
(c) the D2H of one slide's results alone, (d) the device step on resident buffers."""
import os, sys, time
sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))
import torch
from gpma_gen import config_stream, bfs_root, CONFIGS
from paper_journals_pvldb_shalht17_b200 import Gpma
from paper_journals_pvldb_shalht17_b200.pipeline import SlidingWindowPipeline

dev = torch.device("cuda:0")
torch.cuda.set_device(dev)
cfg = CONFIGS[2]
sw = config_stream(2, device=dev)
V, B = cfg.V, sw.batch
s = torch.cuda.Stream(dev)
with torch.cuda.stream(s):
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(V, k0.contiguous(), v0.contiguous(), stream=s)
torch.cuda.synchronize()
nnz_cap = sw.window + B
slide = [0]


def run_pipe(nsteps, skip_d2h):
    pipe = SlidingWindowPipeline(g, V, B, nnz_cap, dev, pr_tol=1e-3, copy_csr=False, copy_results=not skip_d2h)
    batches = []
    for j in range(nsteps + 1):
        dk, ik, iv = sw.slide(slide[0] + j)
        batches.append((dk.cpu().pin_memory(), ik.cpu().pin_memory(), iv.cpu().pin_memory()))
    roots = [bfs_root(sw, cfg.seed, slide[0] + j) for j in range(nsteps + 1)]
    slide[0] += nsteps + 1
    pipe.stage(0, *batches[0]); pipe.run(0, roots[0]); pipe.drain()
    t0 = time.perf_counter()
    pipe.stage(1, *batches[1])
    for j in range(1, nsteps + 1):
        if j + 1 <= nsteps:
            pipe.stage((j + 1) % 2, *batches[j + 1])
        pipe.run(j % 2, roots[j])
    pipe.drain()
    return (time.perf_counter() - t0) * 1e3 / nsteps


print("e2e pipelined  ms/step", run_pipe(5, False))
print("e2e pipelined, no D2H  ms/step", run_pipe(5, True))
# D2H alone
lv = torch.empty(V, dtype=torch.int32, device=dev); x = torch.empty(V, dtype=torch.float64, device=dev)
hl = torch.empty(V, dtype=torch.int32, pin_memory=True); hx = torch.empty(V, dtype=torch.float64, pin_memory=True)
torch.cuda.synchronize()
t0 = time.perf_counter()
for _ in range(5):
    hl.copy_(lv, non_blocking=True); hl.copy_(lv, non_blocking=True); hx.copy_(x, non_blocking=True)
torch.cuda.synchronize()
ms = (time.perf_counter() - t0) * 1e3 / 5
print("D2H of levels+labels+x alone ms", ms, "GB/s", 16 * V / ms / 1e6)
hb = torch.empty(B, dtype=torch.int64, pin_memory=True); db = torch.empty(B, dtype=torch.int64, device=dev)
torch.cuda.synchronize(); t0 = time.perf_counter()
for _ in range(5):
    db.copy_(hb, non_blocking=True)
torch.cuda.synchronize()
ms = (time.perf_counter() - t0) * 1e3 / 5
print("H2D 8MB ms", ms, "GB/s", 8 * B / ms / 1e6)
# device step on resident buffers
levels = torch.empty(V, dtype=torch.int32, device=dev); labels = torch.empty(V, dtype=torch.int32, device=dev)
xx = torch.empty(V, dtype=torch.float64, device=dev)
rp = torch.empty(V + 1, dtype=torch.int64, device=dev); col = torch.empty(nnz_cap, dtype=torch.int32, device=dev)
cv = torch.empty(nnz_cap, dtype=torch.int32, device=dev)
with torch.cuda.stream(s):
    g.gpma_pagerank(xx, warm_start=False, tol_l1=1e-3, stream=s)
torch.cuda.synchronize()
t0 = time.perf_counter()
for j in range(5):
    dk, ik, iv = sw.slide(slide[0] + j)
    with torch.cuda.stream(s):
        g.gpma_update_batch(dk, None, 1, stream=s); g.gpma_update_batch(ik, iv, 0, stream=s)
        g.gpma_bfs(bfs_root(sw, cfg.seed, slide[0] + j), levels, stream=s); g.gpma_cc(labels, stream=s)
        g.gpma_pagerank(xx, warm_start=True, tol_l1=1e-3, stream=s); g.gpma_export_csr(rp, col, cv, stream=s)
torch.cuda.synchronize()
print("device step (wall, incl. slide generation) ms", (time.perf_counter() - t0) * 1e3 / 5)

# ---- timeline of the pipelined slides: compute (cs) and copy (xs) intervals
pipe = SlidingWindowPipeline(g, V, B, nnz_cap, dev, pr_tol=1e-3, copy_csr=False)
nst = 4
batches, roots = [], []
for j in range(nst + 1):
    dk, ik, iv = sw.slide(slide[0] + j)
    batches.append((dk.cpu().pin_memory(), ik.cpu().pin_memory(), iv.cpu().pin_memory()))
    roots.append(bfs_root(sw, cfg.seed, slide[0] + j))
ev = []
orig_run = pipe.run


def timed_run(slot, root):
    a = torch.cuda.Event(enable_timing=True); a.record(pipe.cs)
    orig_run(slot, root)
    b = torch.cuda.Event(enable_timing=True); b.record(pipe.cs)
    c = torch.cuda.Event(enable_timing=True); c.record(pipe.xs)
    ev.append((a, b, c, time.perf_counter()))


pipe.run = timed_run
t00 = torch.cuda.Event(enable_timing=True)
t00.record(pipe.cs)
pipe.stage(0, *batches[0]); pipe.run(0, roots[0])
pipe.stage(1, *batches[1])
for j in range(1, nst + 1):
    if j + 1 <= nst:
        pipe.stage((j + 1) % 2, *batches[j + 1])
    pipe.run(j % 2, roots[j])
pipe.drain()
for j, (a, b, c, th) in enumerate(ev):
    print(f"slide {j}: compute {t00.elapsed_time(a):8.2f} -> {t00.elapsed_time(b):8.2f} ms, copies done {t00.elapsed_time(c):8.2f} ms")
