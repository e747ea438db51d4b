import os, sys
sys.path.insert(0, os.getcwd())
import numpy as np, torch
import oracle as O
from paper_journals_pvldb_shalht17_b200 import Gpma
from tests.gpu_helpers import keys_t, vals_t, gpu_dump
for knobs in ({}, {"GPMA_INS_LEAFSORT": "0"}, {"GPMA_LVL_COOP": "0"}):
    for k_, v_ in knobs.items(): os.environ[k_] = v_
    V = 64
    g = Gpma.gpma_create(V, None, None)
    o = O.Oracle(V, [], [])
    k = (5 << 32) | 7
    for n in (3000, 300, 257, 64):
        g2 = Gpma.gpma_create(V, None, None); o2 = O.Oracle(V, [], [])
        g2.insert(keys_t([k] * n), vals_t(list(range(n))))
        o2.insert([k] * n, list(range(n)))
        gk = gpu_dump(g2)[0]; ok_, ov = o2.dump()
        st = g2.gpma_stats()
        print(knobs, n, "equal" if np.array_equal(gk, ok_) else "DIFF", {x: st[x] for x in ("live_edges", "last_unique", "last_pending", "last_windows_rewritten", "last_top_level", "last_level0_windows")})
    for k_ in knobs: del os.environ[k_]
