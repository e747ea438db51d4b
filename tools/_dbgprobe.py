import sys, os, ctypes, numpy as np, torch
sys.path.insert(0, os.getcwd())
from gpma_gen import config_stream
from paper_journals_pvldb_shalht17_b200 import Gpma
from paper_journals_pvldb_shalht17_b200.gpma import lib
dev = torch.device("cuda:0"); sw = config_stream(1, device=dev); k0, v0 = sw.initial()
g = Gpma.gpma_create(1_600_000, k0.contiguous(), v0.contiguous())
out = (ctypes.c_ulonglong * 64)()
for B in (100, 1000, 2000):
    pos = 0
    for it in range(8):
        dk = sw.keys[pos:pos + B]; ik = sw.keys[sw.window + pos: sw.window + pos + B]; iv = sw.vals[sw.window + pos: sw.window + pos + B]
        pos += B
        for i in range(64): out[i] = 0
        lib().gp_dbg_times(out)
        g.gpma_update_batch(dk, None, 1); g.gpma_update_batch(ik, iv, 0); torch.cuda.synchronize()
        lib().gp_dbg_times(out)
        t = np.array(out[:], dtype=np.int64)
        if it >= 5:
            base = t[0]
            print(B, {i: round((t[i] - base) / 1e3, 2) for i in range(23) if t[i] >= base and t[i] > 0})
