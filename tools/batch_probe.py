"""Update anatomy at one configs[1] batch size (tools only): CUDA-event times of the last slides and the library profiler table of the last one.  usage: python tools/batch_probe.py <batch>"""
import os, sys, torch
sys.path.insert(0, os.getcwd())
from gpma_gen import CONFIGS, config_stream
from paper_journals_pvldb_shalht17_b200 import Gpma
dev = torch.device("cuda:0"); torch.cuda.set_device(dev)
sw = config_stream(1, device=dev); sw.batch = int(sys.argv[1])
s = torch.cuda.Stream(dev)
with torch.cuda.stream(s):
    k0, v0 = sw.initial()
    g = Gpma.gpma_create(CONFIGS[1].V, k0.contiguous(), v0.contiguous(), stream=s)
    for i in range(12):
        dk, ik, iv = [t.contiguous() for t in sw.slide(i)]
        prof = i == 11
        if prof: g.gpma_debug_profile("*")
        s.synchronize()
        e = [torch.cuda.Event(enable_timing=True) for _ in range(3)]
        e[0].record(s); g.gpma_update_batch(dk, None, 1, stream=s); e[1].record(s); g.gpma_update_batch(ik, iv, 0, stream=s); e[2].record(s)
        e[2].synchronize()
        if i >= 9: print(i, "delete %.3f insert %.3f ms" % (e[0].elapsed_time(e[1]), e[1].elapsed_time(e[2])), g.gpma_stats_host()["last_pending_level1"])
        if prof:
            t = g.gpma_debug_profile_read()
            print(sum(v[1] for v in t.values()), sum(v[0] for v in t.values()))
            for k, v in sorted(t.items(), key=lambda kv: -kv[1][1])[:14]: print("   ", k, v)
