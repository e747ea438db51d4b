#!/usr/bin/env python
"""Top SASS lines by warp-stall samples from an ncu report: python tools/ncu_hot.py rep [n]"""
import csv, io, subprocess, sys
rep = sys.argv[1]; n = int(sys.argv[2]) if len(sys.argv) > 2 else 20
raw = subprocess.check_output(["ncu", "-i", rep, "--page", "source", "--csv", "--print-source=sass"],
                              stderr=subprocess.DEVNULL).decode()
rows = list(csv.reader(io.StringIO(raw)))
hdr = rows[1]; ci = {h: i for i, h in enumerate(hdr)}
s = ci["Warp Stall Sampling (All Samples)"]
data = [(float(r[s] or 0), r[ci["Address"]], r[ci["Source"]]) for r in rows[2:] if len(r) > s]
tot = sum(d[0] for d in data) or 1
for v, a, src in sorted(data, reverse=True)[:n]:
    print(f"{100 * v / tot:5.1f}%  {a}  {src[:100]}")
