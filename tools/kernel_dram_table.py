"""Per-kernel DRAM throughput of one bench step from an ncu --csv launch list (tools only):
python tools/kernel_dram_table.py <launches.csv> [peak_GBs] [random_ceiling_GBs]
Takes the launches of the last full step (from the last-but-one lazy delete to the last one),
aggregates them by kernel and prints time, DRAM bytes, achieved DRAM GB/s and its fraction of the
measured copy peak (MEASURED_PEAKS.json) and of the random-access ceiling
(profiles/random_access: ~40 G random 128-B line fetches/s = 5.1 TB/s of DRAM traffic)."""
import collections
import csv
import json
import os
import sys

rows = list(csv.reader(open(sys.argv[1])))
root = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
peak = float(sys.argv[2]) if len(sys.argv) > 2 else json.load(open(os.path.join(root, "MEASURED_PEAKS.json")))["hbm_gbs"]
rnd = float(sys.argv[3]) if len(sys.argv) > 3 else 5100.0
hi = [i for i, r in enumerate(rows) if r and r[0] == "ID"][0]
h = rows[hi]
ki, mi, vi, ii = h.index("Kernel Name"), h.index("Metric Name"), h.index("Metric Value"), h.index("ID")
per = collections.defaultdict(dict)
for r in rows[hi + 1:]:
    per[int(r[ii])][r[mi]] = float(r[vi].replace(",", "")) if r[vi] else 0.0
    nm = r[ki][5:] if r[ki].startswith("void ") else r[ki]
    per[int(r[ii])]["name"] = nm.split("(")[0].split("<")[0]
ids = sorted(per)
starts = [i for i in ids if per[i]["name"].startswith("k_lazy_delete")]
a, b = (starts[-2], starts[-1]) if len(starts) > 1 else (starts[-1], ids[-1] + 1)
agg = collections.defaultdict(lambda: [0, 0.0, 0.0])
for i in ids:
    if a <= i < b:
        p = per[i]
        e = agg[p["name"]]
        e[0] += 1
        e[1] += p.get("gpu__time_duration.sum", 0) / 1e3
        e[2] += p.get("dram__bytes_read.sum", 0) + p.get("dram__bytes_write.sum", 0)
tot = sum(e[1] for e in agg.values())
print(f"# one step = launches {a}..{b - 1} of {sys.argv[1]}: {tot:.1f} us of kernels (serialised, ncu)")
print(f"# peak (copy) {peak:.0f} GB/s; random-access ceiling {rnd:.0f} GB/s of DRAM traffic")
print(f"{'kernel':28s} {'launches':>8s} {'us':>9s} {'share':>6s} {'DRAM MB':>9s} {'GB/s':>7s} {'/peak':>6s} {'/rand':>6s}")
for k, (n, us, by) in sorted(agg.items(), key=lambda kv: -kv[1][1]):
    gbs = by / (us * 1e3) if us else 0.0
    print(f"{k:28s} {n:8d} {us:9.1f} {us / tot:6.1%} {by / 1e6:9.1f} {gbs:7.0f} {gbs / peak:6.2f} {gbs / rnd:6.2f}")
