"""Print the kernels of the last update slide in an ncu --csv launch list (tools only):
usage: python tools/launch_table.py <launches.csv> [first-kernel-prefix]"""
import collections
import csv
import sys

rows = list(csv.reader(open(sys.argv[1])))
first = sys.argv[2] if len(sys.argv) > 2 else "k_lazy"
hi = [i for i, r in enumerate(rows) if r and r[0] == "ID"][0]
h = rows[hi]
ki, mi, vi, ii = h.index("Kernel Name"), h.index("Metric Name"), h.index("Metric Value"), h.index("ID")
per = collections.defaultdict(dict)
for r in rows[hi + 1:]:
    per[int(r[ii])][r[mi]] = r[vi]
    per[int(r[ii])]["name"] = r[ki][5:] if r[ki].startswith("void ") else r[ki]
ids = sorted(per)
names = [per[i]["name"] for i in ids]
starts = [i for i, n in enumerate(names) if n.startswith(first)]
a = starts[-2] if len(starts) > 1 else starts[-1]
b = starts[-1] if len(starts) > 1 else len(ids)
tot = 0.0
for i in ids[a - 4:b - 4]:
    p = per[i]
    t = float(p.get("gpu__time_duration.sum", 0)) / 1e3
    tot += t
    print(f"{p['name'][:44]:44s} {t:8.2f} us  rd {float(p.get('dram__bytes_read.sum', 0)) / 1e6:8.2f} MB  "
          f"wr {float(p.get('dram__bytes_write.sum', 0)) / 1e6:8.2f} MB")
print(f"total {tot:.1f} us")
