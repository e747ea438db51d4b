"""Brief per-kernel summary of an ncu --set full report (tools only):
python tools/ncu_brief.py <report.ncu-rep>  -> time, DRAM bytes, throughput %, occupancy, top stalls."""
import csv
import io
import subprocess
import sys

raw = subprocess.run(["ncu", "-i", sys.argv[1], "--page", "raw", "--csv"], capture_output=True, text=True).stdout
rows = list(csv.reader(io.StringIO(raw)))
h = rows[0]


def col(r, name):
    return r[h.index(name)] if name in h else ""


stall = [i for i, x in enumerate(h) if x.startswith("smsp__average_warps_issue_stalled_") and
         x.endswith("_per_issue_active.ratio")]
for r in rows[2:]:
    name = col(r, "Kernel Name")[:40]
    t = col(r, "gpu__time_duration.sum")
    rd = float(col(r, "dram__bytes_read.sum") or 0)
    wr = float(col(r, "dram__bytes_write.sum") or 0)
    print(f"{name:40s} t={t} us  dram rd={rd:.1f} wr={wr:.1f} MB  dram%={col(r, 'gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed')}"
          f"  sm%={col(r, 'sm__throughput.avg.pct_of_peak_sustained_elapsed')}  warps%={col(r, 'sm__warps_active.avg.pct_of_peak_sustained_active')}"
          f"  regs={col(r, 'launch__registers_per_thread')}  inst={col(r, 'smsp__inst_executed.sum')}  l2hit={col(r, 'lts__t_sector_hit_rate.pct')}")
    st = sorted(((float(r[i] or 0), h[i][len("smsp__average_warps_issue_stalled_"):-len("_per_issue_active.ratio")])
                 for i in stall), reverse=True)[:5]
    print("    stalls:", ", ".join(f"{n}={v:.2f}" for v, n in st))
