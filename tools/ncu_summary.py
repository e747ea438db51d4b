#!/usr/bin/env python
"""Summarise ncu outputs into profiles/ (run here, on the CPU box, after tools/profile_r*.sh).

usage: python tools/ncu_summary.py <round-tag> <launches.csv> <full.ncu-rep>
writes profiles/<tag>_launches_summary.json, profiles/<tag>_ncu_full.json,
profiles/<tag>_ncu_summary.md and profiles/ncu_traffic.json (dram bytes per launch of each
fully-profiled kernel, read by bench.py for roofline.traffic).
"""
import collections
import csv
import io
import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _num(x):
    try:
        return float(x.replace(",", ""))
    except Exception:
        return None


def launches(path):
    rows = list(csv.reader(open(path)))
    # skip ncu banner lines until the header
    start = next(i for i, r in enumerate(rows) if r and r[0] == "ID")
    hdr = rows[start]
    ki, mi, vi, ui = hdr.index("Kernel Name"), hdr.index("Metric Name"), hdr.index("Metric Value"), hdr.index("Metric Unit")
    per = collections.defaultdict(lambda: {"launches": 0, "ms": 0.0, "dram_bytes": 0.0})
    seen = set()
    # keep the sliding-window steps only: launches from the 2nd k_validate on (the 1st
    # belongs to gpma_create, whose bulk sort/layout is setup, not the hot path)
    ids = []
    for r in rows[start + 1:]:
        if len(r) > ki and r[ki].startswith("k_validate") and r[0] not in ids:
            ids.append(r[0])
    first_step = int(ids[1]) if len(ids) > 1 else 0
    scale = {"nsecond": 1e-6, "ns": 1e-6, "usecond": 1e-3, "us": 1e-3, "msecond": 1.0, "ms": 1.0, "second": 1e3,
             "byte": 1.0, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}
    for r in rows[start + 1:]:
        if len(r) <= vi:
            continue
        if not r[0].isdigit() or int(r[0]) < first_step:
            continue
        name = r[ki].split("(")[0].split("<")[0].replace("void ", "").replace("gp::", "")
        v = _num(r[vi])
        if v is None:
            continue
        v *= scale.get(r[ui], 1.0)
        key = (r[0], name)
        if r[mi] == "gpu__time_duration.sum":
            per[name]["ms"] += v
            if key not in seen:
                per[name]["launches"] += 1
                seen.add(key)
        elif r[mi].startswith("dram__bytes"):
            per[name]["dram_bytes"] += v
    tot = sum(p["ms"] for p in per.values())
    out = {k: {**v, "share": v["ms"] / tot if tot else 0.0} for k, v in
           sorted(per.items(), key=lambda kv: -kv[1]["ms"])}
    return out, tot


WANT = {
    "gpu__time_duration.sum": "duration",
    "dram__bytes_read.sum": "dram_read",
    "dram__bytes_write.sum": "dram_write",
    "gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed": "dram_pct_peak",
    "lts__t_sector_hit_rate.pct": "l2_hit_pct",
    "sm__throughput.avg.pct_of_peak_sustained_elapsed": "sm_pct_peak",
    "sm__warps_active.avg.pct_of_peak_sustained_active": "warps_active_pct",
    "launch__registers_per_thread": "regs",
    "smsp__average_warps_issue_stalled_long_scoreboard_per_issue_active.ratio": "stall_long_scoreboard",
    "smsp__average_warps_issue_stalled_lg_throttle_per_issue_active.ratio": "stall_lg_throttle",
    "lts__t_sectors_srcunit_tex_op_red_lookup_miss.sum": "l2_red_sector_miss",
}


def full(path):
    raw = subprocess.check_output(["ncu", "-i", path, "--page", "raw", "--csv"], stderr=subprocess.DEVNULL)
    rows = list(csv.reader(io.StringIO(raw.decode())))
    hdr, units = rows[0], rows[1]
    idx = {k: hdr.index(k) for k in WANT if k in hdr}
    res = []
    for r in rows[2:]:
        d = {"kernel": r[hdr.index("Kernel Name")].split("(")[0].split("<")[0].replace("void ", "").replace("gp::", "")}
        for k, i in idx.items():
            v = _num(r[i])
            u = units[i]
            if v is not None and k.startswith("dram__bytes"):
                v *= {"byte": 1, "Kbyte": 1e3, "Mbyte": 1e6, "Gbyte": 1e9}.get(u, 1)
            if v is not None and k == "gpu__time_duration.sum":
                v *= {"nsecond": 1e-6, "usecond": 1e-3, "msecond": 1.0}.get(u, 1)
            d[WANT[k]] = v
        res.append(d)
    return res


def main():
    tag, lpath, fpath = sys.argv[1:4]
    prof = os.path.join(ROOT, "profiles")
    os.makedirs(prof, exist_ok=True)
    per, tot = launches(lpath)
    json.dump({"source": os.path.basename(lpath), "total_ms": tot, "kernels": per},
              open(os.path.join(prof, f"{tag}_launches_summary.json"), "w"), indent=1)
    fr = full(fpath)
    json.dump(fr, open(os.path.join(prof, f"{tag}_ncu_full.json"), "w"), indent=1)
    traffic = {}
    for d in fr:
        if d.get("dram_read") is not None:
            traffic.setdefault(d["kernel"], []).append(d["dram_read"] + d.get("dram_write", 0))
    traffic = {k: sum(v) / len(v) for k, v in traffic.items()}
    json.dump({"tag": tag, "dram_bytes_per_launch": traffic},
              open(os.path.join(prof, "ncu_traffic.json"), "w"), indent=1)
    with open(os.path.join(prof, f"{tag}_ncu_summary.md"), "w") as f:
        f.write(f"# {tag}: ncu summary\n\n## Launch list of the sliding-window steps (cold-cache, serialised; compare shares)\n\n")
        f.write(f"Total over the listed launches: {tot:.3f} ms (all steps of the profiled command).\n\n")
        f.write("| kernel | launches | total ms | share | DRAM GB |\n|---|---|---|---|---|\n")
        for k, v in list(per.items())[:25]:
            f.write(f"| {k} | {v['launches']} | {v['ms']:.3f} | {100 * v['share']:.1f}% | {v['dram_bytes'] / 1e9:.3f} |\n")
        f.write("\n## Full-set captures\n\n| kernel | ms | DRAM rd GB | DRAM wr GB | DRAM % peak | L2 hit % | SM % | warps % | regs | stall long-sb | RED L2 miss sectors |\n|---|---|---|---|---|---|---|---|---|---|---|\n")
        for d in fr:
            g = lambda k, s=1.0, fmt="{:.3f}": (fmt.format(d[k] / s) if d.get(k) is not None else "-")
            f.write(f"| {d['kernel']} | {g('duration')} | {g('dram_read', 1e9)} | {g('dram_write', 1e9)} | "
                    f"{g('dram_pct_peak', 1, '{:.1f}')} | {g('l2_hit_pct', 1, '{:.1f}')} | {g('sm_pct_peak', 1, '{:.1f}')} | "
                    f"{g('warps_active_pct', 1, '{:.1f}')} | {g('regs', 1, '{:.0f}')} | {g('stall_long_scoreboard', 1, '{:.1f}')} | "
                    f"{g('l2_red_sector_miss', 1, '{:.0f}')} |\n")
    print(open(os.path.join(prof, f"{tag}_ncu_summary.md")).read())


if __name__ == "__main__":
    main()
