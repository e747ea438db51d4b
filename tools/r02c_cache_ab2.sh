#!/bin/bash
# block-cache threshold A/B on one box: the library built twice (1 MiB / 64 MiB), alternating runs
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
cp paper_journals_pvldb_shalht17_b200/lib/libgpma.so /tmp/lib_1m.so
sed -i 's/constexpr size_t BIG_BLOCK = 1u << 20;/constexpr size_t BIG_BLOCK = 64u << 20;/' paper_journals_pvldb_shalht17_b200/csrc/primitives.cu
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
cp paper_journals_pvldb_shalht17_b200/lib/libgpma.so /tmp/lib_64m.so
for v in 1m 64m 1m 64m; do
  cp /tmp/lib_$v.so paper_journals_pvldb_shalht17_b200/lib/libgpma.so
  timeout 600 python bench.py --no-cpu-baseline --no-e2e --no-sweep > gpurun_out/cab_$v.json 2>/dev/null
  python - $v gpurun_out/cab_$v.json <<'PY'
import json, sys
d = json.loads(open(sys.argv[2]).read().strip().splitlines()[-1]); x = d["resize_stress"]
print(sys.argv[1], round(d["ms_per_step"], 3), {k: round(v, 4) for k, v in d["breakdown_ms"].items() if isinstance(v, float)},
      round(x["ms_per_step_mean"], 3), x["slowest_steps"][:2])
PY
done
