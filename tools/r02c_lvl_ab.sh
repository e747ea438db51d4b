#!/bin/bash
# configs[3] resize stress, repeated (per-step p50 / p99 / max of the ordinary steps), with the
# environment settings given as arguments ("-" = defaults)
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
i=0
for kv in "$@"; do
  i=$((i+1))
  if [ "$kv" = "-" ]; then e=""; else e="$kv"; fi
  env $e timeout 900 python bench.py --steps 5 --warmup 3 --no-sweep --no-cpu-baseline --no-e2e > gpurun_out/lv_$i.json 2>/dev/null
  python - "$kv" gpurun_out/lv_$i.json <<'PY'
import json, sys
d = json.loads(open(sys.argv[2]).read().strip().splitlines()[-1])
r = d["resize_stress"]
print(sys.argv[1], "mean %.3f" % r["ms_per_step_mean"], "slowest", r["slowest_steps"], "other p50/p99/max",
      [round(x, 3) for x in r["ms_other_step_p50_p99_max"]])
PY
done
