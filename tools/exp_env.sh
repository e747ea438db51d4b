#!/bin/bash
# experiment: run the serial bench (profiled warm step) under several env settings and
# print step time + the listed kernels.  usage: exp_env.sh "kern1,kern2" "ENV=a ENV2=b" "ENV=c" ...
mkdir -p gpurun_out
kern=$1; shift
i=0
for setting in "$@"; do
  env $setting python bench.py --no-sweep --no-cpu-baseline --no-e2e --steps 5 --profile-all > gpurun_out/env_$i.json 2>gpurun_out/env_$i.err
  python - "$i" "$setting" "$kern" <<'PY'
import json,sys
i,setting,kern=sys.argv[1],sys.argv[2],sys.argv[3].split(",")
try:
    d=json.loads(open(f"gpurun_out/env_{i}.json").read().strip().splitlines()[-1])
    t=d["kernel_table_warm_step"]
    print(f"[{setting}] step {d['ms_per_step']:.3f}", {k: round(t[k]["ms"],3) for k in kern if k in t},
          {k:round(v,3) for k,v in d["breakdown_ms"].items() if isinstance(v,float)})
except Exception as e: print(setting, "fail", e, open(f"gpurun_out/env_{i}.err").read()[-500:])
PY
  i=$((i+1))
done
