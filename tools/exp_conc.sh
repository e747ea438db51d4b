#!/bin/bash
# experiment: grid cap x stream priorities for the concurrent analytics step
mkdir -p gpurun_out
run() {  # name, env...
  name=$1; shift
  env "$@" python bench.py --no-sweep --no-cpu-baseline --no-e2e --steps 10 $EXTRA > gpurun_out/x_$name.json 2>/dev/null
  python - "$name" <<'PY'
import json,sys
n=sys.argv[1]
try:
    d=json.loads(open(f"gpurun_out/x_{n}.json").read().strip().splitlines()[-1])
    b=d["breakdown_ms"]; print(n, round(d["ms_per_step"],3), {k:(round(v,2) if isinstance(v,float) else v) for k,v in b.items() if k!="analytics"})
except Exception as e: print(n, "fail", e)
PY
}
EXTRA=--serial-analytics run serial_def GPMA_GRID_CAP=1184
EXTRA=--serial-analytics run serial_8k GPMA_GRID_CAP=8192
EXTRA= run conc_def GPMA_GRID_CAP=1184
EXTRA= run conc_def_prio GPMA_GRID_CAP=1184 GPMA_FAN_PRIO=0,-1,-2,0
EXTRA= run conc_8k GPMA_GRID_CAP=8192
EXTRA= run conc_8k_prio GPMA_GRID_CAP=8192 GPMA_FAN_PRIO=0,-1,-2,0
EXTRA= run conc_32k_prio GPMA_GRID_CAP=32768 GPMA_FAN_PRIO=0,-1,-2,0
EXTRA= run conc_2k_prio GPMA_GRID_CAP=2368 GPMA_FAN_PRIO=0,-1,-2,0
