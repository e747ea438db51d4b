#!/bin/bash
# experiment: per-kernel time vs grid cap (serial analytics, profiled warm step)
mkdir -p gpurun_out
for cap in 1184 2368 4736 9472 18944; do
  GPMA_GRID_CAP=$cap python bench.py --no-sweep --no-cpu-baseline --no-e2e --steps 5 --serial-analytics --profile-all > gpurun_out/cap_$cap.json 2>/dev/null
done
python - <<'PY'
import json
caps=[1184,2368,4736,9472,18944]
T={}
for c in caps:
    d=json.loads(open(f"gpurun_out/cap_{c}.json").read().strip().splitlines()[-1])
    print(c, round(d["ms_per_step"],3))
    for k,v in d["kernel_table_warm_step"].items(): T.setdefault(k,{})[c]=v["ms"]
for k,row in sorted(T.items(), key=lambda kv:-kv[1].get(1184,0))[:25]:
    print(f"{k:28s}", " ".join(f"{row.get(c,0):7.3f}" for c in caps))
PY
