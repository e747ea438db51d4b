#!/bin/bash
# analytics A/B (under gpurun): concurrent analytics and the CC / BFS strategy knobs
tag=${1:-x}
B="python bench.py --no-sweep --no-resize --no-e2e --no-cpu-baseline --steps 10"
for kv in "X=1" "GPMA_CC_SAMPLE=1" "GPMA_CC_SAMPLE=0" "GPMA_BFS_SPARSE=8192" "GPMA_BFS_SPARSE=131072"; do
  echo "$kv $(env $kv timeout 600 $B 2>/dev/null | tail -1 | python -c 'import json,sys; d=json.loads(sys.stdin.read()); print(round(d["ms_per_step"],3), {k: round(v,3) for k,v in d["breakdown_ms"].items() if isinstance(v,float)})')" >> gpurun_out/${tag}_analytics.txt
done
echo "concurrent $(timeout 600 $B --concurrent-analytics 2>/dev/null | tail -1 | python -c 'import json,sys; d=json.loads(sys.stdin.read()); print(round(d["ms_per_step"],3), {k: (round(v,3) if isinstance(v,float) else v) for k,v in d["breakdown_ms"].items()})')" >> gpurun_out/${tag}_analytics.txt
