#!/bin/bash
# configs[3] ordinary steps under the insert / level-loop knobs (under gpurun)
tag=${1:-x}
for kv in "X=1" "GPMA_INS_LEAFSORT=0" "GPMA_LVL_COOP=0" "GPMA_LVL_COOP=0 GPMA_GATHER_BIG=0" "GPMA_LVL_COOP=0 GPMA_LVL_SMALL=0"; do
  echo "$kv $(env $kv timeout 300 python tools/resize_steps_ab.py --grow 40 2>&1 | tail -1)" >> gpurun_out/${tag}_c3ab.txt
done
