#!/bin/bash
# Update-path A/B of the strategy knobs + a warm launch list (under gpurun): tools/r02_probe_knobs.sh <tag>
tag=${1:-x}
mkdir -p gpurun_out
for kv in "X=1" "GPMA_DEL_SORT=1" "GPMA_INS_LEAFSORT=0" "GPMA_INS_THREAD=0" "GPMA_INS_FUSED=0"; do
  echo "$kv $(env $kv python tools/upd_probe.py --slides 10 2>&1 | tail -1 | cut -c1-120)" >> gpurun_out/${tag}_knobs.txt
done
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --cache-control none --kernel-name-base function -k regex:"^k_" -c 600 --csv --log-file gpurun_out/${tag}_warm_launches.csv \
    python tools/upd_probe.py --slides 6 > /dev/null 2>&1
echo "ncu_rc=$?"
