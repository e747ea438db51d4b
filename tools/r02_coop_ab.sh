#!/bin/bash
# pending segsort + coop CTAs A/B (under gpurun)
tag=${1:-x}
mkdir -p gpurun_out
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_edge_cases.py -m gpu -q -x > gpurun_out/${tag}_tests.txt 2>&1
echo "rc=$?" >> gpurun_out/${tag}_tests.txt
for kv in "GPMA_COOP_CTAS=1" "GPMA_COOP_CTAS=2" "GPMA_COOP_CTAS=4"; do
  echo "$kv $(env $kv timeout 300 python tools/upd_probe.py --slides 25 2>&1 | tail -1 | cut -c1-100)" >> gpurun_out/${tag}_coop.txt
  echo "$kv $(env $kv timeout 300 python tools/resize_steps_ab.py --grow 40 2>&1 | tail -1)" >> gpurun_out/${tag}_coop.txt
done
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --cache-control none --kernel-name-base function -k regex:"^k_" -c 2000 --csv --log-file gpurun_out/${tag}_warm_launches.csv \
    python tools/upd_probe.py --slides 22 > /dev/null 2>&1
