#!/bin/bash
# small-batch anatomy + cold launch list of one B=1000 slide (under gpurun)
tag=${1:-x}
mkdir -p gpurun_out
timeout 300 python tools/small_batch_probe.py 100 1000 > gpurun_out/${tag}_small.txt 2>&1
timeout 300 ncu --metrics gpu__time_duration.sum --clock-control none --kernel-name-base function -k regex:"^k_" -c 200 \
   --csv --log-file gpurun_out/${tag}_small_launches.csv python tools/small_batch_probe.py 1000 > /dev/null 2>&1
