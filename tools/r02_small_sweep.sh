#!/bin/bash
# small-batch slide latency vs the one-kernel threshold (under gpurun): tools/r02_small_sweep.sh <tag>
tag=${1:-x}
for lim in 0 256 2048; do
  echo "GPMA_SMALL=$lim" >> gpurun_out/${tag}_small.txt
  GPMA_SMALL=$lim python tools/small_batch_probe.py 100 256 512 1000 2000 2>&1 | grep "^B=" >> gpurun_out/${tag}_small.txt
done
