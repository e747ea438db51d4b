#!/bin/bash
# small-batch path vs the multi-kernel path at B = 100 .. 4096 (under gpurun)
tag=${1:-x}
mkdir -p gpurun_out
for sm in 0 256 1024 2048; do
  echo "GPMA_SMALL=$sm" >> gpurun_out/${tag}_sweep.txt
  GPMA_SMALL=$sm timeout 300 python tools/small_batch_probe.py 100 500 1000 2000 2>&1 | grep "^B=" >> gpurun_out/${tag}_sweep.txt
done
