#!/bin/bash
# k_small_insert / k_small_delete at B=1000 (GPMA_SMALL=2048): timing + one full ncu capture with source
tag=${1:-x}
mkdir -p gpurun_out
GPMA_SMALL=2048 timeout 300 python tools/small_batch_probe.py 1000 2000 > gpurun_out/${tag}_small2048.txt 2>&1
GPMA_SMALL=2048 timeout 600 ncu --set full --import-source on --clock-control none -k regex:"k_small_insert|k_small_delete" -s 20 -c 2 \
   -o gpurun_out/${tag}_small python tools/small_batch_probe.py 1000 > gpurun_out/${tag}_small_ncu.log 2>&1
