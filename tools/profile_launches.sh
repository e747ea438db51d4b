#!/bin/bash
# Launch list of the bench command (per-launch device time + DRAM bytes of every k_* launch)
# usage (GPU box): tools/profile_launches.sh <tag>
tag=${1:-r01}
mkdir -p gpurun_out
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --kernel-name-base function -k regex:"^k_" -c 4000 --csv --log-file gpurun_out/launches_$tag.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep --no-resize > gpurun_out/launches_bench_$tag.log 2>&1
