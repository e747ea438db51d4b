#!/bin/bash
# ncu evidence for profiles/: (1) per-launch device times of the bench command (launch list),
# (2) one --set full capture of the dominant kernels.  Run under gpurun (1 GPU).
set -x
mkdir -p gpurun_out
ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --kernel-name-base function -k regex:"^k_" -c 3000 --csv --log-file gpurun_out/launches_r01.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep --no-resize > gpurun_out/launches_bench.log 2>&1
ncu --set full --clock-control none --import-source on --kernel-name-base function \
    -k regex:"k_pr_push_win|k_cc_sample|k_cc_hook|k_exp_write|k_bfs_sweep|k_level0|k_lazy_delete|k_prepass" \
    -s 30 -c 10 -o gpurun_out/full_r01 \
    python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep --no-resize > gpurun_out/full_bench.log 2>&1
ls -la gpurun_out
