#!/bin/bash
# Round-2 last pass (under gpurun, 1 GPU): build, smoke, the default bench line with its per-slide
# log, and the launch list of one bench step (the kernels' share of the step).
tag=${1:-r02d}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/${tag}_build.log 2>&1; echo "build_rc=$?"
timeout 300 python __graft_entry__.py smoke > gpurun_out/${tag}_smoke.log 2>&1; echo "smoke_rc=$?"
timeout 1500 python bench.py --log-jsonl gpurun_out/${tag}_slides.jsonl > gpurun_out/${tag}_bench.json 2> gpurun_out/${tag}_bench.err
echo "bench_rc=$?"
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --cache-control none --kernel-name-base function -k regex:"^k_" -c 3000 --csv --log-file gpurun_out/${tag}_launches.csv \
    python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep --no-resize > gpurun_out/${tag}_launches_bench.log 2>&1
echo "launches_rc=$?"
