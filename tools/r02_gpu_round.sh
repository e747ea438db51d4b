#!/bin/bash
# One GPU round trip (run under gpurun): build, GPU tests, bench line, launch list of one step.
# usage: tools/r02_gpu_round.sh <tag> [pytest -k expr]
tag=${1:-x}; kexpr=${2:-}
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/${tag}_build.log 2>&1
if [ -n "$kexpr" ]; then
  timeout 900 python -m pytest tests -m gpu -x -q -k "$kexpr" > gpurun_out/${tag}_tests.log 2>&1
else
  timeout 900 python -m pytest tests -m gpu -x -q > gpurun_out/${tag}_tests.log 2>&1
fi
echo "tests_rc=$?"; tail -3 gpurun_out/${tag}_tests.log
timeout 600 python bench.py --steps 20 --warmup 5 --no-sweep --no-resize --no-cpu-baseline --no-e2e > gpurun_out/${tag}_bench.json 2> gpurun_out/${tag}_bench.err
echo "bench_rc=$?"; tail -2 gpurun_out/${tag}_bench.err
timeout 600 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none \
    --kernel-name-base function -k regex:"^k_" -c 1500 --csv --log-file gpurun_out/${tag}_launches.csv \
    python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline --no-sweep --no-resize > gpurun_out/${tag}_launches_bench.log 2>&1
echo "ncu_rc=$?"
