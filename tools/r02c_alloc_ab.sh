#!/bin/bash
# big-block cache check (under gpurun): all GPU tests, the resize trace with allocation times,
# the bench resize stress with the cache on and off
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/al_tests.log 2>&1
echo "tests_rc=$?"; tail -2 gpurun_out/al_tests.log
GPMA_TRACE_ALLOC=1 timeout 900 python tools/resize_trace.py 3 > gpurun_out/al_tr.txt 2>&1
grep "^rep" gpurun_out/al_tr.txt
for c in 1 0 1; do
  GPMA_BLOCK_CACHE=$c timeout 600 python bench.py --steps 5 --warmup 3 --no-sweep --no-cpu-baseline --no-e2e > gpurun_out/al_bench_$c.json 2>/dev/null
  python -c "
import json; d=json.loads(open('gpurun_out/al_bench_$c.json').read().strip().splitlines()[-1]); r=d['resize_stress']; print('cache=$c', r['ms_resize_steps'], round(r['ms_other_step_mean'],3), round(d['ms_per_step'],3))"
done
