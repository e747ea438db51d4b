#!/bin/bash
# every GPU test, then the bench (no sweep / e2e / cpu baseline) twice
mkdir -p gpurun_out
tag=${1:-full}
python -c "import __graft_entry__ as g; g.build()" > gpurun_out/${tag}_build.log 2>&1 || { tail -20 gpurun_out/${tag}_build.log; exit 1; }
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/${tag}_tests.log 2>&1
echo "tests_rc=$?"; tail -3 gpurun_out/${tag}_tests.log
for r in 1 2; do
  timeout 600 python bench.py --steps 20 --warmup 5 --no-sweep --no-cpu-baseline --no-e2e > gpurun_out/${tag}_bench_$r.json 2>/dev/null
  python -c "
import json; d=json.loads(open('gpurun_out/${tag}_bench_$r.json').read().strip().splitlines()[-1]); r=d['resize_stress']
print('run $r', 'ms/step %.3f' % d['ms_per_step'], {k: round(v, 4) for k, v in d['breakdown_ms'].items() if isinstance(v, float)}, 'upd %.4f' % d['update_only']['ms_per_slide'], 'resize', r['ms_resize_steps'], round(r['ms_other_step_mean'], 3))"
done
