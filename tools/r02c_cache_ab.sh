#!/bin/bash
# block cache on / off: the bench with the configs[1] sweep and the configs[3] resize stress
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for c in 1 1 1; do
  GPMA_BLOCK_CACHE=$c timeout 900 python bench.py --steps 10 --warmup 5 --no-cpu-baseline --no-e2e > gpurun_out/ca_$c.json 2>/dev/null
  python -c "
import json; d=json.loads(open('gpurun_out/ca_$c.json').read().strip().splitlines()[-1]); r=d['resize_stress']; b=d['batch_sweep']
print('cache=$c', 'step %.3f' % d['ms_per_step'], 'resize', r['ms_resize_steps'], round(r['ms_other_step_mean'],3), 'sweep', [round(p['gpma_plus']['ms_per_slide_mean'],4) for p in b['points']], b['analytics_after_update_ms'])"
done
