#!/bin/bash
# device level loop pending limit: configs[2] step, configs[1] sweep, configs[3] resize stress
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for kv in "X=1" "GPMA_COOP_MAXP=262144" "GPMA_COOP_MAXP=65536" "X=1" "GPMA_COOP_MAXP=262144"; do
  env $kv timeout 900 python bench.py --steps 20 --warmup 5 --no-cpu-baseline --no-e2e > gpurun_out/mp_$kv.json 2>/dev/null
  python -c "
import json; d=json.loads(open('gpurun_out/mp_$kv.json').read().strip().splitlines()[-1]); r=d['resize_stress']; b=d['batch_sweep']
print('$kv', 'step %.3f' % d['ms_per_step'], 'ins %.4f' % d['breakdown_ms']['insert'], 'resize', r['ms_resize_steps'], 'mean %.3f' % r['ms_per_step_mean'], 'sweep', [round(p['gpma_plus']['ms_per_slide_mean'],4) for p in b['points']])"
done
