mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for c in 1 1 1 0; do
  GPMA_BLOCK_CACHE=$c timeout 600 python bench.py --steps 5 --warmup 3 --no-sweep --no-cpu-baseline --no-e2e > gpurun_out/al2_bench_$c.json 2>/dev/null
  python -c "
import json; d=json.loads(open('gpurun_out/al2_bench_$c.json').read().strip().splitlines()[-1]); r=d['resize_stress']; print('cache=$c', r['ms_resize_steps'], round(r['ms_other_step_mean'],3), round(d['ms_per_step'],3))"
done
