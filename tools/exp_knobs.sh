run() { python bench.py --steps 6 --warmup 2 --profile-all --no-cpu-baseline --no-e2e 2>&1 | tail -1 | python -c "import json,sys; d=json.loads(sys.stdin.read()); t=d['kernel_table_warm_step']; print('$1', round(d['ms_per_step'],2), {k: round(v,2) for k,v in d['breakdown_ms'].items()}, {k:(v['launches'], round(v['ms'],3)) for k,v in t.items() if k.startswith(('k_pr_push','k_cc_','k_bfs_sweep'))})"; }
for P in 1 2 3 4; do GPMA_PR_PASSES=$P run "P=$P"; done
for M in 0 1 2; do GPMA_CC_MODE=$M run "CC=$M"; done
