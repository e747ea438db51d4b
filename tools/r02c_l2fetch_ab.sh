mkdir -p gpurun_out
nvcc -O3 -gencode arch=compute_100a,code=sm_100a -o /tmp/rand_bw tools/micro/rand_bw.cu && /tmp/rand_bw > gpurun_out/rand_bw4.jsonl 2>&1
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
for gr in "" 32 64 128; do
  GPMA_L2_FETCH=$gr timeout 600 python bench.py --steps 20 --warmup 5 --no-sweep --no-resize --no-cpu-baseline --no-e2e > gpurun_out/gr_${gr:-def}.json 2> gpurun_out/gr_${gr:-def}.err
  echo "gr=$gr rc=$?"
done
