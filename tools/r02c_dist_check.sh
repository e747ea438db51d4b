#!/bin/bash
# the bench's other arms (under gpurun, one GPU): the sharded path at N = 1 over NCCL, the N = 2
# logic with both ranks on cuda:0 over gloo (correctness of the N > 1 code path only -- not a
# timing), and the reference arm (the oracle)
mkdir -p gpurun_out
python -c "import __graft_entry__ as g; g.build()" > /dev/null 2>&1
timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 1 --master-addr 127.0.0.1 --master-port 29511 \
  bench.py --force-dist --steps 3 --warmup 3 --no-e2e > gpurun_out/dist1.json 2> gpurun_out/dist1.err
echo "dist1 rc=$?"; tail -c 600 gpurun_out/dist1.json; echo
GPMA_BENCH_SHARE_GPU=1 timeout 900 python -m torch.distributed.run --nnodes=1 --nproc-per-node 2 --master-addr 127.0.0.1 \
  --master-port 29512 bench.py --gpus 2 --steps 2 --warmup 3 --no-e2e > gpurun_out/dist2.json 2> gpurun_out/dist2.err
echo "dist2 rc=$?"; tail -c 600 gpurun_out/dist2.json; echo
timeout 900 python bench.py --impl reference --steps 2 --warmup 3 > gpurun_out/ref.json 2> gpurun_out/ref.err
echo "ref rc=$?"; tail -c 600 gpurun_out/ref.json; echo
