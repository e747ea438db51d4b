#!/bin/bash
# A/B of GPMA_ILP (keys per thread of the random-probe kernels) + ncu of the leaf kernel (under gpurun)
tag=${1:-x}
mkdir -p gpurun_out
for kv in "GPMA_ILP=1" "GPMA_ILP=2" "GPMA_ILP=4"; do
  echo "$kv $(env $kv python tools/upd_probe.py --slides 10 2>&1 | tail -1 | cut -c1-100)" >> gpurun_out/${tag}_ilp.txt
done
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"k_ins_leaf_u|k_locate_u_r|k_lazy_delete_r" -s 6 -c 6 \
   -o gpurun_out/${tag}_full python tools/upd_probe.py --slides 4 > gpurun_out/${tag}_ncu.log 2>&1
echo "ncu_rc=$?"
