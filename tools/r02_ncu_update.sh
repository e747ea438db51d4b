#!/bin/bash
# ncu --set full of the update kernels (under gpurun): tools/r02_ncu_update.sh <tag> <kernel regex>
tag=${1:-x}; kre=${2:-"k_ins_leaf|k_del_mark|k_os_pass|k_locate"}
mkdir -p gpurun_out
python tools/upd_probe.py --slides 8 > gpurun_out/${tag}_probe.json 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"$kre" -s 10 -c 6 \
   -o gpurun_out/${tag}_full python tools/upd_probe.py --slides 4 > gpurun_out/${tag}_ncu.log 2>&1
echo "ncu_rc=$?"
