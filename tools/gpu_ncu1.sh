#!/bin/bash
# one full ncu capture of a kernel: tools/gpu_ncu1.sh TAG KERNEL_REGEX CONFIG
tag=$1; k=$2; c=$3
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on -k regex:$k -s 20 -c 1 \
  -o gpurun_out/${tag} python tools/run_once.py $c 1 > gpurun_out/${tag}_ncu.log 2>&1
