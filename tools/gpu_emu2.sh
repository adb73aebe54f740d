#!/bin/bash
# Multi-GPU projection with the session-2 3D kernel (16 x 64 tiles): one rank's slab of heat-3D
# 1024^3 per call (HEXS_DIST_EMULATE_RANK=r/P), compute only (=1) and with the device-initiated
# exchange kernels (=3); N = 1 through the dist path for the baseline.
tag=${1:-emu2}
mkdir -p gpurun_out/$tag
timeout 400 python bench.py --config heat3d1024 --no-cpu > gpurun_out/$tag/P1.json 2>> gpurun_out/$tag/err.txt
for rp in 1/2 2/4 4/8; do
  P=${rp#*/}; r=${rp%/*}
  for m in 1 3; do
    HEXS_DIST_EMULATE=$m HEXS_DIST_EMULATE_RANK=$rp timeout 400 python bench.py --config heat3d1024 --steps 3 --warmup 3 --no-cpu \
      > gpurun_out/$tag/emu${m}_r${r}_P${P}.json 2>> gpurun_out/$tag/err.txt
  done
done
