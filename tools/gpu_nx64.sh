#!/bin/bash
# 3D tile-shape experiment: 16 lines x 64 columns (NX = 64 build) against 16 x 32 and 32 x 32.
tag=${1:-nx}
mkdir -p gpurun_out
L=paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil_nx64.so
HEXS_LIB=$L timeout 300 python tools/nx64_check.py > gpurun_out/${tag}_check.log 2>&1
HEXS_LIB=$L timeout 300 python bench.py --config heat3d --no-cpu --tile 3,7,16 > gpurun_out/${tag}_nx64.json 2>> gpurun_out/${tag}.err
timeout 300 python bench.py --config heat3d --no-cpu --tile 3,7,16 > gpurun_out/${tag}_nx32_ny16.json 2>> gpurun_out/${tag}.err
timeout 300 python bench.py --config heat3d --no-cpu > gpurun_out/${tag}_default.json 2>> gpurun_out/${tag}.err
