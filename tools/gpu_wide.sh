#!/bin/bash
# Wide 3D tiles (16 x 64, 8 x 128) and the FDTD predicated-store slots: parity + bench lines.
tag=${1:-wd}
mkdir -p gpurun_out
timeout 300 python tools/nx64_check.py > gpurun_out/${tag}_check.log 2>&1
timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k fdtd > gpurun_out/${tag}_fdtd_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_fdtd_pytest.log
timeout 300 python bench.py --config fdtd2d --no-cpu > gpurun_out/${tag}_fdtd2d.json 2>> gpurun_out/${tag}.err
for t in 3,7,16 3,7,8 2,7,16 3,7,32; do
  timeout 300 python bench.py --config heat3d --no-cpu --tile $t >> gpurun_out/${tag}_heat3d.json 2>> gpurun_out/${tag}.err
done
for t in 2,7,16 2,7,32; do
  timeout 300 python bench.py --config heat3d27 --no-cpu --tile $t >> gpurun_out/${tag}_heat3d27.json 2>> gpurun_out/${tag}.err
  timeout 300 python bench.py --config gradient3d --no-cpu --tile $t >> gpurun_out/${tag}_gradient3d.json 2>> gpurun_out/${tag}.err
done
