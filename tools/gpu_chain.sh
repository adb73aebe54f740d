#!/bin/bash
# Chained 3D launches: a short smoke first (bounded), then the 3D parity suite and bench lines.
tag=${1:-ch}
mkdir -p gpurun_out
timeout 120 python -m pytest tests/test_gpu_parity.py -x -q -k "test_3d and star3d7 and float32" > gpurun_out/${tag}_quick.log 2>&1
rc=$?; echo "rc=$rc" >> gpurun_out/${tag}_quick.log
if [ $rc -ne 0 ]; then exit 0; fi
timeout 1500 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q -k "3d" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for c in heat3d gradient3d heat3d27 heat3d1024; do
  timeout 400 python bench.py --config $c --no-cpu > gpurun_out/${tag}_bench_$c.json 2>> gpurun_out/${tag}_bench.err
done
HEXS_F3_CHAIN=0 timeout 300 python bench.py --config heat3d --no-cpu > gpurun_out/${tag}_bench_heat3d_nochain.json 2>> gpurun_out/${tag}_bench.err
