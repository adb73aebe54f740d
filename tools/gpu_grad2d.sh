#!/bin/bash
# gradient2d with the merged column-partial body: parity + tile sweep; heat2d5 unchanged check.
tag=${1:-g2}
mkdir -p gpurun_out
timeout 600 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q -k "gradient2d or 2d_small" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for t in 1,1 1,3 2,3; do
  timeout 300 python bench.py --config gradient2d --no-cpu --tile $t >> gpurun_out/${tag}_sweep.json 2>> gpurun_out/${tag}.err
done
timeout 300 python bench.py --config heat2d5 --no-cpu > gpurun_out/${tag}_heat2d5.json 2>> gpurun_out/${tag}.err
