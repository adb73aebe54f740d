#!/bin/bash
# 2D drift mode (no CTA barrier per level) against the default: parity + bench lines.
tag=${1:-dr}
mkdir -p gpurun_out
L=paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil_drift.so
HEXS_LIB=$L timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fullsize.py -x -q -k "2d" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for c in heat2d5 heat2d9 gradient2d; do
  HEXS_LIB=$L timeout 300 python bench.py --config $c --no-cpu > gpurun_out/${tag}_drift_$c.json 2>> gpurun_out/${tag}.err
  timeout 300 python bench.py --config $c --no-cpu > gpurun_out/${tag}_main_$c.json 2>> gpurun_out/${tag}.err
done
