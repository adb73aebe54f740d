#!/bin/bash
# 2D experiment: one body for column-partial chunks too (HEXS_MERGE_COLP=1) against the default.
tag=${1:-cp}
mkdir -p gpurun_out
L=paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil_colp.so
HEXS_LIB=$L timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k "2d" > gpurun_out/${tag}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_pytest.log
for c in heat2d5 heat2d9 gradient2d; do
  HEXS_LIB=$L timeout 300 python bench.py --config $c --no-cpu > gpurun_out/${tag}_colp_$c.json 2>> gpurun_out/${tag}.err
  timeout 300 python bench.py --config $c --no-cpu > gpurun_out/${tag}_main_$c.json 2>> gpurun_out/${tag}.err
done
timeout 900 python -m pytest tests/test_gpu_parity.py -x -q -k "tile_shapes" > gpurun_out/${tag}_shapes_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_shapes_pytest.log
