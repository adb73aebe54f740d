#!/bin/bash
# FDTD build-variant comparison: parity subset + bench line per experiment library.
tag=${1:-fdv}
mkdir -p gpurun_out
for v in main rp2 ring3 nopair; do
  if [ $v = main ]; then lib=""; else lib=paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil_$v.so; fi
  HEXS_LIB=$lib timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k fdtd > gpurun_out/${tag}_${v}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_${v}_pytest.log
  HEXS_LIB=$lib timeout 300 python bench.py --config fdtd2d --no-cpu > gpurun_out/${tag}_${v}_bench.json 2>> gpurun_out/${tag}_bench.err
done
