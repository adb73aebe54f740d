#!/bin/bash
# FDTD chunk-shape experiments (experiment builds): parity subset + bench line at the (11, 5) tile.
tag=${1:-fs}
mkdir -p gpurun_out
for v in main rp2 c128rp2 c128rp2nb3 c32rp8; do
  if [ $v = main ]; then lib=""; else lib=paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil_$v.so; fi
  HEXS_LIB=$lib timeout 600 python -m pytest tests/test_gpu_parity.py -x -q -k "fdtd_fast_kernel or full_size_fdtd" > gpurun_out/${tag}_${v}_pytest.log 2>&1; echo "rc=$?" >> gpurun_out/${tag}_${v}_pytest.log
  HEXS_LIB=$lib timeout 300 python bench.py --config fdtd2d --no-cpu --tile 11,5 > gpurun_out/${tag}_${v}_bench.json 2>> gpurun_out/${tag}.err
done
