for v in s3t; do
  HEXS_LIB=paper_conf_cgo_grosserchsv14_b200/lib/libhexstencil_$v.so python tools/s3_trace.py 512 6 > gpurun_out/trace_$v.txt 2>&1
  echo "== $v"; grep "span" gpurun_out/trace_$v.txt; grep -A4 "per-warp" gpurun_out/trace_$v.txt
done
