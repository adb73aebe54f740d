for v in "HEXS_DIST_FUSED=1" "HEXS_DIST_FUSED=1 HEXS_DIST_MIRFENCE=0" "HEXS_DIST_FUSED=1 HEXS_DIST_FUSED_NOSTORE=1"; do
  env $v HEXS_DIST_EMULATE=3 HEXS_DIST_EMULATE_RANK=4/8 timeout 300 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu 2>/dev/null | python -c "
import json,sys
d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('P8 $v', round(d['ms_per_step'],2), d['roofline']['block_kernel_ms'])"
done
