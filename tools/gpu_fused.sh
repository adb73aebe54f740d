mkdir -p gpurun_out/loop
timeout 600 python -m pytest tests/test_gpu_parity.py -q -m gpu -k "loopback or dist_plan" -p no:cacheprovider > gpurun_out/loop/pytest.txt 2>&1; echo "rc=$?" >> gpurun_out/loop/pytest.txt
tail -6 gpurun_out/loop/pytest.txt
for v in "HEXS_DIST_FUSED=1" "HEXS_DIST_FUSED=1 HEXS_DIST_FUSED_NOSTORE=1" "HEXS_DIST_FUSED=0"; do
  env $v HEXS_DIST_EMULATE=3 HEXS_DIST_EMULATE_RANK=1/2 timeout 300 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu 2>/dev/null | python -c "
import json,sys
d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('$v', round(d['ms_per_step'],2), d['roofline']['block_kernel_ms'])"
done
mkdir -p gpurun_out/r2f
for P in 2 4 8; do
  r=$((P/2))
  for F in 1 0; do
  HEXS_DIST_FUSED=$F HEXS_DIST_EMULATE=3 HEXS_DIST_EMULATE_RANK=$r/$P timeout 300 python bench.py --config heat3d1024 --steps 2 --warmup 3 --no-cpu > gpurun_out/r2f/emu3_F${F}_P$P.json 2>gpurun_out/r2f/emu3_F${F}_P$P.err
  python -c "
import json
d=json.loads(open('gpurun_out/r2f/emu3_F${F}_P$P.json').read().strip().splitlines()[-1]); e=d['emulated_rank']
print('mode 3 fused=$F', $P, e['rank'], round(d['ms_per_step'],2), d['config']['local_extents'], d['config']['halo_exchange'])"
  done
done
