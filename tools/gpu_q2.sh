for t in 2,7 3,7 3,5 2,5; do
timeout 600 python bench.py --config heat3d27 --steps 3 --warmup 3 --no-cpu --tile $t 2>/dev/null | python -c "
import json,sys
d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('box27 $t', round(d['value'],1), round(d['naive_gups'],1), round(d['speedup_vs_naive'],3), d['config']['tile'])"
done
for t in 2,7 3,7 1,7; do
timeout 600 python bench.py --config gradient3d --steps 3 --warmup 3 --no-cpu --tile $t 2>/dev/null | python -c "
import json,sys
d=json.loads(sys.stdin.read().strip().splitlines()[-1]); print('grad3d $t', round(d['value'],1), round(d['naive_gups'],1), round(d['speedup_vs_naive'],3), d['config']['tile'])"
done
