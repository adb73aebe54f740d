#!/bin/bash
# usage: tools/sweep.sh CONFIG "h,w0 h,w0 ..."  -> one bench line per tile (no CPU baseline)
cfg=$1; shift
for t in $@; do
  python bench.py --config $cfg --steps 3 --warmup 3 --no-cpu --tile $t 2>&1 | python -c "
import sys,json
for l in sys.stdin:
    if l.startswith('{'):
        d=json.loads(l); r=d['roofline']
        print('$t', 'GUp/s=%.0f naive=%.0f x%.2f launch=%.3fms frac=%.3f fast=%s' % (d['value'], d['naive_gups'], d['speedup_vs_naive'], r['avg_launch_ms'], r['frac'], r['kernel']))
    elif 'Error' in l or 'error' in l: print('$t', l.strip())
"
done
