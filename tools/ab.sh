#!/bin/bash
# A/B the library variants under variants/ with tools/job_trace.py (factor time + per-type job means);
# usage: tools/ab.sh [rounds] [n ...]
R=${1:-1}; shift; NS=${@:-3840 19200}
for r in $(seq $R); do
for lib in variants/*.so; do
  for n in $NS; do
    CHOL_LIB_OVERRIDE=$lib python tools/job_trace.py $n 1 2>/dev/null | python -c "
import json,sys; d=json.loads(sys.stdin.readline())
print('$lib', $n, 'factor_ms %.3f util %.3f' % (d['factor_ms'], d['utilisation']), ' '.join('%s %.1f' % (k, d[k]['mean_us']) for k in ['UPD','TRSM','DIAG','PANEL','PUPD','TS','TU'] if k in d))"
  done
done
done
