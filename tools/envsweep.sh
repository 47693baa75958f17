#!/bin/bash
# tools/envsweep.sh VAR "v1 v2 ..." "n1 n2 ..." : job_trace factor time per env value
VAR=$1; VALS=$2; NS=${3:-"3840 19200"}
for v in $VALS; do for n in $NS; do
  env $VAR=$v python tools/job_trace.py $n 1 2>/dev/null | python -c "
import json,sys; d=json.loads(sys.stdin.readline())
print('$VAR=$v', $n, 'factor_ms %.3f util %.3f' % (d['factor_ms'], d['utilisation']), ' '.join('%s %.1f' % (k, d[k]['mean_us']) for k in ['UPD','TRSM','DIAG','PANEL','PUPD','TS','TU'] if k in d))"
done; done
