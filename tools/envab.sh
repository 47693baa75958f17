#!/bin/bash
# tools/envab.sh "ENV1=a ENV2=b" "ENV1=c" ... -- n1 n2 : job_trace per env setting (current library)
SETS=(); while [ "$1" != "--" ] && [ -n "$1" ]; do SETS+=("$1"); shift; done; shift; NS=${@:-"9600 19200"}
for set in "${SETS[@]}"; do for n in $NS; do
  env $set python tools/job_trace.py $n 1 2>/dev/null | python -c "
import json,sys; d=json.loads(sys.stdin.readline())
print('$set', $n, 'factor_ms %.3f util %.3f' % (d['factor_ms'], d['utilisation']), ' '.join('%s %.1f' % (k, d[k]['mean_us']) for k in ['UPD','TRSM','DIAG','PANEL','PUPD','TS','TU'] if k in d))"
done; done
