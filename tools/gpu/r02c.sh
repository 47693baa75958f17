set -x
for m in factor batch; do
  CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py $m 46080
  CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py $m 19200
done
python tools/phases_run.py factor 46080
python tools/phases_run.py batch 46080
python tools/phases_run.py batch 46080 540
