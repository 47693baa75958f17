set -x
CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py factor 46080
CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py batch 46080
python tools/clock_batch.py 46080
