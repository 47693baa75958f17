set -x
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -8
python tools/env_time.py 3840,9600,19200,46080 ""
CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py factor 46080
python tools/job_trace.py 19200 0 2>&1 | tail -2 | head -1 | cut -c1-900
