set -x
python tools/phases_run.py factor 46080
python tools/phases_run.py factor 19200
CHOL_LIB_OVERRIDE=variants/phases_tma.so python tools/phases_run.py factor 46080
timeout 1200 python -m pytest tests -m gpu -q -x -k "parity or production or sched or dist or solve" 2>&1 | tail -5
python tools/env_time.py 19200,46080 ""
