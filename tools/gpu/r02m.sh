export CHOL_WATCHDOG_S=20
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -6
unset CHOL_WATCHDOG_S
python tools/env_time.py 9600,19200,46080 ""
CHOL_LIB_OVERRIDE=variants/phases.so python tools/phases_run.py factor 46080
