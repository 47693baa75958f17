export CHOL_WATCHDOG_S=15
timeout 60 python tools/hetero_debug.py 8 3 2>&1 | tail -6; echo rc=$?
timeout 60 python tools/hetero_debug.py 12 6 2>&1 | tail -6; echo rc=$?
