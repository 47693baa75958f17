export PYTHONUNBUFFERED=1
CHOL_LIB_OVERRIDE=variants/phases.so timeout 120 python tools/phases_run.py factor 19200 > gpurun_out/tphases.txt 2>&1
timeout 120 python tools/chain_trace.py 10 3 --list > gpurun_out/chain_N10_b.txt 2>&1
