export PYTHONUNBUFFERED=1
for n in 960 9600 19200; do CHOL_LIB_OVERRIDE=variants/hops.so timeout 60 python tools/phases_run.py factor $n; done > gpurun_out/hops.txt 2>&1
timeout 120 python tools/chain_trace.py 10 3 --list > gpurun_out/chain_N10.txt 2>&1
timeout 60 python tools/chain_trace.py 1 3 --list > gpurun_out/chain_N1.txt 2>&1
