export PYTHONUNBUFFERED=1
for n in 960 9600 19200; do CHOL_LIB_OVERRIDE=variants/hops.so timeout 60 python tools/phases_run.py factor $n; done > gpurun_out/hops2.txt 2>&1
timeout 900 python tools/libab.py 960,3840,7680,9600,11520,19200 variants/base.so variants/new.so --rounds 2 --reps 5 > gpurun_out/ab1.txt 2>&1
CHOL_LIB_OVERRIDE=variants/new.so timeout 60 python tools/chain_trace.py 1 3 --list > gpurun_out/chain_N1_new.txt 2>&1
CHOL_LIB_OVERRIDE=variants/new.so timeout 600 python -m pytest tests/test_gpu_production.py tests/test_gpu_sched.py -m gpu -x -q > gpurun_out/pytest_new.txt 2>&1
