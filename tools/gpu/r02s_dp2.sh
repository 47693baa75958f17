export PYTHONUNBUFFERED=1
timeout 1200 python tools/libab.py 960,3840,5760,7680,9600,11520,19200 variants/base2.so variants/dp2.so variants/dp2.so:CHOL_POTRF_DP=0 --rounds 2 --reps 5 > gpurun_out/ab_dp2.txt 2>&1
CHOL_LIB_OVERRIDE=variants/dp2.so timeout 120 python tools/chain_trace.py 1 5 --list > gpurun_out/chain_N1_dp2.txt 2>&1
