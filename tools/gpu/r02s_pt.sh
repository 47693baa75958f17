export PYTHONUNBUFFERED=1
for i in 1 2 3; do variants/bin/pt_old; variants/bin/pt_new; done > gpurun_out/potf2_total.txt 2>&1
CHOL_LIB_OVERRIDE=variants/pf.so timeout 60 python tools/chain_trace.py 1 5 --list > gpurun_out/chain_N1_pf.txt 2>&1
CHOL_LIB_OVERRIDE=variants/pf.so timeout 120 python tools/chain_trace.py 10 3 --list > gpurun_out/chain_N10_pf.txt 2>&1
