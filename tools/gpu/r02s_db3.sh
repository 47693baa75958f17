export PYTHONUNBUFFERED=1
for rc in 32 48; do echo RC=$rc; CHOL_SOLVE_RC=$rc timeout 300 python tools/solve_bench.py 19200 2,8,24,33,48,64; CHOL_SOLVE_RC=$rc timeout 300 python tools/solve_bench.py 46080 8,48; done > gpurun_out/solve_db3.txt 2>&1
