export PYTHONUNBUFFERED=1
CHOL_SOLVE_RC=48 timeout 600 python -m pytest tests/test_gpu_solve.py -m gpu -x -q > gpurun_out/pytest_db.txt 2>&1
for rc in 64 48; do echo RC=$rc; CHOL_SOLVE_RC=$rc timeout 300 python tools/solve_bench.py 19200 192,960; CHOL_SOLVE_RC=$rc timeout 300 python tools/solve_bench.py 46080 192,960; done > gpurun_out/solve_db.txt 2>&1
