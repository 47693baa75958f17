export PYTHONUNBUFFERED=1
timeout 600 python -m pytest tests/test_gpu_solve.py -m gpu -x -q > gpurun_out/pytest_db2.txt 2>&1
for rc in 32 48; do echo RC=$rc; CHOL_SOLVE_RC=$rc timeout 300 python tools/solve_bench.py 19200 96,128,160; done > gpurun_out/solve_db2.txt 2>&1
timeout 300 python tools/solve_bench.py 46080 1,96,960 >> gpurun_out/solve_db2.txt 2>&1
