export PYTHONUNBUFFERED=1
CHOL_LIB_OVERRIDE=variants/dbB.so timeout 600 python -m pytest tests/test_gpu_solve.py -m gpu -x -q > gpurun_out/pytest_db6.txt 2>&1
for lib in dbA dbB; do echo $lib; CHOL_LIB_OVERRIDE=variants/$lib.so timeout 300 python tools/solve_bench.py 19200 48,96,192,960; CHOL_LIB_OVERRIDE=variants/$lib.so timeout 300 python tools/solve_bench.py 46080 96,960; done > gpurun_out/solve_db6.txt 2>&1
