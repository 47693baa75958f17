timeout 600 python -m pytest tests/test_gpu_solve.py -m gpu -q 2>&1 | tail -2
CHOL_SOLVE_RC=32 python tools/solve_bench.py 19200 33,96,192,960
python tools/solve_bench.py 19200 33,96,192,960
python tools/solve_bench.py 46080 96,960
