export PYTHONUNBUFFERED=1
timeout 600 python -m pytest tests/test_gpu_solve.py -m gpu -x -q > gpurun_out/pytest_db8.txt 2>&1
timeout 300 python tools/solve_bench.py 19200 33,96,192,960 > gpurun_out/solve_db8.txt 2>&1
timeout 300 python tools/solve_bench.py 46080 96,960 >> gpurun_out/solve_db8.txt 2>&1
