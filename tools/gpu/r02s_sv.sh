export PYTHONUNBUFFERED=1
timeout 600 python -m pytest tests/test_gpu_solve.py -m gpu -x -q > gpurun_out/pytest_sv.txt 2>&1
for lib in variants/pf2.so variants/sv2.so; do echo $lib; CHOL_LIB_OVERRIDE=$lib timeout 300 python tools/solve_bench.py 19200 1,96,192,960; CHOL_LIB_OVERRIDE=$lib timeout 300 python tools/solve_bench.py 46080 96,960; done > gpurun_out/solve_ab.txt 2>&1
