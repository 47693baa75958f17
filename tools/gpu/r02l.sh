export CHOL_WATCHDOG_S=10
timeout 600 python -m pytest tests/test_gpu_sched.py tests/test_gpu_solve.py -m gpu -v -x > gpurun_out/pytest_l.log 2>&1
tail -5 gpurun_out/pytest_l.log
