export PYTHONUNBUFFERED=1
timeout 900 python -m pytest tests/test_gpu_sched.py -m gpu -x -q -k "block_level or trace_respects" > gpurun_out/pytest_jt.txt 2>&1
