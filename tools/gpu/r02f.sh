set -x
timeout 1500 python -m pytest tests -m gpu -q 2>&1 | tail -25
python tools/env_time.py 9600,19200,46080 ""
python tools/job_trace.py 19200 0 2>&1 | tail -3
