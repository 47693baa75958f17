set -x
timeout 1200 python -m pytest tests/test_gpu_dist.py tests/test_gpu_production.py -m gpu -q -x 2>&1 | tail -5
python bench.py --logical-ranks 2 --n 19200 --steps 3 --warmup 2 2>&1 | tail -1
python bench.py --logical-ranks 4 --n 19200 --steps 3 --warmup 2 2>&1 | tail -1
python bench.py --logical-ranks 8 --n 38400 --steps 2 --warmup 1 2>&1 | tail -1
