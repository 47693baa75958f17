export CHOL_WATCHDOG_S=30
timeout 1500 python -m pytest tests -m gpu -q -x 2>&1 | tail -4
python bench.py --logical-ranks 2 --n 19200 --steps 3 --warmup 2 2>&1 | tail -1 | cut -c1-200
python bench.py --logical-ranks 4 --n 19200 --steps 3 --warmup 2 2>&1 | tail -1 | cut -c1-200
python bench.py --logical-ranks 4 --n 9600 --steps 3 --warmup 2 2>&1 | tail -1 | cut -c1-200
