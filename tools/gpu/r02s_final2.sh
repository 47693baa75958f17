# final validation after the solve change: smoke, GPU tests, bench line, reference arm
export PYTHONUNBUFFERED=1
python -c "import __graft_entry__ as g; g.smoke()" > gpurun_out/smoke_final2.log 2>&1; echo smoke_rc=$?
timeout 1200 python -m pytest tests -m gpu -x -q > gpurun_out/pytest_gpu_final2.log 2>&1; echo pytest_rc=$?
python bench.py > gpurun_out/bench_final2.json 2> gpurun_out/bench_final2.err; echo bench_rc=$?
