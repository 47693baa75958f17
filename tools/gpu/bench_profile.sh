# bench line + ncu launch list + ncu --set full of k_sched at the bench sizes (round-2 profiles)
set -x
python bench.py > gpurun_out/bench.json 2> gpurun_out/bench.err; echo bench_rc=$?
python bench.py --impl reference > gpurun_out/bench_ref.json 2>> gpurun_out/bench.err; echo ref_rc=$?
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none -c 400 --csv --log-file gpurun_out/launches.csv python bench.py --steps 2 --warmup 3 --no-e2e --no-cpu-baseline --extra-n 0 > gpurun_out/bench_ncu.log 2>&1; echo ncu_list_rc=$?
timeout 900 ncu --set full --clock-control none --import-source on -k 'regex:^k_sched$' -c 1 -o gpurun_out/sched46080 python tools/profile_run.py 46080 sched > gpurun_out/ncu46080.log 2>&1; echo ncu46_rc=$?
timeout 600 ncu --set full --clock-control none --import-source on -k 'regex:^k_sched$' -c 1 -o gpurun_out/sched19200 python tools/profile_run.py 19200 sched > gpurun_out/ncu19200.log 2>&1; echo ncu19_rc=$?
