set -x
timeout 600 ncu --section SourceCounters --section WarpStateStats --section SpeedOfLight --clock-control none --import-source on -k 'regex:^k_sched$' -c 1 -o gpurun_out/src19200_r02j python tools/profile_run.py 19200 sched > gpurun_out/ncu_r02j.log 2>&1; echo rc=$?
