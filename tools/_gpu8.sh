mkdir -p gpurun_out
ncu --metrics gpu__time_duration.sum,sm__cycles_active.avg,launch__grid_size --clock-control none -c 60 --csv --log-file gpurun_out/small_launches.csv python tools/small_profile.py > /dev/null 2>&1
ncu --set full --clock-control none --import-source on -k regex:k1_bulk -s 20 -c 1 -o gpurun_out/prof_small python tools/small_profile.py > /dev/null 2>&1
python tools/ncu_summary.py gpurun_out/prof_small.ncu-rep > gpurun_out/small_ncu.txt 2>&1
