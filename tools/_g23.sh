timeout 300 ncu --metrics gpu__time_duration.sum,launch__grid_size,launch__block_size --clock-control none --csv --log-file gpurun_out/small_launches.csv python tools/small_profile.py > /dev/null 2>&1
tail -12 gpurun_out/small_launches.csv | cut -c1-300
