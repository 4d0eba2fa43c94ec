mkdir -p gpurun_out
python tools/window_speed.py 48 65 128 129 256 1000 4096 > gpurun_out/g14_speed.txt 2>&1
ncu --set full --clock-control none -k regex:k1_bulk -s 2 -c 1 -o gpurun_out/prof_lw128 python tools/lw_once.py 128 > gpurun_out/g14_ncu.log 2>&1
python tools/ncu_summary.py gpurun_out/prof_lw128.ncu-rep > gpurun_out/g14_lw128.txt 2>&1
