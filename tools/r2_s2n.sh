#!/bin/bash
# profiles of the current default on C4 (trace, launch list, ncu of the heaviest top-down / bottom-up / hub levels),
# app timings (BC on C3, CC on C2 / C4)
mkdir -p gpurun_out
T=${TAG:-r2s2n}
timeout 900 python tools/trace_bfs.py c4 2 > gpurun_out/${T}_trace_c4.txt 2>&1
read TDL BUL < <(python tools/pick_levels.py gpurun_out/${T}_trace_c4.txt)
echo "td=$TDL bu=$BUL" >> gpurun_out/${T}_trace_c4.txt
export GCGT_TUNE=graph=0
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_c4.csv python tools/prof_bfs.py --config c4 --reps 1 > gpurun_out/${T}_launches_c4.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_c4.csv --json gpurun_out/${T}_launches_c4.json > gpurun_out/${T}_launches_c4.txt 2>&1
bash tools/ncu_one.sh ${T}_exp_c4 expand_kernel $TDL c4
bash tools/ncu_one.sh ${T}_bu_c4 bu_kernel $BUL c4
bash tools/ncu_one.sh ${T}_hub_c4 hub_kernel $TDL c4
unset GCGT_TUNE
timeout 1200 python tools/bench_apps.py bc c3 8 > gpurun_out/${T}_app_bc_c3.json 2> gpurun_out/${T}_app_bc_c3.err
timeout 900 python tools/bench_apps.py cc c2 5 > gpurun_out/${T}_app_cc_c2.json 2> gpurun_out/${T}_app_cc_c2.err
timeout 1500 python tools/bench_apps.py cc c4 3 > gpurun_out/${T}_app_cc_c4.json 2> gpurun_out/${T}_app_cc_c4.err
timeout 900 python tools/bench_apps.py bfs c3 8 > gpurun_out/${T}_app_bfs_c3.json 2> gpurun_out/${T}_app_bfs_c3.err
