#!/bin/bash
# r2 session-2 pass b: C4 per-level trace, launch list (host-driven loop so ncu sees every kernel), ncu --set full of the
# heaviest top-down and bottom-up levels, then the full-size parity tests
mkdir -p gpurun_out
T=${TAG:-r2s2b}
timeout 600 python tools/trace_bfs.py c4 2 > gpurun_out/${T}_trace_c4.txt 2>&1
read TDL BUL < <(python tools/pick_levels.py gpurun_out/${T}_trace_c4.txt)
echo "td=$TDL bu=$BUL" >> gpurun_out/${T}_trace_c4.txt
export GCGT_TUNE=graph=0
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_c4.csv python tools/prof_bfs.py --config c4 --reps 1 > gpurun_out/${T}_launches_c4.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_c4.csv --json gpurun_out/${T}_launches_c4.json > gpurun_out/${T}_launches_c4.txt 2>&1
bash tools/ncu_one.sh ${T}_exp_c4 expand_kernel $TDL c4
bash tools/ncu_one.sh ${T}_bu_c4 bu_kernel $BUL c4
unset GCGT_TUNE
timeout 2400 python -m pytest tests/test_gpu_fullsize.py -m gpu -x -q --timeout 2400 -s > gpurun_out/${T}_fullsize.txt 2>&1
echo "fullsize rc=$?" >> gpurun_out/${T}_fullsize.txt
