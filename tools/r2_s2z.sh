#!/bin/bash
# final records at HEAD: smoke, every GPU test (incl. full-size), C4 launch list + ncu of the heaviest levels
mkdir -p gpurun_out
T=${TAG:-r2s2z}
timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
echo "smoke rc=$?" >> gpurun_out/${T}_smoke.txt
timeout 2400 python -m pytest tests -m gpu -q --timeout 2400 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 900 python tools/trace_bfs.py c4 2 > gpurun_out/${T}_trace_c4.txt 2>&1
read TDL BUL < <(python tools/pick_levels.py gpurun_out/${T}_trace_c4.txt)
echo "td=$TDL bu=$BUL" >> gpurun_out/${T}_trace_c4.txt
export GCGT_TUNE=graph=0
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_c4.csv python tools/prof_bfs.py --config c4 --reps 1 > gpurun_out/${T}_launches_c4.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_c4.csv --json gpurun_out/${T}_launches_c4.json > gpurun_out/${T}_launches_c4.txt 2>&1
bash tools/ncu_one.sh ${T}_bu_c4 bu_kernel $BUL c4
bash tools/ncu_one.sh ${T}_exp_c4 expand_kernel $TDL c4
