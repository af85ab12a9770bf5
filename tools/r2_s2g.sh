#!/bin/bash
# bench (default C4) + reference arm + C4 trace + launch list + ncu of the heaviest top-down / bottom-up levels
mkdir -p gpurun_out
T=${TAG:-r2s2g}
timeout 1500 python bench.py > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err
echo "bench rc=$?" >> gpurun_out/${T}_bench.err
timeout 900 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/${T}_ref.json 2> gpurun_out/${T}_ref.err
timeout 600 python tools/trace_bfs.py c4 2 > gpurun_out/${T}_trace_c4.txt 2>&1
read TDL BUL < <(python tools/pick_levels.py gpurun_out/${T}_trace_c4.txt)
echo "td=$TDL bu=$BUL" >> gpurun_out/${T}_trace_c4.txt
export GCGT_TUNE=graph=0
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_c4.csv python tools/prof_bfs.py --config c4 --reps 1 > gpurun_out/${T}_launches_c4.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_c4.csv --json gpurun_out/${T}_launches_c4.json > gpurun_out/${T}_launches_c4.txt 2>&1
bash tools/ncu_one.sh ${T}_exp_c4 expand_kernel $TDL c4
bash tools/ncu_one.sh ${T}_hub_c4 hub_flat_kernel $TDL c4
bash tools/ncu_one.sh ${T}_bu_c4 bu_kernel $BUL c4
# bottom-up variants: work counters of one BFS (same root) and an ncu capture of the flat kernel
for tune in "" "bu_flat=1"; do
  GCGT_TUNE="$tune" timeout 600 python tools/prof_bfs.py --config c4 --reps 2 > gpurun_out/${T}_stats_${tune:-default}.txt 2>&1
done
GCGT_TUNE=graph=0,bu_flat=1 bash tools/ncu_one.sh ${T}_buflat_c4 bu_flat_kernel $BUL c4
GCGT_TUNE=dir_edges=1,alpha_edges=140 timeout 600 python tools/trace_bfs.py c4 2 > gpurun_out/${T}_trace_c4_edges.txt 2>&1
GCGT_TUNE=dir_edges=1,alpha_edges=140 timeout 600 python tools/trace_bfs.py c3 2 > gpurun_out/${T}_trace_c3_edges.txt 2>&1
timeout 600 python tools/trace_bfs.py c3 2 > gpurun_out/${T}_trace_c3.txt 2>&1
