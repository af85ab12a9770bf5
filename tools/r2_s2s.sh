#!/bin/bash
# BC on C3: launch list of one source (which kernel takes the 1 s)
mkdir -p gpurun_out
T=${TAG:-r2s2s}
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/${T}_launches_bc_c3.csv python tools/prof_bfs.py --config c3 --reps 1 --app bc --bc-sources 1 > gpurun_out/${T}_launches_bc_c3.log 2>&1
python tools/launches.py gpurun_out/${T}_launches_bc_c3.csv --json gpurun_out/${T}_launches_bc_c3.json > gpurun_out/${T}_launches_bc_c3.txt 2>&1
python tools/launches.py gpurun_out/${T}_launches_bc_c3.csv --seq > gpurun_out/${T}_launches_bc_c3_seq.txt 2>&1
