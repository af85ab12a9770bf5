# usage: bash tools/gpu_prof.sh TAG KERNEL_REGEX SKIP [CONFIG]  (under gpurun)
#   launch list (time + DRAM bytes per launch) of one BFS, then one `ncu --set full` capture of KERNEL_REGEX
TAG=${1:-run}; KRE=${2:-expand_kernel}; SKIP=${3:-12}; CFG=${4:-c2}
mkdir -p gpurun_out
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/launches_$TAG.csv python tools/prof_bfs.py --config $CFG --reps 1 > gpurun_out/launches_$TAG.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled -k regex:"$KRE" -s $SKIP -c 1 \
  -o gpurun_out/prof_$TAG python tools/prof_bfs.py --config $CFG --reps 1 > gpurun_out/prof_$TAG.log 2>&1
tail -3 gpurun_out/prof_$TAG.log
