# usage: bash tools/gpu_prof2.sh TAG CONFIG [KRE SKIP]... (under gpurun)
#   launch list (time + DRAM bytes per launch) of one BFS, then one `ncu --set full` capture per (regex, skip) pair,
#   each summarised on the box (ncu_brief + srcprof) so only text travels back
TAG=$1; CFG=$2; shift 2
mkdir -p gpurun_out
timeout 900 ncu --metrics gpu__time_duration.sum,dram__bytes_read.sum,dram__bytes_write.sum --clock-control none --csv \
  --log-file gpurun_out/launches_$TAG.csv python tools/prof_bfs.py --config $CFG --reps 1 > gpurun_out/launches_$TAG.log 2>&1
python tools/launches.py gpurun_out/launches_$TAG.csv --json gpurun_out/launches_$TAG.json | head -20
i=0
while [ $# -ge 2 ]; do
  KRE=$1; SKIP=$2; shift 2; i=$((i+1))
  timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled -k regex:"$KRE" -s $SKIP -c 1 \
    -o /tmp/prof_${TAG}_$i python tools/prof_bfs.py --config $CFG --reps 1 > gpurun_out/prof_${TAG}_$i.log 2>&1
  tail -2 gpurun_out/prof_${TAG}_$i.log
  python tools/ncu_brief.py /tmp/prof_${TAG}_$i.ncu-rep > gpurun_out/ncu_${TAG}_$i.txt 2>&1
  python tools/srcprof.py /tmp/prof_${TAG}_$i.ncu-rep 50 > gpurun_out/src_${TAG}_$i.txt 2>&1
  head -45 gpurun_out/ncu_${TAG}_$i.txt
done
