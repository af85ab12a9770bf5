# usage (under gpurun): bash tools/ncu_one.sh TAG KERNEL_REGEX SKIP CONFIG  — one `ncu --set full` capture of the
# (SKIP+1)-th launch of KERNEL_REGEX in one BFS of CONFIG; keeps only text summaries (brief metrics + source lines)
TAG=$1; KRE=$2; SKIP=$3; CFG=${4:-c2}; APP=${5:-bfs}
mkdir -p gpurun_out
timeout 900 ncu --set full --clock-control none --import-source on --kernel-name-base demangled -k regex:"$KRE" -s $SKIP -c 1 \
  -o /tmp/prof_$TAG python tools/prof_bfs.py --config $CFG --reps 1 --app $APP > gpurun_out/prof_$TAG.log 2>&1
python tools/ncu_brief.py /tmp/prof_$TAG.ncu-rep > gpurun_out/ncu_$TAG.txt 2>&1
python tools/srcprof.py /tmp/prof_$TAG.ncu-rep 45 > gpurun_out/ncu_${TAG}_src.txt 2>&1
