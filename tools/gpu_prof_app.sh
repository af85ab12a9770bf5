# usage: bash tools/gpu_prof_app.sh TAG APP CONFIG KERNEL_REGEX SKIP   (under gpurun): one ncu --set full capture
TAG=$1; APP=$2; CFG=$3; KRE=$4; SKIP=$5
mkdir -p gpurun_out
timeout 1200 ncu --set full --clock-control none --import-source on --kernel-name-base demangled -k regex:"$KRE" -s $SKIP -c 1 \
  -o gpurun_out/prof_$TAG python tools/prof_bfs.py --config $CFG --app $APP --reps 1 > gpurun_out/prof_$TAG.log 2>&1
ncu -i gpurun_out/prof_$TAG.ncu-rep --page raw --csv > gpurun_out/prof_${TAG}_raw.csv 2>/dev/null
tail -2 gpurun_out/prof_$TAG.log
