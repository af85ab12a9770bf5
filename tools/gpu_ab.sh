# usage: bash tools/gpu_ab.sh TAG "TUNE_A" "TUNE_B" ...  (under gpurun): GPU parity tests, then per tuning string a
#   per-level trace summary of c2 and c3 (1 root) and a short bench, all text under gpurun_out/
TAG=$1; shift
mkdir -p gpurun_out
[ -n "$NOTEST" ] || timeout 900 python -m pytest tests -m gpu -x -q 2>&1 | tail -4
for T in "$@"; do
  echo "== GCGT_TUNE=$T"
  GCGT_TUNE=$T timeout 300 python tools/trace_bfs.py c2 2 > gpurun_out/trace_c2_${TAG}_${T//[=,]/_}.log 2>&1
  grep spans gpurun_out/trace_c2_${TAG}_${T//[=,]/_}.log | cut -c1-200
  GCGT_TUNE=$T timeout 300 python tools/trace_bfs.py c3 1 > gpurun_out/trace_c3_${TAG}_${T//[=,]/_}.log 2>&1
  grep spans gpurun_out/trace_c3_${TAG}_${T//[=,]/_}.log | cut -c1-200
  [ -n "$NOBENCH" ] || GCGT_TUNE=$T timeout 600 python bench.py --steps 16 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/bench_${TAG}_${T//[=,]/_}.json 2> gpurun_out/bench_${TAG}.err
  [ -n "$NOBENCH" ] || python -c "import json,sys; d=json.load(open(sys.argv[1])); print('bench', d['value'], 'GTEPS', d['ms_per_step'], 'ms', 'frac', d['roofline']['frac'], d['clocks'])" gpurun_out/bench_${TAG}_${T//[=,]/_}.json
done
