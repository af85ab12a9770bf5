# usage: bash tools/gpu_iter.sh TAG  (under gpurun): BFS parity tests, per-level traces of c2/c3, short bench
TAG=${1:-it}
mkdir -p gpurun_out
timeout 900 python -m pytest tests -m gpu -x -q -k "bfs or smoke or c2_full or degenerate or hub" 2>&1 | tail -8
timeout 300 python tools/trace_bfs.py c2 2 > gpurun_out/trace_c2_$TAG.log 2>&1; grep -v "^#" gpurun_out/trace_c2_$TAG.log | tail -32
timeout 300 python tools/trace_bfs.py c3 1 > gpurun_out/trace_c3_$TAG.log 2>&1; tail -14 gpurun_out/trace_c3_$TAG.log
timeout 600 python bench.py --steps 8 --warmup 3 --no-cpu-baseline > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err; tail -3 gpurun_out/bench_$TAG.err; cat gpurun_out/bench_$TAG.json
