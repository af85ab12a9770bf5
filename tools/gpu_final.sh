# usage: bash tools/gpu_final.sh TAG (under gpurun): smoke, GPU parity, launch list + ncu captures of the dominant
#   kernels of one C2 BFS, the default bench line (cpu_baseline + e2e), the reference arm; text only under gpurun_out/
TAG=${1:-final}
mkdir -p gpurun_out
python -c "import __graft_entry__ as e; e.smoke()" 2>&1 | tail -2
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -3
bash tools/gpu_prof2.sh $TAG c2 "expand_kernel" 17 "bu_kernel" 18 "hub_kernel" 16 "commit_dense" 17 > gpurun_out/prof_$TAG.txt 2>&1
tail -5 gpurun_out/prof_$TAG.txt
timeout 900 python bench.py > gpurun_out/bench_$TAG.json 2> gpurun_out/bench_$TAG.err; tail -2 gpurun_out/bench_$TAG.err; cat gpurun_out/bench_$TAG.json
timeout 600 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/ref_$TAG.json 2> gpurun_out/ref_$TAG.err; cat gpurun_out/ref_$TAG.json
