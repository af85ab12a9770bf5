# session-4 verification after the bu_beta default change (run under gpurun): smoke, GPU parity, bench C2 line,
# C4 (uk-2007-like) beta check and bench line; text only under gpurun_out/
mkdir -p gpurun_out
python -c "import __graft_entry__ as e; e.smoke()" 2>&1 | tail -2
timeout 1200 python -m pytest tests -m gpu -x -q 2>&1 | tail -3
timeout 900 python bench.py > gpurun_out/bench_s4v.json 2> gpurun_out/bench_s4v.err; tail -2 gpurun_out/bench_s4v.err; cat gpurun_out/bench_s4v.json
timeout 900 python tools/sweep.py c4 bu_beta=24 bu_beta=128 > gpurun_out/sw_c4.txt 2>&1; cat gpurun_out/sw_c4.txt
timeout 900 python bench.py --config c4 --steps 4 --warmup 3 --no-cpu-baseline --no-e2e > gpurun_out/bench_s4v_c4.json 2> gpurun_out/bench_s4v_c4.err; tail -2 gpurun_out/bench_s4v_c4.err; cat gpurun_out/bench_s4v_c4.json
