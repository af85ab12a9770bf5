#!/bin/bash
# final build: smoke, every GPU test, bench (C4) + reference arm
mkdir -p gpurun_out
T=${TAG:-r2s2ac}
timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
echo "smoke rc=$?" >> gpurun_out/${T}_smoke.txt
timeout 2400 python -m pytest tests -m gpu -q --timeout 2400 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
timeout 1500 python bench.py > gpurun_out/${T}_bench.json 2> gpurun_out/${T}_bench.err
echo "bench rc=$?" >> gpurun_out/${T}_bench.err
timeout 900 python bench.py --impl reference --steps 2 --warmup 1 > gpurun_out/${T}_ref.json 2> gpurun_out/${T}_ref.err
