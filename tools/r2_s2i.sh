#!/bin/bash
# full build: smoke + GPU parity, then bench / profiles (r2_s2g.sh)
mkdir -p gpurun_out
T=${TAG:-r2s2i}
timeout 300 python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_smoke.txt 2>&1
echo "smoke rc=$?" >> gpurun_out/${T}_smoke.txt
timeout 1500 python -m pytest tests -m "gpu and not slow" -x -q --timeout 600 > gpurun_out/${T}_pytest.txt 2>&1
echo "pytest rc=$?" >> gpurun_out/${T}_pytest.txt
TAG=$T bash tools/r2_s2g.sh
