#!/bin/bash
mkdir -p gpurun_out
T=${TAG:-r2i}
TUNES=("bu_grow=0,bu_alpha=25" "dir_bits=1,bu_grow=0,alpha_bits=20" "dir_bits=1,bu_grow=0,alpha_bits=25" "dir_bits=1,bu_grow=0,alpha_bits=30" "dir_bits=1,alpha_bits=25")
timeout 600 python tools/sweep_tunes.py c2 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c2.txt 2>&1
timeout 800 python tools/sweep_tunes.py c3 8 "${TUNES[@]}" > gpurun_out/${T}_sweep_c3.txt 2>&1
timeout 1000 python tools/sweep_tunes.py c4 6 "${TUNES[@]}" > gpurun_out/${T}_sweep_c4.txt 2>&1
timeout 600 compute-sanitizer --tool racecheck --racecheck-report hazard python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_racecheck.txt 2>&1
echo "rc=$?" >> gpurun_out/${T}_racecheck.txt
timeout 600 compute-sanitizer --tool synccheck python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_synccheck.txt 2>&1
echo "rc=$?" >> gpurun_out/${T}_synccheck.txt
timeout 600 compute-sanitizer --tool memcheck python -c "import __graft_entry__ as e; e.smoke()" > gpurun_out/${T}_memcheck.txt 2>&1
echo "rc=$?" >> gpurun_out/${T}_memcheck.txt
