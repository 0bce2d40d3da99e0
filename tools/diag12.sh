cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag12.log; : > $O
run() { echo "== $*" >> $O; timeout 200 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run DIAG_TIMEOUT=60 python tools/split_diag.py C2 0 5
run DIAG_TIMEOUT=60 python tools/split_diag.py C4 0 5
run DIAG_TIMEOUT=60 python tools/split_diag.py C4 8 5
run DIAG_TIMEOUT=60 python tools/split_diag.py C5 0 5
run DIAG_TIMEOUT=120 DIAG_N=16777216 python tools/split_diag.py C5 0 3
run DIAG_TIMEOUT=60 python tools/split_diag.py C1 0 5
grep "^C\|^==\|rc=" $O
