cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag11.log; : > $O
run() { echo "== $*" >> $O; timeout 100 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run CULI_SPLIT_STATS=1 DIAG_TIMEOUT=60 python tools/split_diag.py C2 0 5
run CULI_SPLIT_STATS=1 DIAG_TIMEOUT=60 CULI_STEAL_GATE=0 python tools/split_diag.py C2 0 3
run DIAG_TIMEOUT=60 python tools/split_diag.py C5 0 5
run DIAG_TIMEOUT=60 DIAG_N=5000 python tools/split_diag.py C5 1 10
run DIAG_TIMEOUT=60 DIAG_N=2000 python tools/split_diag.py C5 1 10
run DIAG_TIMEOUT=60 python tools/split_diag.py C4 0 3
grep "^C\|^==\|rc=\|culi split" $O
