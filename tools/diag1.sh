cd $GRAFT_REPO_ROOT 2>/dev/null || cd /root/repo
O=gpurun_out/diag1.log; : > $O
run() { echo "== $*" >> $O; timeout 150 env "$@" >> $O 2>&1 || echo "rc=$?" >> $O; }
run CULI_LIB=scratch/libculi_r1.so python tools/split_diag.py C2 0 5
run DUMMY=1 python tools/split_diag.py C2 0 5
run CULI_SPLIT_FIRST=2 python tools/split_diag.py C2 0 5
run CULI_LIB=scratch/libculi_r1.so python tools/split_diag.py C5 0 5
run DUMMY=1 python tools/split_diag.py C5 0 5
run CULI_WAIT_MS=2000 DIAG_N=2000 python tools/split_diag.py C5 1 3
run CULI_WAIT_MS=2000 DIAG_N=2000 python tools/split_diag.py C5 0 3
run CULI_LIB=scratch/libculi_r1.so python tools/split_diag.py C4 0 5
run DUMMY=1 python tools/split_diag.py C4 0 5
run DUMMY=1 python tools/split_diag.py C4 8 5
run DUMMY=1 python tools/split_diag.py C1 0 5
run DUMMY=1 python tools/split_diag.py C1 8 5
cat $O
